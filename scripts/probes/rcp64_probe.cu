// Accuracy of the fp64 reciprocal forms: rcp.approx.ftz.f64 seed, seed + two
// Newton steps (product), seed + one cubic step r0 (1 + e + e^2) (experiment),
// against IEEE division, over 2^26 random inputs spanning [2^-30, 2^30).
#include <cstdio>
#include <cstdint>
#include <cstring>
#include <cuda_runtime.h>
__device__ double seed(double x) { double r; asm("rcp.approx.ftz.f64 %0, %1;" : "=d"(r) : "d"(x)); return r; }
__device__ double newton2(double x) {
    double r = seed(x), e = fma(-x, r, 1.0);
    r = fma(r, e, r); e = fma(-x, r, 1.0); return fma(r, e, r);
}
__device__ double cubic(double x) { double r = seed(x), e = fma(-x, r, 1.0); return fma(r, fma(e, e, e), r); }
__device__ unsigned long long h(unsigned long long z) {
    z += 0x9E3779B97F4A7C15ull; z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
    z = (z ^ (z >> 27)) * 0x94D049BB133111EBull; return z ^ (z >> 31);
}
__global__ void k(unsigned long long *out, long n) {
    double m[3] = {0, 0, 0};
    for (long i = blockIdx.x * (long)blockDim.x + threadIdx.x; i < n; i += (long)gridDim.x * blockDim.x) {
        const unsigned long long u = h(i);
        const double mant = 1.0 + double(u >> 12) * 0x1p-52;
        const double x = ldexp(mant, int((u & 63) - 30)) * ((u >> 6) & 1 ? -1.0 : 1.0);
        const double ref = 1.0 / x;
        const double v[3] = {seed(x), newton2(x), cubic(x)};
        for (int q = 0; q < 3; ++q) m[q] = fmax(m[q], fabs((v[q] - ref) / ref));
    }
    for (int q = 0; q < 3; ++q) atomicMax(out + q, (unsigned long long)__double_as_longlong(m[q]));
}
int main() {
    unsigned long long *d, hbuf[3];
    cudaMalloc(&d, 24); cudaMemset(d, 0, 24);
    k<<<148 * 8, 256>>>(d, 1L << 26);
    cudaMemcpy(hbuf, d, 24, cudaMemcpyDeviceToHost);
    const char *nm[3] = {"seed rcp.approx.ftz.f64", "seed + 2 Newton (product)", "seed + cubic (experiment)"};
    for (int q = 0; q < 3; ++q) {
        double v; memcpy(&v, &hbuf[q], 8);
        printf("%-28s max rel err %.3e (%.1f ulp of 2^-53)\n", nm[q], v, v / 0x1p-53);
    }
    return 0;
}
