// Microbenchmark: issue rate of FFMA vs FFMA2 (packed fp32x2) on sm_100a.
#include <cstdio>
#include <cuda_runtime.h>
template <int MODE>
__global__ void k(float *out, float s, int iters) {
    float a[8], b[8];
    for (int i = 0; i < 8; ++i) { a[i] = threadIdx.x * 1e-3f + i; b[i] = s + i; }
    for (int it = 0; it < iters; ++it) {
        if constexpr (MODE == 0) {
#pragma unroll
            for (int i = 0; i < 8; ++i) a[i] = fmaf(a[i], b[i], s);
#pragma unroll
            for (int i = 0; i < 8; ++i) b[i] = fmaf(b[i], a[i], s);
        } else {
#pragma unroll
            for (int i = 0; i < 8; i += 2) {
                float2 r = __ffma2_rn(make_float2(a[i], a[i + 1]), make_float2(b[i], b[i + 1]), make_float2(s, s));
                a[i] = r.x; a[i + 1] = r.y;
            }
#pragma unroll
            for (int i = 0; i < 8; i += 2) {
                float2 r = __ffma2_rn(make_float2(b[i], b[i + 1]), make_float2(a[i], a[i + 1]), make_float2(s, s));
                b[i] = r.x; b[i + 1] = r.y;
            }
        }
    }
    float acc = 0;
    for (int i = 0; i < 8; ++i) acc += a[i] + b[i];
    out[blockIdx.x * blockDim.x + threadIdx.x] = acc;
}
int main() {
    float *o;
    cudaMalloc(&o, 148 * 8 * 1024 * 4);
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0); cudaEventCreate(&e1);
    const int iters = 20000;
    for (int mode = 0; mode < 2; ++mode) {
        for (int rep = 0; rep < 2; ++rep) {
            cudaEventRecord(e0);
            if (mode == 0) k<0><<<148 * 4, 512>>>(o, 0.999f, iters); else k<1><<<148 * 4, 512>>>(o, 0.999f, iters);
            cudaEventRecord(e1);
            cudaEventSynchronize(e1);
            float ms; cudaEventElapsedTime(&ms, e0, e1);
            double flops = 2.0 * 16 * iters * 148.0 * 4 * 512;
            if (rep) printf("mode %s: %.3f ms  %.1f TFLOP/s fp32\n", mode ? "FFMA2" : "FFMA", ms, flops / ms / 1e9);
        }
    }
    return 0;
}
