// Microbenchmark: per-SM issue rates of the instruction classes the split
// kernel is made of (FFMA, FFMA2, MUFU.RCP, SHFL, LDS.128, STS.128) and of
// mixes of them, at 16 and 32 warps per SM (one CTA per SM).  Output:
// warp-instructions per SM clock for the measured class.
//   nvcc -O3 -gencode arch=compute_100a,code=sm_100a pipe_rates.cu -o pipe_rates
#include <cstdio>
#include <cuda_runtime.h>

constexpr int ITERS = 4096;

template <int MODE>
__global__ void k(float *out, float s, long long *cyc) {
    __shared__ float4 sm[1024 * 2];
    float a[8], b[8];
    for (int i = 0; i < 8; ++i) {
        a[i] = threadIdx.x * 1e-3f + i + 1.f;
        b[i] = s + i;
    }
    double x[8], y[8];
    for (int i = 0; i < 8; ++i) {
        x[i] = a[i];
        y[i] = b[i];
    }
    for (int i = threadIdx.x; i < 2048; i += blockDim.x) sm[i] = make_float4(s, s, s, s);
    __syncthreads();
    long long t0 = clock64();
    for (int it = 0; it < ITERS; ++it) {
        if constexpr (MODE == 0) {  // FFMA 3-reg: 16 per iter
#pragma unroll
            for (int i = 0; i < 8; ++i) a[i] = fmaf(a[i], b[i], b[(i + 1) & 7]);
#pragma unroll
            for (int i = 0; i < 8; ++i) b[i] = fmaf(b[i], a[i], a[(i + 1) & 7]);
        } else if constexpr (MODE == 1) {  // FFMA2: 8 per iter
#pragma unroll
            for (int i = 0; i < 8; i += 2) {
                float2 r = __ffma2_rn(make_float2(a[i], a[i + 1]), make_float2(b[i], b[i + 1]),
                                      make_float2(b[(i + 2) & 7], b[(i + 3) & 7]));
                a[i] = r.x;
                a[i + 1] = r.y;
            }
#pragma unroll
            for (int i = 0; i < 8; i += 2) {
                float2 r = __ffma2_rn(make_float2(b[i], b[i + 1]), make_float2(a[i], a[i + 1]),
                                      make_float2(a[(i + 2) & 7], a[(i + 3) & 7]));
                b[i] = r.x;
                b[i + 1] = r.y;
            }
        } else if constexpr (MODE == 2) {  // MUFU.RCP: 16 per iter
#pragma unroll
            for (int i = 0; i < 8; ++i) asm volatile("rcp.approx.ftz.f32 %0, %1;" : "=f"(a[i]) : "f"(a[i] + b[i]));
#pragma unroll
            for (int i = 0; i < 8; ++i) asm volatile("rcp.approx.ftz.f32 %0, %1;" : "=f"(b[i]) : "f"(b[i] + a[i]));
        } else if constexpr (MODE == 3) {  // SHFL down: 16 per iter
#pragma unroll
            for (int i = 0; i < 8; ++i) a[i] = __shfl_down_sync(0xffffffffu, a[i], 1) ;
#pragma unroll
            for (int i = 0; i < 8; ++i) b[i] = __shfl_up_sync(0xffffffffu, b[i], 1);
        } else if constexpr (MODE == 4) {  // LDS.128: 8 per iter (conflict-free)
#pragma unroll
            for (int i = 0; i < 8; ++i) {
                float4 v = sm[(threadIdx.x + 32 * i + int(a[i & 7]) ) & 2047];
                a[i] += v.x + v.z;
                b[i] += v.y * v.w;
            }
        } else if constexpr (MODE == 5) {  // STS.128: 8 per iter
#pragma unroll
            for (int i = 0; i < 8; ++i) sm[(threadIdx.x + 32 * i + it) & 2047] = make_float4(a[i], b[i], a[i], b[i]);
        } else if constexpr (MODE == 6) {  // mix per 2 rows: 4.5 FFMA2 : 2 MUFU (the row update)
#pragma unroll
            for (int i = 0; i < 8; i += 2) {
                float2 d = __ffma2_rn(make_float2(a[i], a[i + 1]), make_float2(b[i], b[i + 1]), make_float2(s, s));
                float r0, r1;
                asm volatile("rcp.approx.ftz.f32 %0, %1;" : "=f"(r0) : "f"(d.x));
                asm volatile("rcp.approx.ftz.f32 %0, %1;" : "=f"(r1) : "f"(d.y));
                float2 r = make_float2(r0, r1);
                float2 m = __fmul2_rn(make_float2(a[i], a[i + 1]), r);
                float2 n = __ffma2_rn(m, make_float2(b[i], b[i + 1]), r);
                float2 q = __ffma2_rn(n, m, d);
                a[i] = q.x;
                a[i + 1] = q.y;
                b[i] = n.x;
                b[i + 1] = n.y;
            }
        } else if constexpr (MODE == 8) {  // FMUL: 16 per iter
#pragma unroll
            for (int i = 0; i < 8; ++i) a[i] = a[i] * b[(i + 1) & 7];
#pragma unroll
            for (int i = 0; i < 8; ++i) b[i] = b[i] * a[(i + 1) & 7];
        } else if constexpr (MODE == 9) {  // FMUL2: 8 per iter
#pragma unroll
            for (int i = 0; i < 8; i += 2) {
                float2 r = __fmul2_rn(make_float2(a[i], a[i + 1]), make_float2(b[(i + 2) & 7], b[(i + 3) & 7]));
                a[i] = r.x;
                a[i + 1] = r.y;
            }
#pragma unroll
            for (int i = 0; i < 8; i += 2) {
                float2 r = __fmul2_rn(make_float2(b[i], b[i + 1]), make_float2(a[(i + 2) & 7], a[(i + 3) & 7]));
                b[i] = r.x;
                b[i + 1] = r.y;
            }
        } else if constexpr (MODE == 10) {  // FFMA with an immediate addend: 16 per iter
#pragma unroll
            for (int i = 0; i < 8; ++i) a[i] = fmaf(a[i], b[i], 1.0f);
#pragma unroll
            for (int i = 0; i < 8; ++i) b[i] = fmaf(b[i], a[i], 1.0f);
        } else if constexpr (MODE == 11) {  // STS.32 conflict-free: 16 per iter
#pragma unroll
            for (int i = 0; i < 16; ++i) reinterpret_cast<float *>(sm)[(threadIdx.x + 32 * i + it) & 8191] = a[i & 7];
        } else if constexpr (MODE == 12) {  // mix: 16 FFMA (3-reg, ~24 SMSP cycles) + 6 STS.32 (6 SM cycles)
#pragma unroll
            for (int i = 0; i < 8; ++i) a[i] = fmaf(a[i], b[i], b[(i + 1) & 7]);
#pragma unroll
            for (int i = 0; i < 6; ++i) reinterpret_cast<float *>(sm)[(threadIdx.x + 32 * i + it) & 8191] = a[i];
#pragma unroll
            for (int i = 0; i < 8; ++i) b[i] = fmaf(b[i], a[i], a[(i + 1) & 7]);
        } else if constexpr (MODE == 13) {  // mix: 16 FFMA (3-reg) + 1 LDS.128 (4 SM cycles)
#pragma unroll
            for (int i = 0; i < 8; ++i) a[i] = fmaf(a[i], b[i], b[(i + 1) & 7]);
            {
                float4 v = sm[(threadIdx.x + int(a[0])) & 2047];
                a[1] += v.x + v.z;
                b[1] += v.y * v.w;
            }
#pragma unroll
            for (int i = 0; i < 8; ++i) b[i] = fmaf(b[i], a[i], a[(i + 1) & 7]);
        } else if constexpr (MODE == 14) {  // DFMA: 16 per iter
#pragma unroll
            for (int i = 0; i < 8; ++i) x[i] = fma(x[i], y[i], y[(i + 1) & 7]);
#pragma unroll
            for (int i = 0; i < 8; ++i) y[i] = fma(y[i], x[i], x[(i + 1) & 7]);
        } else if constexpr (MODE == 15) {  // DMUL: 16 per iter
#pragma unroll
            for (int i = 0; i < 8; ++i) x[i] = x[i] * y[(i + 1) & 7];
#pragma unroll
            for (int i = 0; i < 8; ++i) y[i] = y[i] * x[(i + 1) & 7];
        } else if constexpr (MODE == 16) {  // MUFU.RCP64H: 16 per iter
#pragma unroll
            for (int i = 0; i < 8; ++i) asm volatile("rcp.approx.ftz.f64 %0, %1;" : "=d"(x[i]) : "d"(x[i]));
#pragma unroll
            for (int i = 0; i < 8; ++i) asm volatile("rcp.approx.ftz.f64 %0, %1;" : "=d"(y[i]) : "d"(y[i]));
        } else if constexpr (MODE == 7) {  // SHFL + FFMA2 mix (6 shfl : 9 FFMA2)
#pragma unroll
            for (int i = 0; i < 6; ++i) a[i] = __shfl_down_sync(0xffffffffu, a[i], 1);
#pragma unroll
            for (int j = 0; j < 9; ++j) {
                const int i = (2 * j) & 7;
                float2 r = __ffma2_rn(make_float2(b[i], b[i + 1]), make_float2(a[(i + 6) & 7], a[(i + 7) & 7]),
                                      make_float2(s, s));
                b[i] = r.x;
                b[i + 1] = r.y;
            }
        }
    }
    long long t1 = clock64();
    float acc = 0;
    for (int i = 0; i < 8; ++i) acc += a[i] + b[i] + float(x[i] + y[i]);
    __syncthreads();
    acc += sm[(threadIdx.x * 7) & 2047].z;
    out[blockIdx.x * blockDim.x + threadIdx.x] = acc;
    if (threadIdx.x == 0) cyc[blockIdx.x] = t1 - t0;
}

template <int MODE>
void run(const char *name, double per_iter, int threads, float *o, long long *c) {
    k<MODE><<<148, threads>>>(o, 0.999f, c);
    k<MODE><<<148, threads>>>(o, 0.999f, c);
    cudaDeviceSynchronize();
    long long h[148];
    cudaMemcpy(h, c, sizeof(h), cudaMemcpyDeviceToHost);
    double mx = 0;
    for (int i = 0; i < 148; ++i) mx = h[i] > mx ? h[i] : mx;
    const double warps = threads / 32.0;
    printf("%-28s warps/SM %2d: %.3f warp-instr per SM clock (%.2f cycles per warp-instr per SMSP)\n", name,
           int(warps), per_iter * ITERS * warps / mx, mx / (per_iter * ITERS * warps / 4.0));
}

int main() {
    float *o;
    long long *c;
    cudaMalloc(&o, 148 * 1024 * 4);
    cudaMalloc(&c, 148 * 8);
    for (int th : {512, 1024}) {
        run<0>("FFMA (3-reg)", 16, th, o, c);
        run<1>("FFMA2", 8, th, o, c);
        run<2>("MUFU.RCP", 16, th, o, c);
        run<3>("SHFL", 16, th, o, c);
        run<4>("LDS.128", 8, th, o, c);
        run<5>("STS.128", 8, th, o, c);
        run<6>("mix: 4 FFMA2/FMUL2 per 2 MUFU (count MUFU)", 8, th, o, c);
        run<7>("mix: 6 SHFL per 9 FFMA2 (count SHFL)", 6, th, o, c);
        run<8>("FMUL", 16, th, o, c);
        run<9>("FMUL2", 8, th, o, c);
        run<10>("FFMA imm addend", 16, th, o, c);
        run<11>("STS.32", 16, th, o, c);
        run<12>("mix 16 FFMA + 6 STS.32 (count FFMA)", 16, th, o, c);
        run<13>("mix 16 FFMA + 1 LDS.128 (count FFMA)", 16, th, o, c);
        run<14>("DFMA", 16, th, o, c);
        run<15>("DMUL", 16, th, o, c);
        run<16>("MUFU.RCP64H", 16, th, o, c);
    }
    cudaError_t e = cudaGetLastError();
    printf("err: %s\n", cudaGetErrorString(e));
    return 0;
}
