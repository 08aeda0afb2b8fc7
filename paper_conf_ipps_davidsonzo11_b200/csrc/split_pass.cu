// split_pass.cu -- G1: one HBM pass of k_p fused global PCR splitting levels.
//
// Paper: Stage 2 "splits one system with PCR ... until each subsystem fits in
// shared memory" in one kernel call (§III-B); Stage 1
// splits one system cooperatively with several processors (§III-C,
// P:L474-493).  Here both are the same kernel: `segs` CTAs cooperate on one
// system (segs > 1: stage 1, several blocks per system; segs == 1: stage 2),
// each CTA walking a contiguous range of tiles.  Unlike the paper's stage 1
// (one level per launch because of the global dependency), a tile carries a
// (2^k_p - 1)-row halo on each side, so k_p levels are fused into one pass
// over HBM with no inter-CTA synchronisation.
//
// Per tile: load rows [t0-H, t0+TILE+H) (rows outside [0, L) are identity
// rows), normalise (b = 1) on the first pass, run k_p PCR levels in shared
// memory, and write the TILE valid rows DE-INTERLEAVED: residue rho = i mod
// 2^k_p of slot sigma goes to output slot (sigma << k_p) + rho, position
// i >> k_p, so every subsystem is contiguous for the next stage.
#include "common.cuh"

namespace tds {


template <typename T, bool RAW, int QMAX>
__global__ void __launch_bounds__(512) split_pass_kernel(const SplitArgs<T> A) {
    extern __shared__ __align__(16) unsigned char smem_raw[];
    T *sa = reinterpret_cast<T *>(smem_raw);
    T *sc = sa + A.ep;
    T *sd = sc + A.ep;
    const int tid = threadIdx.x;
    const int NT = blockDim.x;
    const int kp = A.kp;
    const int H = (1 << kp) - 1;
    const int TILE = A.tile;
    const int E = TILE + 2 * H;
    const int ps = kp > 5 ? kp : 5;  // smem padding shift: index + (index >> ps)

    const int64_t sigma = int64_t(blockIdx.x) / A.segs;
    const int g = int(int64_t(blockIdx.x) % A.segs);
    int64_t L;
    const int kprev = RAW ? 0 : pass_levels(A.geom.npass, A.geom.kpass);
    if (RAW) {
        L = A.n;
    } else {
        const int64_t rho = sigma & ((int64_t(1) << kprev) - 1);
        const int64_t r = rho;
        L = r < A.n ? (A.n - r + (int64_t(1) << kprev) - 1) >> kprev : 0;
    }
    const int64_t in_base = sigma * A.in_stride;
    const int64_t ntiles = (L + TILE - 1) / TILE;
    const int64_t t_begin = g * ntiles / A.segs;
    const int64_t t_end = (g + 1) * ntiles / A.segs;
    const int per_res_shift = __ffs(TILE) - 1 - kp;  // log2(TILE >> kp)
    const int per_res_mask = (1 << per_res_shift) - 1;

    for (int64_t ti = t_begin; ti < t_end; ++ti) {
        const int64_t t0 = ti * TILE;
        // ---- load tile + halo, normalise on the first pass
        for (int e = tid; e < E; e += NT) {
            const int64_t row = t0 - H + e;
            T va = T(0), vc = T(0), vd = T(0);
            if (row >= 0 && row < L) {
                const int64_t o = in_base + row;
                if (RAW) {
                    const T rb = rcp(A.b[o]);
                    va = (row > 0 ? A.a[o] : T(0)) * rb;
                    vc = (row < L - 1 ? A.c[o] : T(0)) * rb;
                    vd = A.d[o] * rb;
                } else {
                    va = A.a[o];
                    vc = A.c[o];
                    vd = A.d[o];
                }
            }
            const int pe = e + (e >> ps);
            sa[pe] = va;
            sc[pe] = vc;
            sd[pe] = vd;
        }
        __syncthreads();
        // ---- k_p PCR levels (strides 1, 2, ..., 2^(k_p-1)) in shared memory
        for (int j = 0; j < kp; ++j) {
            const int s = 1 << j;
            T na[QMAX], nc[QMAX], nd[QMAX];
#pragma unroll
            for (int q = 0; q < QMAX; ++q) {
                const int e = tid + q * NT;
                if (e >= s && e < E - s) {
                    const int pl = (e - s) + ((e - s) >> ps);
                    const int pm = e + (e >> ps);
                    const int pr = (e + s) + ((e + s) >> ps);
                    T a = sa[pm], c = sc[pm], d = sd[pm];
                    row_update(a, c, d, sa[pl], sc[pl], sd[pl], sa[pr], sc[pr], sd[pr]);
                    na[q] = a;
                    nc[q] = c;
                    nd[q] = d;
                }
            }
            __syncthreads();
#pragma unroll
            for (int q = 0; q < QMAX; ++q) {
                const int e = tid + q * NT;
                if (e >= s && e < E - s) {
                    const int pm = e + (e >> ps);
                    sa[pm] = na[q];
                    sc[pm] = nc[q];
                    sd[pm] = nd[q];
                }
            }
            __syncthreads();
        }
        // ---- de-interleaved write: consecutive threads -> consecutive j of one residue
        const int64_t valid = (L - t0 < TILE) ? (L - t0) : TILE;
        for (int o = tid; o < TILE; o += NT) {
            const int rr = o >> per_res_shift;
            const int jj = o & per_res_mask;
            const int q = rr + (jj << kp);
            if (q < valid) {
                const int e = H + q;
                const int pe = e + (e >> ps);
                const int64_t oidx = out_slot_index(sigma, kprev, kp, rr) * A.out_slot + (t0 >> kp) + jj;
                A.oa[oidx] = sa[pe];
                A.oc[oidx] = sc[pe];
                A.od[oidx] = sd[pe];
            }
        }
        __syncthreads();
    }
}

template <typename T, bool RAW, int Q>
static cudaError_t launch_q(const SplitArgs<T> &A, int64_t grid, int threads, size_t smem, cudaStream_t st) {
    auto kern = split_pass_kernel<T, RAW, Q>;
    cudaError_t e = cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    if (e != cudaSuccess) return e;
    kern<<<(unsigned)grid, threads, smem, st>>>(A);
    return cudaGetLastError();
}

template <typename T>
cudaError_t launch_split_pass(const SplitArgs<T> &A, bool raw, int64_t grid, int threads, size_t smem,
                              cudaStream_t st) {
    const int E = A.tile + 2 * ((1 << A.kp) - 1);
    const int q = (E + threads - 1) / threads;
    if (q <= 8) return raw ? launch_q<T, true, 8>(A, grid, threads, smem, st) : launch_q<T, false, 8>(A, grid, threads, smem, st);
    if (q <= 16) return raw ? launch_q<T, true, 16>(A, grid, threads, smem, st) : launch_q<T, false, 16>(A, grid, threads, smem, st);
    if (q <= 24) return raw ? launch_q<T, true, 24>(A, grid, threads, smem, st) : launch_q<T, false, 24>(A, grid, threads, smem, st);
    return cudaErrorInvalidConfiguration;
}

template cudaError_t launch_split_pass<float>(const SplitArgs<float> &, bool, int64_t, int, size_t, cudaStream_t);
template cudaError_t launch_split_pass<double>(const SplitArgs<double> &, bool, int64_t, int, size_t, cudaStream_t);

}  // namespace tds
