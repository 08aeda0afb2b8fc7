// split_pipe.cu -- G1, persistent TMA-prefetched form of the register split
// kernel (k_p <= 4 fused PCR levels per HBM pass; §III-B/C).
//
// Work items are tiles (slot sigma, tile ti) of 16*(NT-2) output rows; a
// resident CTA walks items w = blockIdx.x, += gridDim.x.  Each CTA owns ONE
// shared-memory stage holding the next tile's input rows (4 raw arrays on the
// first pass, 3 normalised ones after): as soon as every thread has copied the
// current tile into registers the stage is refilled with cp.async.bulk (the
// Tensor Memory Accelerator) while the CTA runs the PCR levels and the
// de-interleaved stores -- HBM reads of tile i+1 overlap compute on tile i.
// Levels and stores are those of split_reg.cu (reg_level / store_run), so the
// output is bit-identical.
#include "pipe.cuh"
#include "split_reg.cuh"

namespace tds {

template <typename T, int KP, bool RAW>
__global__ void __launch_bounds__(kRegSplitThreads, 2) split_pipe_kernel(const SplitArgs<T> A, int64_t tps,
                                                                       int64_t nitems) {
    constexpr int R = kRegSplitRows;
    constexpr int NT = kRegSplitThreads;
    constexpr int NW = NT / 32;
    constexpr int SM = 1 << (KP - 1);
    constexpr int NR = 1 << KP;
    constexpr int G = R >> KP;
    constexpr int NA = RAW ? 4 : 3;         // arrays streamed
    constexpr int ROWS = NT * R;            // rows per stage (tile + halo threads)
    constexpr int TV = ROWS - 2 * R;        // valid rows per tile
    extern __shared__ __align__(128) unsigned char smem_raw[];
    T *stage = reinterpret_cast<T *>(smem_raw);  // [NA][ROWS]
    __shared__ T eL[2][3][NW][SM];
    __shared__ T eR[2][3][NW][SM];
    __shared__ __align__(8) uint64_t bar;
    const int t = threadIdx.x, lane = t & 31, warp = t >> 5;
    const int kprev = RAW ? 0 : pass_levels(A.geom.npass, A.geom.kpass);

    auto slot_len = [&](int64_t sigma) -> int64_t {
        if (RAW) return A.n;
        const int64_t r = slot_residue(sigma & ((int64_t(1) << kprev) - 1), A.geom.npass, A.geom.kpass);
        return r < A.n ? (A.n - r + (int64_t(1) << kprev) - 1) >> kprev : 0;
    };
    const T *src_arr[4] = {A.a, A.c, A.d, A.b};  // RAW also streams b
    // rows [g0, g0 + nb) of the item go to the stage by TMA (16-byte granules)
    auto item_rows = [&](int64_t w, int64_t &sigma, int64_t &t0, int64_t &L, int64_t &g0, int64_t &g1,
                         int64_t &gt) {
        sigma = w / tps;
        t0 = (w % tps) * TV;
        L = slot_len(sigma);
        g0 = t0 - R < 0 ? 0 : t0 - R;
        g1 = t0 + TV + R < L ? t0 + TV + R : L;
        gt = g0 + (((g1 - g0) * int64_t(sizeof(T))) & ~int64_t(15)) / int64_t(sizeof(T));  // TMA part end
        if (g1 < g0) g1 = gt = g0;
    };
    auto issue = [&](int64_t w) {  // thread 0 only
        if (w >= nitems) return;
        int64_t sigma, t0, L, g0, g1, gt;
        item_rows(w, sigma, t0, L, g0, g1, gt);
        const uint32_t bytes = uint32_t((gt - g0) * sizeof(T));
        mbar_expect_tx(&bar, NA * bytes);
        if (bytes) {
            const int64_t so = g0 - (t0 - R);  // stage row of g0
            for (int q = 0; q < NA; ++q)
                bulk_g2s(stage + q * ROWS + so, src_arr[q] + sigma * A.in_stride + g0, bytes, &bar);
        }
    };
    if (t == 0) {
        mbar_init(&bar, 1);
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
        issue(blockIdx.x);
    }
    __syncthreads();
    T *el = &eL[0][0][0][0], *er = &eR[0][0][0][0];

    for (int64_t it = 0;; ++it) {
        const int64_t w = int64_t(blockIdx.x) + it * gridDim.x;
        if (w >= nitems) break;
        int64_t sigma, t0, L, g0, g1, gt;
        item_rows(w, sigma, t0, L, g0, g1, gt);
        mbar_wait(&bar, uint32_t(it & 1));
        const int64_t i0 = t0 - R + int64_t(t) * R;  // first row of this thread
        T ra[R], rc[R], rd[R], rb[RAW ? R : 1];
        lds_rows<T, R>(stage + 0 * ROWS + t * R, ra, lane);
        lds_rows<T, R>(stage + 1 * ROWS + t * R, rc, lane);
        lds_rows<T, R>(stage + 2 * ROWS + t * R, rd, lane);
        if constexpr (RAW) lds_rows<T, R>(stage + 3 * ROWS + t * R, rb, lane);
        if (i0 < g0 || i0 + R > gt) {  // rows outside the TMA range: global tail or identity
#pragma unroll
            for (int v = 0; v < R; ++v) {
                const int64_t row = i0 + v;
                if (row < 0 || row >= L) {
                    ra[v] = T(0);
                    rc[v] = T(0);
                    rd[v] = T(0);
                    if constexpr (RAW) rb[v] = T(1);
                } else if (row >= gt) {
                    const int64_t o = sigma * A.in_stride + row;
                    ra[v] = A.a[o];
                    rc[v] = A.c[o];
                    rd[v] = A.d[o];
                    if constexpr (RAW) rb[v] = A.b[o];
                }
            }
        }
        __syncthreads();  // the stage is consumed: prefetch the next tile
        if (t == 0) issue(w + gridDim.x);
        if constexpr (RAW) {
#pragma unroll
            for (int v = 0; v < R; ++v) {
                const T inv = rcp(rb[v]);
                ra[v] = (i0 + v > 0 ? ra[v] : T(0)) * inv;
                rc[v] = (i0 + v < L - 1 ? rc[v] : T(0)) * inv;
                rd[v] = rd[v] * inv;
            }
        }
        if constexpr (KP >= 1) reg_level<T, R, 1, NW, SM>(ra, rc, rd, el, er, 0, lane, warp);
        if constexpr (KP >= 2) reg_level<T, R, 2, NW, SM>(ra, rc, rd, el, er, 1, lane, warp);
        if constexpr (KP >= 3) reg_level<T, R, 4, NW, SM>(ra, rc, rd, el, er, 0, lane, warp);
        if constexpr (KP >= 4) reg_level<T, R, 8, NW, SM>(ra, rc, rd, el, er, 1, lane, warp);
        if (t >= 1 && t <= NT - 2 && i0 < L) {
            const int64_t jb = i0 >> KP;
            const bool full = i0 + R <= L;
#pragma unroll
            for (int rho = 0; rho < NR; ++rho) {
                const int64_t o = out_slot_index(sigma, kprev, KP, rho) * A.out_slot + jb;
                T va[G], vc[G], vd[G];
#pragma unroll
                for (int u = 0; u < G; ++u) {
                    va[u] = ra[rho + NR * u];
                    vc[u] = rc[rho + NR * u];
                    vd[u] = rd[rho + NR * u];
                }
                if (full) {
                    store_run<T, G>(A.oa + o, va);
                    store_run<T, G>(A.oc + o, vc);
                    store_run<T, G>(A.od + o, vd);
                } else {
#pragma unroll
                    for (int u = 0; u < G; ++u) {
                        if (i0 + rho + NR * u < L) {
                            A.oa[o + u] = va[u];
                            A.oc[o + u] = vc[u];
                            A.od[o + u] = vd[u];
                        }
                    }
                }
            }
        }
    }
}

template <typename T, int KP, bool RAW>
static cudaError_t launch_sp(const SplitArgs<T> &A, int64_t tps, int64_t nitems, cudaStream_t st) {
    auto kern = split_pipe_kernel<T, KP, RAW>;
    const size_t smem = size_t(RAW ? 4 : 3) * kRegSplitThreads * kRegSplitRows * sizeof(T);
    cudaError_t e = cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    if (e != cudaSuccess) return e;
    int dev = 0, sms = 148, occ = 1;
    cudaGetDevice(&dev);
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
    cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, kern, kRegSplitThreads, smem);
    const int64_t grid = std::min<int64_t>(nitems, int64_t(std::max(occ, 1)) * sms);
    kern<<<(unsigned)grid, kRegSplitThreads, smem, st>>>(A, tps, nitems);
    return cudaGetLastError();
}

template <typename T>
cudaError_t launch_split_pipe(const SplitArgs<T> &A, bool raw, int64_t m_in, int64_t max_len, cudaStream_t st) {
    constexpr int TV = kRegSplitThreads * kRegSplitRows - 2 * kRegSplitRows;
    const int64_t tps = (max_len + TV - 1) / TV;
    const int64_t nitems = m_in * tps;
    if (nitems <= 0) return cudaSuccess;
    switch (A.kp) {
        case 1: return raw ? launch_sp<T, 1, true>(A, tps, nitems, st) : launch_sp<T, 1, false>(A, tps, nitems, st);
        case 2: return raw ? launch_sp<T, 2, true>(A, tps, nitems, st) : launch_sp<T, 2, false>(A, tps, nitems, st);
        case 3: return raw ? launch_sp<T, 3, true>(A, tps, nitems, st) : launch_sp<T, 3, false>(A, tps, nitems, st);
        case 4: return raw ? launch_sp<T, 4, true>(A, tps, nitems, st) : launch_sp<T, 4, false>(A, tps, nitems, st);
        default: return cudaErrorInvalidConfiguration;
    }
}

template cudaError_t launch_split_pipe<float>(const SplitArgs<float> &, bool, int64_t, int64_t, cudaStream_t);
template cudaError_t launch_split_pipe<double>(const SplitArgs<double> &, bool, int64_t, int64_t, cudaStream_t);

}  // namespace tds
