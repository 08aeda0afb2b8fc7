// split_pipe.cu -- G1, persistent TMA-prefetched register split kernel:
// k_p <= 7 fused PCR levels per HBM pass (§III-B/C, P:L296-303,
// P:L472-493), output de-interleaved into canonical residue slots.
//
// Work items are tiles (slot sigma, tile ti); a resident CTA walks items
// w = blockIdx.x, += gridDim.x.  Thread t of the 256-thread CTA owns 16
// consecutive rows in registers.  Levels with stride <= 8 rows exchange only
// the first / last s rows with the neighbour threads (reg_level); levels with
// stride 16, 32, 64 rows (k_p = 5..7) exchange whole 16-row blocks with the
// threads 1, 2, 4 away (reg_level_far).  The first and last HT threads of a
// CTA are the tile's halo (16*HT >= 2^k_p - 1 rows per side).
//
// Each CTA owns ONE shared-memory stage holding the next tile's input rows (4
// raw arrays on the first pass, 3 normalised ones after): as soon as every
// thread has copied the current tile into registers (conflict-free rotated
// LDS.128) the stage is refilled by cp.async.bulk (TMA) while the CTA runs
// the PCR levels and the de-interleaved stores.
#include "pipe.cuh"
#include "split_reg.cuh"

namespace tds {

template <int KP>
struct SplitShape {
    static constexpr int R = kRegSplitRows;
    static constexpr int NT = kRegSplitThreads;
    static constexpr int NW = NT / 32;
    static constexpr int HT = KP <= 4 ? 1 : (1 << (KP - 4));  // halo threads per side
    static constexpr int TV = (NT - 2 * HT) * R;               // valid rows per tile
    static constexpr int SMN = (1 << (KP - 1)) < 8 ? (1 << (KP - 1)) : 8;
    static constexpr int FAR = NW * kFarMaxTS * 3 * R;        // one half of a far-level edge buffer
};

template <typename T, int KP, bool RAW>
__global__ void __launch_bounds__(kRegSplitThreads, 2) split_pipe_kernel(const SplitArgs<T> A, int64_t tps,
                                                                       int64_t nitems) {
    using S = SplitShape<KP>;
    constexpr int R = S::R, NT = S::NT, NW = S::NW, HT = S::HT, TV = S::TV, SMN = S::SMN;
    constexpr int NR = 1 << KP;
    constexpr int G = KP <= 4 ? (R >> KP) : 1;
    constexpr int NA = RAW ? 4 : 3;  // arrays streamed
    constexpr int ROWS = NT * R;     // rows per stage (tile + halo threads)
    extern __shared__ __align__(128) unsigned char smem_raw[];
    T *stage = reinterpret_cast<T *>(smem_raw);  // [NA][ROWS]
    T *eF = stage + NA * ROWS;                   // far levels: [2][FAR] first-lane blocks
    T *eB = eF + 2 * S::FAR;                     //             [2][FAR] last-lane blocks
    __shared__ T eL[2][3][NW][SMN];
    __shared__ T eR[2][3][NW][SMN];
    __shared__ __align__(8) uint64_t bar;
    const int t = threadIdx.x, lane = t & 31, warp = t >> 5;
    const int kprev = RAW ? 0 : pass_levels(A.geom.npass, A.geom.kpass);

    auto slot_len = [&](int64_t sigma) -> int64_t {
        if (RAW) return A.n;
        const int64_t r = slot_residue(sigma & ((int64_t(1) << kprev) - 1), A.geom.npass, A.geom.kpass);
        return r < A.n ? (A.n - r + (int64_t(1) << kprev) - 1) >> kprev : 0;
    };
    const T *src_arr[4] = {A.a, A.c, A.d, A.b};  // RAW also streams b
    // rows [g0, gt) of the item go to the stage by TMA (16-byte granules); [gt, g1) by LDG
    auto item_rows = [&](int64_t w, int64_t &sigma, int64_t &t0, int64_t &L, int64_t &g0, int64_t &g1,
                         int64_t &gt) {
        sigma = w / tps;
        t0 = (w % tps) * TV;
        L = slot_len(sigma);
        g0 = t0 - HT * R < 0 ? 0 : t0 - HT * R;
        g1 = t0 + TV + HT * R < L ? t0 + TV + HT * R : L;
        if (g1 < g0) g1 = g0;
        gt = g0 + (((g1 - g0) * int64_t(sizeof(T))) & ~int64_t(15)) / int64_t(sizeof(T));
    };
    auto issue = [&](int64_t w) {  // thread 0 only
        if (w >= nitems) return;
        int64_t sigma, t0, L, g0, g1, gt;
        item_rows(w, sigma, t0, L, g0, g1, gt);
        const uint32_t bytes = uint32_t((gt - g0) * sizeof(T));
        mbar_expect_tx(&bar, NA * bytes);
        if (bytes) {
            const int64_t so = g0 - (t0 - HT * R);  // stage row of g0
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
        const int64_t i0 = t0 - HT * R + int64_t(t) * R;  // first row of this thread
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
        if constexpr (KP >= 1) reg_level<T, R, 1, NW, SMN>(ra, rc, rd, el, er, 0, lane, warp);
        if constexpr (KP >= 2) reg_level<T, R, 2, NW, SMN>(ra, rc, rd, el, er, 1, lane, warp);
        if constexpr (KP >= 3) reg_level<T, R, 4, NW, SMN>(ra, rc, rd, el, er, 0, lane, warp);
        if constexpr (KP >= 4) reg_level<T, R, 8, NW, SMN>(ra, rc, rd, el, er, 1, lane, warp);
        if constexpr (KP >= 5) reg_level_far<T, R, 1, NW>(ra, rc, rd, eF, eB, 0, lane, warp);
        if constexpr (KP >= 6) reg_level_far<T, R, 2, NW>(ra, rc, rd, eF, eB, 1, lane, warp);
        if constexpr (KP >= 7) reg_level_far<T, R, 4, NW>(ra, rc, rd, eF, eB, 0, lane, warp);
        if (t >= HT && t < NT - HT && i0 < L) {
            const bool full = i0 + R <= L;
            if constexpr (KP <= 4) {
                // residue v mod 2^KP owns G consecutive positions: one vector store each
                const int64_t jb = i0 >> KP;
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
            } else {
                // 16 rows = 16 residues (16*((i0>>4) mod 2^(KP-4)) + v) at one position j
                const int64_t j = i0 >> KP;
                const int64_t rbase = ((i0 >> 4) & ((int64_t(1) << (KP - 4)) - 1)) << 4;
#pragma unroll
                for (int v = 0; v < R; ++v) {
                    if (full || i0 + v < L) {
                        const int64_t o = out_slot_index(sigma, kprev, KP, rbase + v) * A.out_slot + j;
                        A.oa[o] = ra[v];
                        A.oc[o] = rc[v];
                        A.od[o] = rd[v];
                    }
                }
            }
        }
    }
}

template <int KP>
constexpr int split_pipe_tv() {
    return SplitShape<KP>::TV;
}

template <typename T, int KP, bool RAW>
static cudaError_t launch_sp(const SplitArgs<T> &A, int64_t m_in, int64_t max_len, cudaStream_t st) {
    using S = SplitShape<KP>;
    auto kern = split_pipe_kernel<T, KP, RAW>;
    const size_t smem = size_t(RAW ? 4 : 3) * S::NT * S::R * sizeof(T) +
                        (KP > 4 ? size_t(4) * S::FAR * sizeof(T) : 0);
    cudaError_t e = cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    if (e != cudaSuccess) return e;
    const int64_t tps = (max_len + S::TV - 1) / S::TV;
    const int64_t nitems = m_in * tps;
    if (nitems <= 0) return cudaSuccess;
    int dev = 0, sms = 148, occ = 1;
    cudaGetDevice(&dev);
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
    cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, kern, S::NT, smem);
    const int64_t grid = std::min<int64_t>(nitems, int64_t(std::max(occ, 1)) * sms);
    kern<<<(unsigned)grid, S::NT, smem, st>>>(A, tps, nitems);
    return cudaGetLastError();
}

template <typename T>
cudaError_t launch_split_pipe(const SplitArgs<T> &A, bool raw, int64_t m_in, int64_t max_len, cudaStream_t st) {
#define TDS_SP(KPV) \
    case KPV: return raw ? launch_sp<T, KPV, true>(A, m_in, max_len, st) : launch_sp<T, KPV, false>(A, m_in, max_len, st)
    switch (A.kp) {
        TDS_SP(1);
        TDS_SP(2);
        TDS_SP(3);
        TDS_SP(4);
        TDS_SP(5);
        TDS_SP(6);
        TDS_SP(7);
        default: return cudaErrorInvalidConfiguration;
    }
#undef TDS_SP
}

template cudaError_t launch_split_pipe<float>(const SplitArgs<float> &, bool, int64_t, int64_t, cudaStream_t);
template cudaError_t launch_split_pipe<double>(const SplitArgs<double> &, bool, int64_t, int64_t, cudaStream_t);

}  // namespace tds
