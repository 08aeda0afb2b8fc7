// split_pipe.cu -- G1, persistent TMA-prefetched register split kernel:
// k_p <= 8 fused PCR levels per HBM pass (§III-B/C, P:L296-303,
// P:L472-493), output de-interleaved into canonical residue slots.
//
// Work items are tiles (slot sigma, tile ti); a resident CTA (256 threads)
// walks items w = blockIdx.x, += gridDim.x.  Each CTA owns ONE shared-memory
// stage holding the next tile's input window (4 raw arrays on the first pass,
// 3 normalised ones after): as soon as every thread has copied the current
// window into registers (conflict-free rotated LDS.128) the stage is refilled
// by cp.async.bulk (TMA) while the CTA computes.
//
// Layout A (the first min(k_p, 4) levels, strides 1..8 rows): lane l of warp w
// owns the 16 rows of A-block a = 30w + l.  Warps overlap by two lanes, so a
// level needs no shared memory and no barrier: neighbour rows come by shuffle
// and the two edge lanes of every warp, which see garbage, are the halo
// (after 4 levels rows closer than 15 to a warp end are invalid: lanes 1..30
// stay exact).  The window is 242 A-blocks; blocks 1..240 are valid.
//   k_p <= 4: residue v mod 2^k_p of a lane's rows owns 16 >> k_p consecutive
//     positions: one vector store per residue, coalesced across the warp.
//   k_p = 5..8: a swizzled shared-memory transpose gives layout B -- thread
//     (rho = t >> 4, b = t & 15) owns members m = LEFT - 16 + 16b + u, u = 0..15,
//     of residue class rho mod 16 (member m = A-block m + 1) -- so the strides
//     16..128 rows of the remaining k_p - 4 levels are strides 1..8 of that
//     class (16-lane shuffles; lanes b = 0 and 15 are the halo), and the store
//     is again one vector run per final residue from lanes b = 1..NB.
#include "pipe.cuh"
#include "split_reg.cuh"

namespace tds {

template <int KP>
struct SplitShape {
    static constexpr int R = kRegSplitRows;
    static constexpr int NT = kRegSplitThreads;
    static constexpr int NW = NT / 32;
    static constexpr int AV = 30 * NW;          // valid A-blocks per window
    static constexpr int ROWS = (AV + 2) * R;   // window rows (A-blocks 0 .. AV+1)
    static constexpr int KQ = KP > 4 ? KP - 4 : 0;
    static constexpr int LEFT = KP > 4 ? (1 << KQ) : 0;                   // B halo members before the output
    static constexpr int NB = KP > 4 ? (AV + 1 - (2 << KQ)) / 16 : 0;     // B blocks stored
    static constexpr int TV = KP > 4 ? NB * 16 * R : AV * R;              // output rows per tile
    static constexpr int HEAD = R + LEFT * R;                             // window rows before the tile
    static_assert(TV % (1 << KP) == 0, "tile must hold whole residue periods");
};

template <typename T, int KP, bool RAW>
__global__ void __launch_bounds__(kRegSplitThreads, sizeof(T) == 4 ? 2 : 1)
    split_pipe_kernel(const SplitArgs<T> A, int64_t tps, int64_t nitems) {
    using S = SplitShape<KP>;
    constexpr int R = S::R, AV = S::AV, TV = S::TV, HEAD = S::HEAD, ROWS = S::ROWS;
    constexpr int NA = RAW ? 4 : 3;                            // arrays streamed
    constexpr int NTR = KP > 4 ? (sizeof(T) == 4 ? 3 : 1) : 0;  // arrays per transpose round
    extern __shared__ __align__(128) unsigned char smem_raw[];
    T *stage = reinterpret_cast<T *>(smem_raw);  // [NA][ROWS]
    T *tbuf = stage + NA * ROWS;                 // [NTR][AV * 16] transpose buffer
    __shared__ __align__(8) uint64_t bar;
    const int t = threadIdx.x, lane = t & 31, warp = t >> 5;
    const int ablk = 30 * warp + lane;  // A-block of this thread
    const int kprev = RAW ? 0 : pass_levels(A.geom.npass, A.geom.kpass);
    const bool small_items = nitems < (int64_t(1) << 31);

    auto slot_len = [&](int64_t sigma) -> int64_t {
        if (RAW) return A.n;
        const int64_t r = sigma & ((int64_t(1) << kprev) - 1);
        return r < A.n ? (A.n - r + (int64_t(1) << kprev) - 1) >> kprev : 0;
    };
    const T *src_arr[4] = {A.a, A.c, A.d, A.b};  // RAW also streams b
    // rows [g0, gt) of the item go to the stage by TMA (16-byte granules); [gt, g1) by LDG
    auto item_rows = [&](int64_t w, int64_t &sigma, int64_t &t0, int64_t &L, int64_t &g0, int64_t &g1,
                         int64_t &gt) {
        if (small_items) {
            const uint32_t q = uint32_t(w) / uint32_t(tps);
            sigma = q;
            t0 = int64_t(uint32_t(w) - q * uint32_t(tps)) * TV;
        } else {
            sigma = w / tps;
            t0 = (w % tps) * TV;
        }
        L = slot_len(sigma);
        g0 = t0 - HEAD < 0 ? 0 : t0 - HEAD;
        g1 = t0 - HEAD + ROWS < L ? t0 - HEAD + ROWS : L;
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
            const int64_t so = g0 - (t0 - HEAD);  // stage row of g0
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

    for (int64_t it = 0;; ++it) {
        const int64_t w = int64_t(blockIdx.x) + it * gridDim.x;
        if (w >= nitems) break;
        int64_t sigma, t0, L, g0, g1, gt;
        item_rows(w, sigma, t0, L, g0, g1, gt);
        mbar_wait(&bar, uint32_t(it & 1));
        const int64_t i0 = t0 - HEAD + int64_t(ablk) * R;  // first row of this thread (layout A)
        T ra[R], rc[R], rd[R], rb[RAW ? R : 1];
        lds_rows<T, R>(stage + 0 * ROWS + ablk * R, ra, lane);
        lds_rows<T, R>(stage + 1 * ROWS + ablk * R, rc, lane);
        lds_rows<T, R>(stage + 2 * ROWS + ablk * R, rd, lane);
        if constexpr (RAW) lds_rows<T, R>(stage + 3 * ROWS + ablk * R, rb, lane);
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
            if (i0 <= 0 || i0 + R >= L) {  // a_0 and c_{n-1} are outside the system
#pragma unroll
                for (int v = 0; v < R; ++v) {
                    if (i0 + v == 0) ra[v] = T(0);
                    if (i0 + v == L - 1) rc[v] = T(0);
                }
            }
            if constexpr (sizeof(T) == 4) {
#pragma unroll
                for (int v = 0; v < R; v += 2) {
                    const float2 inv = make_float2(rcp(rb[v]), rcp(rb[v + 1]));
                    const float2 a = __fmul2_rn(make_float2(ra[v], ra[v + 1]), inv);
                    const float2 c = __fmul2_rn(make_float2(rc[v], rc[v + 1]), inv);
                    const float2 d = __fmul2_rn(make_float2(rd[v], rd[v + 1]), inv);
                    ra[v] = a.x;
                    ra[v + 1] = a.y;
                    rc[v] = c.x;
                    rc[v + 1] = c.y;
                    rd[v] = d.x;
                    rd[v + 1] = d.y;
                }
            } else {
#pragma unroll
                for (int v = 0; v < R; ++v) {
                    const T inv = rcp(rb[v]);
                    ra[v] *= inv;
                    rc[v] *= inv;
                    rd[v] *= inv;
                }
            }
        }
        if constexpr (KP >= 1) reg_level_w<T, R, 1, 32>(ra, rc, rd);
        if constexpr (KP >= 2) reg_level_w<T, R, 2, 32>(ra, rc, rd);
        if constexpr (KP >= 3) reg_level_w<T, R, 4, 32>(ra, rc, rd);
        if constexpr (KP >= 4) reg_level_w<T, R, 8, 32>(ra, rc, rd);
        if constexpr (KP <= 4) {
            constexpr int NR = 1 << KP, G = R >> KP;
            if (lane >= 1 && lane <= 30 && i0 < L) {
                const bool full = i0 + R <= L;
                // residue v mod 2^KP owns G consecutive positions: one vector store each
                const int64_t step = (int64_t(1) << kprev) * A.out_slot;
                const int64_t o0 = out_slot_index(sigma, kprev, KP, 0) * A.out_slot + (i0 >> KP);
#pragma unroll
                for (int rho = 0; rho < NR; ++rho) {
                    const int64_t o = o0 + rho * step;
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
        } else {
            // ---- layout B: 16 consecutive members of residue class rho mod 16
            constexpr int KQ = S::KQ, LEFT = S::LEFT, NB = S::NB;
            constexpr int NQ = 1 << KQ, G = R >> KQ;
            const int rho = t >> 4, b = t & 15;
            const int mb = LEFT - 16 + 16 * b;  // member of u = 0
            const bool wr = lane >= 1 && lane <= 30;
            if constexpr (NTR == 3) {  // one round: 3 buffers
                if (wr) {
                    tr_write<T, R>(ra, tbuf, ablk - 1);
                    tr_write<T, R>(rc, tbuf + AV * 16, ablk - 1);
                    tr_write<T, R>(rd, tbuf + 2 * AV * 16, ablk - 1);
                }
                __syncthreads();
                tr_read<T, R, AV>(ra, tbuf, mb, rho);
                tr_read<T, R, AV>(rc, tbuf + AV * 16, mb, rho);
                tr_read<T, R, AV>(rd, tbuf + 2 * AV * 16, mb, rho);
            } else {  // three rounds through one buffer
                if (wr) tr_write<T, R>(ra, tbuf, ablk - 1);
                __syncthreads();
                tr_read<T, R, AV>(ra, tbuf, mb, rho);
                __syncthreads();
                if (wr) tr_write<T, R>(rc, tbuf, ablk - 1);
                __syncthreads();
                tr_read<T, R, AV>(rc, tbuf, mb, rho);
                __syncthreads();
                if (wr) tr_write<T, R>(rd, tbuf, ablk - 1);
                __syncthreads();
                tr_read<T, R, AV>(rd, tbuf, mb, rho);
            }
            if constexpr (KQ >= 1) reg_level_w<T, R, 1, 16>(ra, rc, rd);
            if constexpr (KQ >= 2) reg_level_w<T, R, 2, 16>(ra, rc, rd);
            if constexpr (KQ >= 3) reg_level_w<T, R, 4, 16>(ra, rc, rd);
            if constexpr (KQ >= 4) reg_level_w<T, R, 8, 16>(ra, rc, rd);
            // member LEFT + 16(b-1) + u is row t0 + 16(16(b-1) + u) + rho
            const int64_t r0 = t0 + 256 * (b - 1) + rho;  // row of u = 0
            if (b >= 1 && b <= NB && r0 < L) {
                const bool full = r0 + 16 * (R - 1) < L;
                const int64_t step = (int64_t(16) << kprev) * A.out_slot;  // residue rho + 16 mu
                const int64_t o0 = out_slot_index(sigma, kprev, KP, rho) * A.out_slot + (r0 >> KP);
#pragma unroll
                for (int mu = 0; mu < NQ; ++mu) {
                    const int64_t o = o0 + mu * step;
                    T va[G], vc[G], vd[G];
#pragma unroll
                    for (int q = 0; q < G; ++q) {
                        va[q] = ra[mu + NQ * q];
                        vc[q] = rc[mu + NQ * q];
                        vd[q] = rd[mu + NQ * q];
                    }
                    if (full) {
                        store_run<T, G>(A.oa + o, va);
                        store_run<T, G>(A.oc + o, vc);
                        store_run<T, G>(A.od + o, vd);
                    } else {
#pragma unroll
                        for (int q = 0; q < G; ++q) {
                            if (r0 + 16 * (mu + NQ * q) < L) {
                                A.oa[o + q] = va[q];
                                A.oc[o + q] = vc[q];
                                A.od[o + q] = vd[q];
                            }
                        }
                    }
                }
            }
        }
    }
}

template <typename T, int KP, bool RAW>
static cudaError_t launch_sp(const SplitArgs<T> &A, int64_t m_in, int64_t max_len, cudaStream_t st) {
    using S = SplitShape<KP>;
    auto kern = split_pipe_kernel<T, KP, RAW>;
    constexpr int NTR = KP > 4 ? (sizeof(T) == 4 ? 3 : 1) : 0;
    const size_t smem = (size_t((RAW ? 4 : 3)) * S::ROWS + size_t(NTR) * S::AV * 16) * sizeof(T);
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
        TDS_SP(8);
        default: return cudaErrorInvalidConfiguration;
    }
#undef TDS_SP
}

template cudaError_t launch_split_pipe<float>(const SplitArgs<float> &, bool, int64_t, int64_t, cudaStream_t);
template cudaError_t launch_split_pipe<double>(const SplitArgs<double> &, bool, int64_t, int64_t, cudaStream_t);

}  // namespace tds
