// onchip_cpipe.cu -- G2 for k = 0 (no split pass): persistent, TMA-fed,
// optionally spread over a thread-block cluster of 2-8 CTAs (§III-A base
// kernel, §III-D Stage 1 "several processors on one system" mapped to a
// cluster with distributed shared memory).
//
// Every system of n rows is solved on chip straight from the caller's a, b,
// c, d: 20 bytes per equation instead of the 52 of a split pass + on-chip +
// placement.  A cluster of C CTAs (C = 1 or 2) x NT threads x R rows per
// thread holds one system (n <= C * NT * R: 16384 fp32 / 8192 fp64 rows for
// C = 2, up to 65536 / 32768 for C = 8); clusters walk systems sys = cluster
// id, += clusters.  Per CTA one
// shared-memory stage holds the next system's 4 raw arrays (one swizzled TMA
// box each); it is refilled as soon as the rows are in registers.
//
// The solve is the warp form of onchip_pipe.cu (CR in registers, CR across
// the 32 lanes of each warp by shuffles, one row per warp left, PCR over
// those rows by one warp, back substitution) with the CTA boundary handled
// like the warp boundary: the last warp's lane-31 chain reads the next CTA's
// published rows through DSMEM, and the per-warp top rows are ALL-GATHERED:
// every CTA receives all C * nwarps of them and solves that small system
// itself (one warp's shuffles up to 32 rows, else shared-memory PCR), so each
// CTA takes its own x of the top rows without a scatter hop (measured against
// gather-to-CTA-0 + scatter: config 2 0.098 -> 0.089 ms, config 4 0.227 ->
// 0.217 ms).  Both cross-CTA hand-offs are point-to-point: st.async stores
// into the peer's shared memory counted on the peer's mbarrier (no cluster
// barrier inside the loop).  x is written in original order (k = 0: no placement).
#include <cooperative_groups.h>

#include "pipe.cuh"

namespace cg = cooperative_groups;

namespace tds {

// The cluster top solve's 32 lane rows by PCR (5 levels, no lane back
// substitution) instead of CR (5 + 5 levels): config 2 0.0810 -> 0.0784 ms
// (gpurun_out/r02b18, profiles/r02b18/).  -DTDS_CPIPE_LANE_PCR=0 restores CR.
#ifndef TDS_CPIPE_LANE_PCR
#define TDS_CPIPE_LANE_PCR 1
#endif

template <int C>
__device__ __forceinline__ void csync() {
    if constexpr (C > 1) cg::this_cluster().sync(); else __syncthreads();
}

// One warp solves a system of 32 * RZ normalised rows (lane l holds rows
// l RZ .. l RZ + RZ - 1): cyclic reduction over log2(RZ) levels in registers,
// then the 32 lane rows by PCR across the lanes (shuffles; every row
// decouples), then back substitution of the register levels; rows outside
// the system are identity rows.  No barrier (the cluster's top rows,
// C = 4 / 8, replace 6 / 7 shared-memory PCR levels with 14 barriers).
template <typename T, int RZ>
__device__ __forceinline__ void warp_cr_solve(T (&ra)[RZ], T (&rc)[RZ], T (&rd)[RZ], int lane) {
    constexpr unsigned FULL = 0xffffffffu;
    constexpr int CR = ilog2c(RZ);
#pragma unroll
    for (int l = 1; l <= CR; ++l) {
        const int s = 1 << (l - 1);
        const T na = __shfl_down_sync(FULL, ra[s - 1], 1), nc = __shfl_down_sync(FULL, rc[s - 1], 1),
                nd = __shfl_down_sync(FULL, rd[s - 1], 1);
        const bool hn = lane < 31;
#pragma unroll
        for (int v = (1 << l) - 1; v < RZ; v += (1 << l)) {
            const bool last = v + s >= RZ;
            row_update_early(ra[v], rc[v], rd[v], ra[v - s], rc[v - s], rd[v - s], last ? (hn ? na : T(0)) : ra[v + s],
                       last ? (hn ? nc : T(0)) : rc[v + s], last ? (hn ? nd : T(0)) : rd[v + s]);
        }
    }
    T za = ra[RZ - 1], zc = rc[RZ - 1], zd = rd[RZ - 1];
#if TDS_CPIPE_LANE_PCR
    // the 32 lane rows by PCR: every lane updates at every level, so after 5
    // levels each row is decoupled (x = d) and no lane back substitution follows
#pragma unroll
    for (int l = 1; l <= 5; ++l) {
        const int s = 1 << (l - 1);
        const T la = __shfl_up_sync(FULL, za, s), lc = __shfl_up_sync(FULL, zc, s), ld = __shfl_up_sync(FULL, zd, s);
        const T xa = __shfl_down_sync(FULL, za, s), xc = __shfl_down_sync(FULL, zc, s),
                xd = __shfl_down_sync(FULL, zd, s);
        const bool hl = lane >= s, hr = lane + s < 32 && !TDS_MUT(3, s >= 4);
        row_update_early(za, zc, zd, hl ? la : T(0), hl ? lc : T(0), hl ? ld : T(0), hr ? xa : T(0),
                         hr ? xc : T(0), hr ? xd : T(0));
    }
    const T xw = zd;
#else
#pragma unroll
    for (int l = 1; l <= 5; ++l) {
        const int s = 1 << (l - 1);
        const T la = __shfl_up_sync(FULL, za, s), lc = __shfl_up_sync(FULL, zc, s), ld = __shfl_up_sync(FULL, zd, s);
        const T xa = __shfl_down_sync(FULL, za, s), xc = __shfl_down_sync(FULL, zc, s),
                xd = __shfl_down_sync(FULL, zd, s);
        const bool hr = lane + s < 32 && !TDS_MUT(3, s >= 4);
        T a = za, c = zc, d = zd;
        row_update_early(a, c, d, la, lc, ld, hr ? xa : T(0), hr ? xc : T(0), hr ? xd : T(0));
        const bool upd = (lane & ((1 << l) - 1)) == (1 << l) - 1;
        za = upd ? a : za;
        zc = upd ? c : zc;
        zd = upd ? d : zd;
    }
    T xw = lane == 31 ? zd : T(0);  // the last row decouples: x = d
#pragma unroll
    for (int l = 5; l >= 1; --l) {
        const int s = 1 << (l - 1);
        const T xl = __shfl_up_sync(FULL, xw, s);
        const T xr = __shfl_down_sync(FULL, xw, s);
        const T xn = zd - za * (lane >= s ? xl : T(0)) - zc * (lane + s < 32 ? xr : T(0));
        xw = (lane & ((1 << l) - 1)) == s - 1 ? xn : xw;
    }
#endif
    T xleft = __shfl_up_sync(FULL, xw, 1);
    if (lane == 0) xleft = T(0);
    rd[RZ - 1] = xw;
#pragma unroll
    for (int l = CR; l >= 1; --l) {
        const int s = 1 << (l - 1);
#pragma unroll
        for (int v = s - 1; v < RZ - 1; v += 2 * s) {
            const T xlv = (v >= s) ? rd[v - s] : xleft;
            rd[v] = rd[v] - ra[v] * xlv - rc[v] * rd[v + s];
        }
    }
}

template <typename T>
__device__ __forceinline__ T *peer(T *p, int rank) {  // DSMEM address of p in cluster CTA `rank`
    return cg::this_cluster().map_shared_rank(p, rank);
}

template <typename T, int R, int C>
__global__ void __launch_bounds__(512, 1)
    onchip_cpipe_kernel(const OnchipArgs<T> A, const __grid_constant__ TmapSet tm, int32_t tma_lines,
                        const __grid_constant__ TmapSet tmx) {
    static_assert(R * sizeof(T) == 64, "64 bytes of rows per thread");
    constexpr int CR = ilog2c(R), ELINE = 128 / int(sizeof(T));
    constexpr int ZMAX = 16 * C > 32 ? 16 * C : 32;  // top rows of a cluster (<= 16 warps per CTA)
    constexpr unsigned FULL = 0xffffffffu;
    extern __shared__ __align__(1024) unsigned char smem_raw[];
    __shared__ __align__(8) uint64_t full_bar;
    const int NT = blockDim.x, ROWS = NT * R;
    const int t = threadIdx.x, lane = t & 31, warp = t >> 5, nwarps = NT >> 5;
    const int rank = C > 1 ? int(cg::this_cluster().block_rank()) : 0;
    const int64_t cid = int64_t(blockIdx.x) / C, ncl = int64_t(gridDim.x) / C;
    T *stage = reinterpret_cast<T *>(smem_raw + ((1024u - (smem_u32(smem_raw) & 1023u)) & 1023u));  // [4][ROWS]
    T *xst = stage + 4 * ROWS;         // [ROWS]           x of the previous system, for its TMA store
    T *e_in = xst + ROWS;              // [nwarps][CR][3]  lane 0's row s-1 before register level l
    T *w_in = e_in + nwarps * CR * 3;  // [nwarps][5][3]   lane s-1 before lane level l
    T *lft = w_in + nwarps * 15;       // [nwarps][5][3]   lane 31-s before lane level l
    // per-warp top rows of the whole cluster, [2][3][ZMAX] (double-buffered by
    // system parity: a peer may already send the next system's rows)
    T *top_base = lft + nwarps * 15;
    T *xtop = top_base + 6 * ZMAX;  // [33] x of this CTA's top rows; [32] = previous CTA's last
    T *rnext = xtop + 33;              // [CR+5][3]        the next CTA's warp-0 rows (e_in, w_in) for our last warp
    // mbarriers of the cluster hand-offs (one phase per system): rnext filled,
    // top rows gathered (CTA 0), x of the top rows delivered
    __shared__ __align__(8) uint64_t mb_next, mb_top;
    const int64_t n = A.n;
    const int64_t tma_rows = int64_t(tma_lines) * ELINE;  // rows of every system in whole TMA lines
    const int64_t row0 = int64_t(rank) * ROWS;              // this CTA's first row of the system

    auto issue = [&](int64_t sys) {  // thread 0
        if (sys >= A.m_systems) return;
        if (tma_lines == 0 || row0 >= tma_rows) {
            mbar_expect_tx(&full_bar, 0);
            return;
        }
        mbar_expect_tx(&full_bar, 4 * uint32_t(ROWS) * sizeof(T));
#pragma unroll
        for (int q = 0; q < 4; ++q)
            tma_load_lines(stage + q * ROWS, &tm.m[q], int(row0 / ELINE), int(sys), &full_bar);
    };
    pdl_wait();  // the previous kernel on the stream is complete before any global access
    if (t == 0) {
        mbar_init(&full_bar, 1);
        mbar_init(&mb_next, 1);
        mbar_init(&mb_top, 1);
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
        issue(cid);
    }
    csync<C>();  // every CTA of the cluster runs (and has its mbarriers) before any DSMEM access
    // peer addresses of the hand-off buffers
    uint32_t prev_rnext = 0, prev_mb_next = 0;
    if constexpr (C > 1) {
        if (rank > 0) {
            prev_rnext = cluster_addr(rnext, rank - 1);
            prev_mb_next = cluster_addr(&mb_next, rank - 1);
        }
    }

    for (int64_t it = 0;; ++it) {
        const int64_t sys = cid + it * ncl;
        if (sys >= A.m_systems) break;
        pdl_trigger_if_last(sys + ncl >= A.m_systems);
        T *top = top_base + int(it & 1) * 3 * ZMAX;
        mbar_wait(&full_bar, uint32_t(it & 1));
        const int64_t i0 = row0 + int64_t(t) * R;  // first row of this thread
        if (row0 + ROWS > tma_rows) {
            // CTA-uniform: rows past the TMA lines are patched into the stage --
            // the tail by LDG, identity rows (0, 1, 0, 0) past n
            for (int j = t; j < ROWS; j += NT) {
                const int64_t i = row0 + j;
                if (i < tma_rows) continue;
                const int o = sw_off<T>(j);
                T va = T(0), vb = T(1), vc = T(0), vd = T(0);
                if (i < n) {
                    const int64_t g = sys * A.batch_stride + i;
                    va = A.a[g];
                    vb = A.b[g];
                    vc = A.c[g];
                    vd = A.d[g];
                }
                stage[o] = va;
                stage[ROWS + o] = vb;
                stage[2 * ROWS + o] = vc;
                stage[3 * ROWS + o] = vd;
            }
            fence_proxy_async_smem();  // before the TMA refill of the stage
            __syncthreads();
        }
        // normalise while loading (b = 1): only 1/b and the three arrays stay live
        T ra[R], rc[R], rd[R];
        {
            T inv[R];
            lds_rows_sw<T, R>(stage + ROWS, t * R, inv);
#pragma unroll
            for (int v = 0; v < R; ++v) inv[v] = rcp(inv[v]);
            lds_rows_sw<T, R>(stage, t * R, ra);
            lds_rows_sw<T, R>(stage + 2 * ROWS, t * R, rc);
            lds_rows_sw<T, R>(stage + 3 * ROWS, t * R, rd);
#pragma unroll
            for (int v = 0; v < R; ++v) {
                ra[v] *= inv[v];
                rc[v] *= inv[v];
                rd[v] *= inv[v];
            }
        }
        __syncthreads();  // the stage is in registers (and the previous x is in xst)
        if (t == 0) {
            if constexpr (C > 1) {  // announce this system's incoming hand-off bytes
                if (rank + 1 < C) mbar_expect_tx(&mb_next, uint32_t((CR + 5) * 3 * sizeof(T)));
                mbar_expect_tx(&mb_top, uint32_t(C * nwarps * 3 * sizeof(T)));  // every CTA gets every top row
            }
            issue(sys + ncl);
            if (it > 0 && tma_lines > 0 && row0 < tma_rows) {  // the previous system's x: one TMA store
                tma_store_lines(&tmx.m[0], xst, int(row0 / ELINE), int(sys - ncl));
                bulk_commit();
            }
        }
        if (i0 <= 0 || i0 + R >= n) {  // a_0 and c_{n-1} are outside the system
#pragma unroll
            for (int v = 0; v < R; ++v) {
                if (i0 + v == 0) ra[v] = T(0);
                if (i0 + v == n - 1) rc[v] = T(0);
            }
        }
        // ---- register CR levels; lane 31 defers its row R-1 chain
#pragma unroll
        for (int l = 1; l <= CR; ++l) {
            const int s = 1 << (l - 1);
            const T pa = ra[s - 1], pc = rc[s - 1], pd = rd[s - 1];
            const T na = __shfl_down_sync(FULL, pa, 1), nc = __shfl_down_sync(FULL, pc, 1),
                    nd = __shfl_down_sync(FULL, pd, 1);
            if (lane == 0) {
                T *e = e_in + (warp * CR + l - 1) * 3;
                e[0] = pa;
                e[1] = pc;
                e[2] = pd;
                if constexpr (C > 1) {
                    if (warp == 0 && rank > 0) {  // the previous CTA's last warp needs them
                        const uint32_t o = prev_rnext + uint32_t((l - 1) * 3 * sizeof(T));
                        st_async(o, pa, prev_mb_next);
                        st_async(o + sizeof(T), pc, prev_mb_next);
                        st_async(o + 2 * sizeof(T), pd, prev_mb_next);
                    }
                }
            }
#pragma unroll
            for (int v = (1 << l) - 1; v < R; v += (1 << l)) {
                const bool last = v == R - 1;
                T a = ra[v], c = rc[v], d = rd[v];
                row_update_early(a, c, d, ra[v - s], rc[v - s], rd[v - s], last ? na : ra[(v + s) % R],
                           last ? nc : rc[(v + s) % R], last ? nd : rd[(v + s) % R]);
                const bool keep = last && lane == 31;
                ra[v] = keep ? ra[v] : a;
                rc[v] = keep ? rc[v] : c;
                rd[v] = keep ? rd[v] : d;
            }
        }
        // ---- CR across lanes; lane 31 (kept at every level) defers
        T za = ra[R - 1], zc = rc[R - 1], zd = rd[R - 1];
#pragma unroll
        for (int l = 1; l <= 5; ++l) {
            const int s = 1 << (l - 1);
            const T la = __shfl_up_sync(FULL, za, s), lc = __shfl_up_sync(FULL, zc, s),
                    ld = __shfl_up_sync(FULL, zd, s);
            const T xa = __shfl_down_sync(FULL, za, s), xc = __shfl_down_sync(FULL, zc, s),
                    xd = __shfl_down_sync(FULL, zd, s);
            if (lane == s - 1) {
                T *w = w_in + (warp * 5 + l - 1) * 3;
                w[0] = za;
                w[1] = zc;
                w[2] = zd;
                if constexpr (C > 1) {
                    if (warp == 0 && rank > 0) {
                        const uint32_t o = prev_rnext + uint32_t((CR + l - 1) * 3 * sizeof(T));
                        st_async(o, za, prev_mb_next);
                        st_async(o + sizeof(T), zc, prev_mb_next);
                        st_async(o + 2 * sizeof(T), zd, prev_mb_next);
                    }
                }
            }
            if (lane == 31 - s) {
                T *f = lft + (warp * 5 + l - 1) * 3;
                f[0] = za;
                f[1] = zc;
                f[2] = zd;
            }
            T a = za, c = zc, d = zd;
            row_update_early(a, c, d, la, lc, ld, xa, xc, xd);
            const bool upd = (lane & ((1 << l) - 1)) == (1 << l) - 1 && lane != 31;
            za = upd ? a : za;
            zc = upd ? c : zc;
            zd = upd ? d : zd;
        }
        if (t == 0) bulk_wait_read0();  // xst is rewritten at the end of this system
        __syncthreads();  // (1) every warp's first rows are published (this CTA)
        if (lane == 31) {  // the deferred chains; the last warp uses the next CTA's pushed rows
            const bool last_warp = warp == nwarps - 1;
            const bool h = !last_warp || (rank + 1 < C && !TDS_MUT(2, true));
            const T *en = e_in + (warp + 1) * CR * 3, *wn = w_in + (warp + 1) * 15;
            if constexpr (C > 1) {
                if (last_warp && rank + 1 < C) {
                    mbar_wait(&mb_next, uint32_t(it & 1));
                    en = rnext;
                    wn = rnext + CR * 3;
                }
            }
#pragma unroll
            for (int l = 1; l <= CR; ++l) {
                const int s = 1 << (l - 1);
                const T *e = en + (l - 1) * 3;
                row_update_early(ra[R - 1], rc[R - 1], rd[R - 1], ra[R - 1 - s], rc[R - 1 - s], rd[R - 1 - s],
                           h ? e[0] : T(0), h ? e[1] : T(0), h ? e[2] : T(0));
            }
            za = ra[R - 1];
            zc = rc[R - 1];
            zd = rd[R - 1];
#pragma unroll
            for (int l = 1; l <= 5; ++l) {
                const T *f = lft + (warp * 5 + l - 1) * 3;
                const T *w = wn + (l - 1) * 3;
                row_update_early(za, zc, zd, f[0], f[1], f[2], h ? w[0] : T(0), h ? w[1] : T(0), h ? w[2] : T(0));
            }
            const int z = rank * nwarps + warp;
            if constexpr (C > 1) {  // all-gather: to every CTA (itself included), counted on its mb_top
#pragma unroll
                for (int q = 0; q < C; ++q) {
                    const uint32_t tq = cluster_addr(top, q), bq = cluster_addr(&mb_top, q);
                    st_async(tq + uint32_t(z * sizeof(T)), za, bq);
                    st_async(tq + uint32_t((ZMAX + z) * sizeof(T)), zc, bq);
                    st_async(tq + uint32_t((2 * ZMAX + z) * sizeof(T)), zd, bq);
                }
            } else {
                top[z] = za;
                top[ZMAX + z] = zc;
                top[2 * ZMAX + z] = zd;
            }
        }
        if constexpr (C == 1) __syncthreads();  // (2) every top row is in top[]
        if constexpr (C > 1) {
            if (C * nwarps > 32 || warp == 0) mbar_wait(&mb_top, uint32_t(it & 1));
        }
        if (C * nwarps > 32 && C * nwarps == ZMAX) {
            // the Z = 64 / 128 top rows (C = 4 / 8, 16 warps): cyclic reduction in one warp (2 / 4 rows per lane)
            constexpr int RZ = ZMAX / 32;
            if (warp == 0) {
                T za2[RZ], zc2[RZ], zd2[RZ];
#pragma unroll
                for (int v = 0; v < RZ; ++v) {
                    za2[v] = top[lane * RZ + v];
                    zc2[v] = top[ZMAX + lane * RZ + v];
                    zd2[v] = top[2 * ZMAX + lane * RZ + v];
                }
                warp_cr_solve<T, RZ>(za2, zc2, zd2, lane);
#pragma unroll
                for (int v = 0; v < RZ; ++v) {  // this CTA's x of the top rows, and the previous CTA's last one
                    const int z = lane * RZ + v, r = z / nwarps, w = z % nwarps;
                    if (r == rank) xtop[w] = zd2[v];
                    if (z == rank * nwarps - 1) xtop[32] = zd2[v];
                }
            }
        } else if (C * nwarps > 32) {
            // PCR over the Z = C * nwarps top rows in shared memory (every row decouples, x = d)
            const int Z = C * nwarps;
            T *za2 = top, *zc2 = top + ZMAX, *zd2 = top + 2 * ZMAX;
            for (int s = 1; s < Z; s <<= 1) {
                T a = T(0), c = T(0), d = T(0);
                if (t < Z) {
                    a = za2[t];
                    c = zc2[t];
                    d = zd2[t];
                    const bool hl = t >= s, hr = t + s < Z && !TDS_MUT(3, s >= 4);
                    row_update_early(a, c, d, hl ? za2[t - s] : T(0), hl ? zc2[t - s] : T(0), hl ? zd2[t - s] : T(0),
                               hr ? za2[t + s] : T(0), hr ? zc2[t + s] : T(0), hr ? zd2[t + s] : T(0));
                }
                __syncthreads();
                if (t < Z) {
                    za2[t] = a;
                    zc2[t] = c;
                    zd2[t] = d;
                }
                __syncthreads();
            }
            // every CTA solved the same system: it takes its own x (and the previous CTA's last)
            if (t < nwarps) xtop[t] = zd2[rank * nwarps + t];
            if (t == 32) xtop[32] = rank > 0 ? zd2[rank * nwarps - 1] : T(0);
        } else if (warp == 0) {  // <= 32 rows: PCR with shuffles, x = d
            const int Z = C * nwarps;
            T a = lane < Z ? top[lane] : T(0), c = lane < Z ? top[ZMAX + lane] : T(0),
              d = lane < Z ? top[2 * ZMAX + lane] : T(0);
            for (int s = 1; s < Z; s <<= 1) {
                const T la = __shfl_up_sync(FULL, a, s), lc = __shfl_up_sync(FULL, c, s),
                        ld = __shfl_up_sync(FULL, d, s);
                const T xa = __shfl_down_sync(FULL, a, s), xc = __shfl_down_sync(FULL, c, s),
                        xd = __shfl_down_sync(FULL, d, s);
                const bool hl = lane >= s, hr = lane + s < Z && !TDS_MUT(3, s >= 4);
                T na = a, nc = c, nd = d;
                row_update_early(na, nc, nd, hl ? la : T(0), hl ? lc : T(0), hl ? ld : T(0), hr ? xa : T(0),
                           hr ? xc : T(0), hr ? xd : T(0));
                a = lane < Z ? na : a;
                c = lane < Z ? nc : c;
                d = lane < Z ? nd : d;
            }
            if (lane < Z) {  // this CTA's x of the top rows, and the previous CTA's last one
                const int r = lane / nwarps, w = lane % nwarps;
                if (r == rank) xtop[w] = d;
                if (lane == rank * nwarps - 1) xtop[32] = d;
            }
        }
        __syncthreads();  // (3) x of this CTA's top rows is in xtop
        // ---- back substitution across lanes, then in registers
        T xw = lane == 31 ? xtop[warp] : T(0);
        const T xprev = warp > 0 ? xtop[warp - 1] : (rank > 0 ? xtop[32] : T(0));
#pragma unroll
        for (int l = 5; l >= 1; --l) {
            const int s = 1 << (l - 1);
            const T xl = __shfl_up_sync(FULL, xw, s);
            const T xr = __shfl_down_sync(FULL, xw, s);
            const T xn = zd - za * (lane >= s ? xl : xprev) - zc * xr;
            xw = (lane & ((1 << l) - 1)) == s - 1 ? xn : xw;
        }
        T xleft = __shfl_up_sync(FULL, xw, 1);
        if (lane == 0) xleft = xprev;
        rd[R - 1] = xw;
#pragma unroll
        for (int l = CR; l >= 1; --l) {
            const int s = 1 << (l - 1);
#pragma unroll
            for (int v = s - 1; v < R - 1; v += 2 * s) {
                const T xlv = (v >= s) ? rd[(v - s + R) % R] : xleft;
                rd[v] = rd[v] - ra[v] * xlv - rc[v] * rd[(v + s) % R];
            }
        }
        // ---- x in original order (k = 0): staged (swizzled) for the next
        // iteration's TMA store -- no global stores pending at the cluster
        // barriers -- except rows past the TMA lines
        T *dst = A.x + sys * A.batch_stride + i0;
        if (tma_lines > 0 && row0 < tma_rows) {
            sts_rows_sw<T, R>(xst, t * R, rd);
            fence_proxy_async_smem();
            if (i0 + R > tma_rows) {
#pragma unroll
                for (int v = 0; v < R; ++v)
                    if (i0 + v >= tma_rows && i0 + v < n) dst[v] = rd[v];
            }
        } else if (i0 + R <= n) {
            constexpr int W = 16 / int(sizeof(T));
#pragma unroll
            for (int q = 0; q < R / W; ++q) {
                if constexpr (sizeof(T) == 4)
                    __stcs(reinterpret_cast<float4 *>(dst) + q,
                           make_float4(rd[4 * q], rd[4 * q + 1], rd[4 * q + 2], rd[4 * q + 3]));
                else
                    __stcs(reinterpret_cast<double2 *>(dst) + q, make_double2(rd[2 * q], rd[2 * q + 1]));
            }
        } else if (i0 < n) {
#pragma unroll
            for (int v = 0; v < R; ++v)
                if (i0 + v < n) dst[v] = rd[v];
        }
        // the next system's first scratch writes follow its stage barrier and the
        // cluster barrier (1) orders every cross-CTA read of this system's scratch
    }
    __syncthreads();
    if (t == 0) {  // the last system's x
        const int64_t nit = (A.m_systems - cid + ncl - 1) / ncl;
        if (nit > 0 && tma_lines > 0 && row0 < tma_rows) {
            tma_store_lines(&tmx.m[0], xst, int(row0 / ELINE), int(cid + (nit - 1) * ncl));
            bulk_commit();
        }
        bulk_wait_all();
    }
    csync<C>();  // no CTA leaves while a peer may still read its shared memory
}

size_t onchip_cpipe_smem_bytes(int32_t dtype, int32_t threads, int32_t cluster) {
    const int64_t R = 64 / dsize(dtype);
    const int64_t nw = threads / 32;
    const int64_t zmax = std::max<int64_t>(32, 16 * cluster);
    return 1024 + size_t((5 * int64_t(threads) * R + nw * (4 + 5 + 5) * 3 + 6 * zmax + 33 + 27) * dsize(dtype));
}

template <typename T>
cudaError_t launch_onchip_cpipe(const OnchipArgs<T> &A, int threads, int sm_count, cudaStream_t st) {
    constexpr int R = 64 / int(sizeof(T)), ELINE = 128 / int(sizeof(T));
    const int C = A.cluster;
    if (C != 1 && C != 2 && C != 4 && C != 8) return cudaErrorInvalidConfiguration;
    if (threads % 32 || threads > 512 || (C * (threads / 32) > 32 && threads < C * 16))
        return cudaErrorInvalidConfiguration;
    const int64_t rows = int64_t(threads) * R;
    const size_t smem = onchip_cpipe_smem_bytes(sizeof(T) == 4 ? TDS_F32 : TDS_F64, threads, C);
    auto kern = C == 8   ? onchip_cpipe_kernel<T, R, 8>
                : C == 4 ? onchip_cpipe_kernel<T, R, 4>
                : C == 2 ? onchip_cpipe_kernel<T, R, 2>
                         : onchip_cpipe_kernel<T, R, 1>;
    int occ = 1;  // CTAs per SM (C == 1) or clusters per device (C > 1)
    cudaError_t e = kernel_setup((const void *)kern, threads, smem, C, &occ);
    if (e != cudaSuccess) return e;
    // whole 128-byte lines of every system go by TMA (rows past them: LDG)
    const int64_t tma_lines = A.n / ELINE;
    if (tma_lines > 0x7fffffffLL || A.m_systems > 0x7fffffffLL) return cudaErrorInvalidConfiguration;
    TmapSet tm{}, tmx{};
    if (tma_lines > 0) {
        const T *arrs[5] = {A.a, A.b, A.c, A.d, A.x};
        for (int q = 0; q < 5; ++q)
            if (!encode_rows_tmap(q < 4 ? &tm.m[q] : &tmx.m[0], arrs[q], int(sizeof(T)), tma_lines, A.m_systems,
                                  A.batch_stride, int(rows / ELINE)))
                return cudaErrorInvalidValue;
    }
    int nclusters = C > 1 ? occ : std::max(occ, 1) * sm_count;
    nclusters = int(std::min<int64_t>(std::max(nclusters, 1), A.m_systems));
    e = launch_pdl(kern, dim3(unsigned(nclusters * C)), dim3(threads), smem, st, C, A, tm, int32_t(tma_lines), tmx);
    if (e != cudaSuccess) return e;
    return cudaGetLastError();
}

template cudaError_t launch_onchip_cpipe<float>(const OnchipArgs<float> &, int, int, cudaStream_t);
template cudaError_t launch_onchip_cpipe<double>(const OnchipArgs<double> &, int, int, cudaStream_t);

}  // namespace tds
