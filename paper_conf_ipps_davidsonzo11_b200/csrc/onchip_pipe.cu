// onchip_pipe.cu -- G2, persistent TMA-pipelined form (one CTA per SM).
//
// Same mathematics as onchip.cu with cluster = 1 (§III-A base kernel:
// c CR levels in registers, c2 CR levels across threads, PCR on the reduced
// system until T chains, Thomas per chain, back substitution), but the CTA is
// persistent and walks subsystems sigma = blockIdx.x, += gridDim.x.  While it
// solves subsystem i from registers, the Tensor Memory Accelerator streams
// subsystems i+1 and i+2 (three contiguous workspace arrays each) into a
// two-stage shared-memory ring with cp.async.bulk + mbarrier transaction
// counts, so HBM traffic never waits for the CR / PCR / Thomas phases.
//
// Shared memory -> registers: thread t owns 16-byte chunks 4t..4t+3 of each
// array (64 bytes, rows tR..tR+R-1).  Read in plain order, lanes 0,2,4,6 of a
// quarter-warp would hit the same bank group (4-way conflict); lane l instead
// reads chunk (q + l/2) mod 4 in instruction q, which is conflict-free, and a
// 4-way select puts every chunk back in its register slot.
#include <cooperative_groups.h>

#include <cstdlib>

#include "pipe.cuh"

namespace cg = cooperative_groups;

namespace tds {

// Ablation build (-DTDS_ONCHIP_ABLATION, diagnostics only -- results are wrong
// when a bit is set): env TDS_ONCHIP_ABLATION = 1 skip the solve, 2 skip the
// TMA loads, 4 skip the x stores.  Product builds compile TDS_OABL to false.
#ifdef TDS_ONCHIP_ABLATION
__constant__ int tds_onchip_ablation;
#define TDS_OABL(bit) ((tds_onchip_ablation & (bit)) != 0)
#else
#define TDS_OABL(bit) false
#endif

template <typename T, int ZR>
__device__ __forceinline__ void reduced_solve_pipe(T *z, int Z, int NT, int t, int log2T);

// Warp-level on-chip solve of one subsystem held as R rows per thread (x
// returned in rd).  c = log2(R) CR levels in registers, 5 CR levels across
// the lanes of each warp (shuffles), then the one remaining row per warp is
// solved with shuffle PCR, and everything is back-substituted.  The
// only row of a warp that reaches into the next warp is lane 31's: its chains
// are deferred until one barrier publishes the next warp's rows (lane 0's
// row s-1 per register level, lane s-1's row per lane level; both depend on
// nothing beyond their own warp).  Every warp then solves the one-row-per-warp
// system itself (no barrier to distribute its x).
// Row updates on the warp form's serial path (lane CR, the deferred chains,
// the top PCR): -DTDS_PIPE_SER_EARLY=1 uses the early operation order there
// (1 dependent op after the reciprocal); the register levels keep row_update.
// Measured neutral on config 3 (on-chip 52.8 vs 52.8 us, gpurun_out/r02b21).
#ifndef TDS_PIPE_SER_EARLY
#define TDS_PIPE_SER_EARLY 0
#endif
template <typename T>
__device__ __forceinline__ void row_update_ser(T &a, T &c, T &d, T al, T cl, T dl, T ar, T cr, T dr) {
    if constexpr (TDS_PIPE_SER_EARLY)
        row_update_early(a, c, d, al, cl, dl, ar, cr, dr);
    else
        row_update(a, c, d, al, cl, dl, ar, cr, dr);
}

template <typename T, int R, typename Hook>
__device__ __forceinline__ void solve_item_warp(T (&ra)[R], T (&rc)[R], T (&rd)[R], T *scr, int lane, int warp,
                                                int nwarps, Hook &&after_barrier) {
    constexpr int CR = ilog2c(R);
    constexpr unsigned FULL = 0xffffffffu;
    T *e_in = scr;                      // [nwarps][CR][3] lane 0's row s-1, level l-1
    T *w_in = e_in + nwarps * CR * 3;   // [nwarps][5][3]  lane s-1 at lane level l-1
    T *lft = w_in + nwarps * 15;        // [nwarps][5][3]  lane 31-s at lane level l-1
    T *top = lft + nwarps * 15;         // [3][32]
    T *xtop = top + 96;                 // [32]
    // register CR levels; lane 31 defers its row R-1 chain
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
        }
#pragma unroll
        for (int v = (1 << l) - 1; v < R; v += (1 << l)) {
            const bool last = v == R - 1;
            T a = ra[v], c = rc[v], d = rd[v];
            row_update(a, c, d, ra[v - s], rc[v - s], rd[v - s], last ? na : ra[(v + s) % R],
                       last ? nc : rc[(v + s) % R], last ? nd : rd[(v + s) % R]);
            const bool keep = last && lane == 31;  // select, not branch: no divergence
            ra[v] = keep ? ra[v] : a;
            rc[v] = keep ? rc[v] : c;
            rd[v] = keep ? rd[v] : d;
        }
    }
    // CR across lanes; lane 31 (kept at every level) defers
    T za = ra[R - 1], zc = rc[R - 1], zd = rd[R - 1];
#pragma unroll
    for (int l = 1; l <= 5; ++l) {
        const int s = 1 << (l - 1);
        const T la = __shfl_up_sync(FULL, za, s), lc = __shfl_up_sync(FULL, zc, s), ld = __shfl_up_sync(FULL, zd, s);
        const T xa = __shfl_down_sync(FULL, za, s), xc = __shfl_down_sync(FULL, zc, s),
                xd = __shfl_down_sync(FULL, zd, s);
        if (lane == s - 1) {
            T *w = w_in + (warp * 5 + l - 1) * 3;
            w[0] = za;
            w[1] = zc;
            w[2] = zd;
        }
        if (lane == 31 - s) {
            T *f = lft + (warp * 5 + l - 1) * 3;
            f[0] = za;
            f[1] = zc;
            f[2] = zd;
        }
        T na2 = za, nc2 = zc, nd2 = zd;
        row_update_ser(na2, nc2, nd2, la, lc, ld, xa, xc, xd);
        const bool upd = (lane & ((1 << l) - 1)) == (1 << l) - 1 && lane != 31;
        za = upd ? na2 : za;
        zc = upd ? nc2 : zc;
        zd = upd ? nd2 : zd;
    }
    __syncthreads();
    after_barrier();
    if (lane == 31) {  // the deferred chains, with the next warp's published rows
        const bool h = warp + 1 < nwarps;
#pragma unroll
        for (int l = 1; l <= CR; ++l) {
            const int s = 1 << (l - 1);
            const T *e = e_in + ((warp + 1) * CR + l - 1) * 3;
            row_update_ser(ra[R - 1], rc[R - 1], rd[R - 1], ra[R - 1 - s], rc[R - 1 - s], rd[R - 1 - s],
                       h ? e[0] : T(0), h ? e[1] : T(0), h ? e[2] : T(0));
        }
        za = ra[R - 1];
        zc = rc[R - 1];
        zd = rd[R - 1];
#pragma unroll
        for (int l = 1; l <= 5; ++l) {
            const T *f = lft + (warp * 5 + l - 1) * 3;
            const T *w = w_in + ((warp + 1) * 5 + l - 1) * 3;
            row_update_ser(za, zc, zd, f[0], f[1], f[2], h ? w[0] : T(0), h ? w[1] : T(0), h ? w[2] : T(0));
        }
        top[warp] = za;
        top[32 + warp] = zc;
        top[64 + warp] = zd;
    }
    __syncthreads();
    // one row per warp: pure PCR with shuffles (every row decouples, x = d),
    // solved redundantly by EVERY warp (identical arithmetic), so each warp
    // takes its own x and the previous warp's by shuffle -- no third barrier
    T xw, xprev;
    {
        T a = lane < nwarps ? top[lane] : T(0), c = lane < nwarps ? top[32 + lane] : T(0),
          d = lane < nwarps ? top[64 + lane] : T(0);
        for (int s = 1; s < nwarps; s <<= 1) {
            const T la = __shfl_up_sync(FULL, a, s), lc = __shfl_up_sync(FULL, c, s), ld = __shfl_up_sync(FULL, d, s);
            const T xa = __shfl_down_sync(FULL, a, s), xc = __shfl_down_sync(FULL, c, s),
                    xd = __shfl_down_sync(FULL, d, s);
            const bool hl = lane >= s, hr = lane + s < nwarps && !TDS_MUT(1, s >= 2);
            T na = a, nc = c, nd = d;
            row_update_ser(na, nc, nd, hl ? la : T(0), hl ? lc : T(0), hl ? ld : T(0), hr ? xa : T(0), hr ? xc : T(0),
                       hr ? xd : T(0));
            a = lane < nwarps ? na : a;
            c = lane < nwarps ? nc : c;
            d = lane < nwarps ? nd : d;
        }
        const T xme = __shfl_sync(FULL, d, warp);
        const T xpw = __shfl_sync(FULL, d, warp > 0 ? warp - 1 : 0);
        xw = lane == 31 ? xme : T(0);
        xprev = warp > 0 ? xpw : T(0);  // row -1 of this warp: previous warp's lane 31
    }
    (void)xtop;
    // back substitution across lanes, then in registers
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
}

template <typename T, int R, bool WL>
__global__ void __launch_bounds__(R * sizeof(T) == 32 ? 1024 : 512, 1)
    onchip_pipe_kernel(const OnchipArgs<T> A, int64_t nslots, const __grid_constant__ TmapSet tm, int32_t tma_lines) {
    static_assert(R * sizeof(T) == 64 || R * sizeof(T) == 32, "pipe kernel: 32 or 64 bytes of rows per thread");
    constexpr int ELINE = 128 / int(sizeof(T));
    extern __shared__ __align__(1024) unsigned char smem_raw[];
    __shared__ __align__(8) uint64_t full_bar[2];
    constexpr int CR = ilog2c(R);
    const int NT = blockDim.x;
    const int ROWS = NT * R;
    const int t = threadIdx.x, lane = t & 31, warp = t >> 5, nwarps = NT >> 5;
    const int c2 = A.tl_levels;
    const int Z = NT >> c2;
    T *stage0 = reinterpret_cast<T *>(smem_raw + ((1024u - (smem_u32(smem_raw) & 1023u)) & 1023u));  // [2][3][ROWS]
    T *z = stage0 + 6 * ROWS;                      // [3][Z]
    T *ya = z + 3 * Z;                             // [4][NT]
    T *yc = ya + NT, *yd = yc + NT, *yx = yd + NT;
    T *edge = yx + NT;                             // [2][3][nwarps]
    const int64_t KK = int64_t(1) << A.K;

    auto slot_len = [&](int64_t sigma) -> int64_t {
        const int64_t r = sigma & (KK - 1);
        return r < A.n ? (A.n - r + KK - 1) >> A.K : 0;
    };
    const int64_t tma_rows = int64_t(tma_lines) * ELINE;  // rows of every slot in whole TMA lines
    // workspace slots are read once (evict first); x slots are re-read by place_x (evict last)
    auto ld_ws = [&](T *dst, const CUtensorMap *map, int slot, uint64_t *bar) {
        if constexpr ((TDS_L2HINT & 1) != 0)
            tma_load_lines_hint(dst, map, 0, slot, bar, l2_evict_first());
        else
            tma_load_lines(dst, map, 0, slot, bar);
    };
    auto st_x = [&](const T *src, int slot) {
        if (TDS_OABL(4)) return;
        if constexpr ((TDS_L2HINT & 2) != 0)
            tma_store_lines_hint(&tm.m[0], src, 0, slot, l2_evict_last());
        else
            tma_store_lines(&tm.m[0], src, 0, slot);
    };
    // work item q solves slot nslots-1-q: the split pass wrote the last slots
    // last, so the first items a CTA waits for are still in L2
    // One swizzled box of ROWS rows per array (lines past the slot are
    // zero-filled).  The a-region of a consumed stage first holds the item's x
    // for the TMA store (x overwrites a in the workspace), so a stage is
    // refilled in two steps: c and d as soon as the stage is in registers,
    // a once the previous x store has read it.
    auto issue_cd = [&](int64_t q, int s) {  // thread 0 only; announces all three arrays
        if (q >= nslots || TDS_OABL(2)) return;
        const int64_t sigma = nslots - 1 - q;
        uint64_t *bar = &full_bar[s];
        if (tma_lines == 0) {
            mbar_expect_tx(bar, 0);
            return;
        }
        mbar_expect_tx(bar, 3 * uint32_t(ROWS) * sizeof(T));
        T *dst = stage0 + size_t(s) * 3 * ROWS;
        ld_ws(dst + ROWS, &tm.m[1], int(sigma), bar);
        ld_ws(dst + 2 * ROWS, &tm.m[2], int(sigma), bar);
    };
    auto issue_a = [&](int64_t q, int s) {  // thread 0 only
        if (q >= nslots || tma_lines == 0 || TDS_OABL(2)) return;
        ld_ws(stage0 + size_t(s) * 3 * ROWS, &tm.m[0], int(nslots - 1 - q), &full_bar[s]);
    };
    pdl_wait();  // the previous kernel on the stream is complete before any global access
    if (t == 0) {
        mbar_init(&full_bar[0], 1);
        mbar_init(&full_bar[1], 1);
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
        issue_cd(blockIdx.x, 0);
        issue_a(blockIdx.x, 0);
        issue_cd(int64_t(blockIdx.x) + gridDim.x, 1);
        issue_a(int64_t(blockIdx.x) + gridDim.x, 1);
    }
    __syncthreads();
    int64_t pend = -1;  // slot whose x waits in the a-region of stage 1-s for its TMA store

    for (int64_t it = 0;; ++it) {
        const int64_t q = int64_t(blockIdx.x) + it * gridDim.x;
        if (q >= nslots) break;
        pdl_trigger_if_last(q + gridDim.x >= nslots);
        const int64_t sigma = nslots - 1 - q;
        const int s = int(it & 1);
        const int64_t L = slot_len(sigma);
        if (!TDS_OABL(2)) mbar_wait(&full_bar[s], uint32_t((it >> 1) & 1));
        T *sb = stage0 + size_t(s) * 3 * ROWS;
        if (L > tma_rows || tma_lines == 0) {
            // CTA-uniform: rows [tma_rows, L) by LDG; with no TMA at all also zero the rest
            const int64_t hi = tma_lines == 0 ? ROWS : L;
            for (int64_t j = tma_rows + t; j < hi; j += NT) {
                const int o = sw_off<T>(int(j));
                const bool in = j < L;
                const int64_t g = sigma * A.slot + j;
                sb[o] = in ? A.a[g] : T(0);
                sb[ROWS + o] = in ? A.c[g] : T(0);
                sb[2 * ROWS + o] = in ? A.d[g] : T(0);
            }
            asm volatile("fence.proxy.async.shared::cta;" ::: "memory");  // before the next TMA refill
            __syncthreads();
        }
        if (A.l2_discard) {  // c', d' of this slot are dead once in shared memory
            const int nl = int(min(L, tma_rows) / ELINE);
            for (int li = t; li < 2 * nl; li += NT)
                l2_discard_line((li < nl ? A.c : A.d) + sigma * A.slot + int64_t(li < nl ? li : li - nl) * ELINE);
        }
        const int64_t jt = int64_t(t) * R;
        T ra[R], rc[R], rd[R];
        lds_rows_sw<T, R>(sb, t * R, ra);
        lds_rows_sw<T, R>(sb + ROWS, t * R, rc);
        lds_rows_sw<T, R>(sb + 2 * ROWS, t * R, rd);
        __syncthreads();  // every thread has read stage s (and written the previous item's x)
        if (t == 0) {
            issue_cd(q + 2 * int64_t(gridDim.x), s);
            if (pend >= 0) {  // the previous item's x: one tensor store from the a-region of stage 1-s
                st_x(stage0 + size_t(1 - s) * 3 * ROWS, int(pend));
                bulk_commit();
            }
        }
        const bool had_pend = pend >= 0;
        pend = -1;
        // once the store has read the region (checked after the solve's first
        // barrier), stage 1-s gets its a-array for item q + G
        auto refill_a = [&]() {
            if (t == 0 && had_pend) {
                bulk_wait_read0();
                issue_a(q + int64_t(gridDim.x), 1 - s);
            }
        };
        if (L == 0) {  // empty slot (2^K > n): uniform
            refill_a();
            continue;
        }

        if constexpr (WL) {
            if (!TDS_OABL(1))
                solve_item_warp<T, R>(ra, rc, rd, ya, lane, warp, nwarps, refill_a);
            else
                refill_a();
        } else {
        refill_a();
        // ---- B1. CR forward levels in registers
#pragma unroll
        for (int l = 1; l <= CR; ++l) {
            const int sl = 1 << (l - 1);
            const T pa = ra[sl - 1], pc = rc[sl - 1], pd = rd[sl - 1];
            T na = __shfl_down_sync(0xffffffffu, pa, 1);
            T nc = __shfl_down_sync(0xffffffffu, pc, 1);
            T nd = __shfl_down_sync(0xffffffffu, pd, 1);
            T *eb = edge + (l & 1) * 3 * nwarps;
            if (lane == 0) {
                eb[warp] = pa;
                eb[nwarps + warp] = pc;
                eb[2 * nwarps + warp] = pd;
            }
            __syncthreads();
            if (lane == 31) {
                const bool h = warp + 1 < nwarps;
                na = h ? eb[warp + 1] : T(0);
                nc = h ? eb[nwarps + warp + 1] : T(0);
                nd = h ? eb[2 * nwarps + warp + 1] : T(0);
            }
#pragma unroll
            for (int v = (1 << l) - 1; v < R; v += (1 << l)) {
                const bool last = (v == R - 1);
                row_update(ra[v], rc[v], rd[v], ra[v - sl], rc[v - sl], rd[v - sl], last ? na : ra[(v + sl) % R],
                           last ? nc : rc[(v + sl) % R], last ? nd : rd[(v + sl) % R]);
            }
        }
        // ---- B2. c2 CR levels across threads
        ya[t] = ra[R - 1];
        yc[t] = rc[R - 1];
        yd[t] = rd[R - 1];
        for (int l = 1; l <= c2; ++l) {
            const int sl = 1 << (l - 1);
            __syncthreads();
            if ((t & ((1 << l) - 1)) == (1 << l) - 1) {
                T a = ya[t], c = yc[t], d = yd[t];
                const bool hr = t + sl < NT;
                row_update(a, c, d, ya[t - sl], yc[t - sl], yd[t - sl], hr ? ya[t + sl] : T(0),
                           hr ? yc[t + sl] : T(0), hr ? yd[t + sl] : T(0));
                ya[t] = a;
                yc[t] = c;
                yd[t] = d;
            }
        }
        __syncthreads();
        // ---- C. the CTA's remaining Z rows: PCR until T chains, Thomas per chain
        const bool top = (t & ((1 << c2) - 1)) == (1 << c2) - 1;
        const int zi = t >> c2;
        if (top) {
            z[zi] = ya[t];
            z[Z + zi] = yc[t];
            z[2 * Z + zi] = yd[t];
        }
        __syncthreads();
        reduced_solve_pipe<T, 1>(z, Z, NT, t, A.log2T);
        if (top) yx[t] = z[2 * Z + zi];
        // ---- D. back substitution across threads, then in registers
        for (int l = c2; l >= 1; --l) {
            const int sl = 1 << (l - 1);
            __syncthreads();
            if ((t & ((1 << l) - 1)) == sl - 1) {
                const T xl = t >= sl ? yx[t - sl] : T(0);
                yx[t] = yd[t] - ya[t] * xl - yc[t] * yx[t + sl];
            }
        }
        __syncthreads();
        rd[R - 1] = yx[t];
        const T xleft = t > 0 ? yx[t - 1] : T(0);
#pragma unroll
        for (int l = CR; l >= 1; --l) {
            const int sl = 1 << (l - 1);
#pragma unroll
            for (int v = sl - 1; v < R - 1; v += 2 * sl) {
                const T xlv = (v >= sl) ? rd[(v - sl + R) % R] : xleft;
                rd[v] = rd[v] - ra[v] * xlv - rc[v] * rd[(v + sl) % R];
            }
        }
        }  // !WL
        T *dst = A.xs + sigma * A.slot + jt;  // per-subsystem x (placement kernel follows)
        if (tma_lines > 0) {
            // x to the a-region of stage s (swizzled like the loads); the next
            // item's first barrier makes it complete, then thread 0 stores it.
            // Rows past the tensor's whole lines go straight to global memory.
            sts_rows_sw<T, R>(sb, t * R, rd);
            fence_proxy_async_smem();
            if (jt + R > tma_rows) {
#pragma unroll
                for (int v = 0; v < R; ++v)
                    if (jt + v >= tma_rows && jt + v < L) dst[v] = rd[v];
            }
            pend = sigma;
        } else if (jt + R <= L) {
            constexpr int W = 16 / int(sizeof(T));
#pragma unroll
            for (int q = 0; q < R / W; ++q) {
                if constexpr (sizeof(T) == 4)
                    __stcs(reinterpret_cast<float4 *>(dst) + q,
                           make_float4(rd[4 * q], rd[4 * q + 1], rd[4 * q + 2], rd[4 * q + 3]));
                else
                    __stcs(reinterpret_cast<double2 *>(dst) + q, make_double2(rd[2 * q], rd[2 * q + 1]));
            }
        } else {
#pragma unroll
            for (int v = 0; v < R; ++v)
                if (jt + v < L) dst[v] = rd[v];
        }
        // no barrier here: the next item's first shared-scratch write follows its
        // stage-consumed barrier, which every thread reaches only after this item
    }
    __syncthreads();  // the last item's x is complete in shared memory
    if (t == 0) {
        if (pend >= 0) {
            // the stage index of the last item: it = number of items - 1
            const int64_t nit = (nslots - int64_t(blockIdx.x) + gridDim.x - 1) / gridDim.x;
            st_x(stage0 + size_t((nit - 1) & 1) * 3 * ROWS, int(pend));
            bulk_commit();
        }
        bulk_wait_all();
    }
}

// PCR until 2^log2T chains, then Thomas per chain, on Z <= ZR * NT rows in z.
template <typename T, int ZR>
__device__ __forceinline__ void reduced_solve_pipe(T *z, int Z, int NT, int t, int log2T) {
    T *za = z, *zc = z + Z, *zd = z + 2 * Z;
    for (int j = 0; j < log2T; ++j) {
        const int s = 1 << j;
        T na[ZR], nc[ZR], nd[ZR];
#pragma unroll
        for (int q = 0; q < ZR; ++q) {
            const int i = t + q * NT;
            if (i < Z) {
                T a = za[i], c = zc[i], d = zd[i];
                const bool hl = i >= s, hr = i + s < Z && !TDS_MUT(4, s >= 4);
                row_update(a, c, d, hl ? za[i - s] : T(0), hl ? zc[i - s] : T(0), hl ? zd[i - s] : T(0),
                           hr ? za[i + s] : T(0), hr ? zc[i + s] : T(0), hr ? zd[i + s] : T(0));
                na[q] = a;
                nc[q] = c;
                nd[q] = d;
            }
        }
        __syncthreads();
#pragma unroll
        for (int q = 0; q < ZR; ++q) {
            const int i = t + q * NT;
            if (i < Z) {
                za[i] = na[q];
                zc[i] = nc[q];
                zd[i] = nd[q];
            }
        }
        __syncthreads();
    }
    const int TC = 1 << log2T;
    for (int ch = t; ch < TC && ch < Z; ch += NT) {
        T cp = zc[ch], dp = zd[ch];
        int q = ch;
        for (int qn = ch + TC; qn < Z; qn += TC) {
            const T aq = za[qn];
            const T w = rcp(fma(-aq, cp, T(1)));
            cp = zc[qn] * w;
            dp = (zd[qn] - aq * dp) * w;
            zc[qn] = cp;
            zd[qn] = dp;
            q = qn;
        }
        T xv = dp;
        for (int qp = q - TC; qp >= ch; qp -= TC) {
            xv = zd[qp] - zc[qp] * xv;
            zd[qp] = xv;
        }
    }
    __syncthreads();
}

// ---- fused x placement (plan x_group = G > 0): a cluster of G persistent
// CTAs walks groups of G adjacent residue classes r0 .. r0+G-1 of one system
// (slots sys 2^K + r, Fig. 3a) in lock step, one class per CTA.
// Row j of class r0+q is original row r0 + q + 2^K j, so the G classes
// together own G-element runs of x.  After the solve, every thread pushes its
// R rows of x (st.async, 16 bytes each) into the a-region of the consumed stage
// of the CTA that stores rows [p SEG, (p+1) SEG) of the group (SEG = rows/G),
// class-major; that CTA transposes the block in place to [row][class] and
// writes it with TMA tensor stores of {G classes x box_rows rows} boxes of the
// x view {2^K, n/2^K, m}: whole G-element runs, no placement kernel, no x-slot
// round trip.  Hand-offs are point-to-point mbarriers (no cluster barrier in
// the loop): x_full counts the bytes pushed into this CTA, ready[p] tells a
// pusher that CTA p has consumed its stage for this item.
// Measured on B200 (profiles/r01h_xgroup.md): bit-identical to the separate
// placement but SLOWER (config 3: 193 us vs 159 us per solve) -- DSMEM moves
// ~20 B/clk per SM, so pushing 32 KB of x per item costs more than place_x's
// L2 round trip, and 1-CTA/SM clusters of 4 / 8 fit only 132 / 120 of the 148
// SMs.  Kept as a tuner dimension (tds_tune tries it; it does not win).
// Direct G-element STG runs instead of the TMA boxes measured slower still.
template <typename T, int R, int G>
__global__ void __launch_bounds__(512, 1)
    onchip_gpipe_kernel(const OnchipArgs<T> A, int64_t ngroups, const __grid_constant__ TmapSet tm,
                        const __grid_constant__ TmapSet tmx, int32_t box_rows) {
    static_assert(R * sizeof(T) == 64, "gpipe kernel: 64 bytes of rows per thread");
    static_assert(R % G == 0 && G * sizeof(T) >= 16, "gpipe kernel: whole 16-byte runs");
    constexpr int ELINE = 128 / int(sizeof(T));
    constexpr int E16 = 16 / int(sizeof(T));  // elements per 16-byte push
    constexpr int PER = R / G;                 // segment rows per thread in the transpose
    extern __shared__ __align__(1024) unsigned char smem_raw[];
    __shared__ __align__(8) uint64_t full_bar[2];
    __shared__ __align__(8) uint64_t x_full;    // x runs of this item pushed into this CTA (bytes)
    __shared__ __align__(8) uint64_t ready[G];  // ready[p]: CTA p consumed its stage (this item)
    const int NT = blockDim.x;
    const int ROWS = NT * R, SEG = ROWS / G;
    const int t = threadIdx.x, lane = t & 31, warp = t >> 5, nwarps = NT >> 5;
    const int rank = int(blockIdx.x % G);
    const int64_t cid = blockIdx.x / G, ncl = gridDim.x / G;
    T *stage0 = reinterpret_cast<T *>(smem_raw + ((1024u - (smem_u32(smem_raw) & 1023u)) & 1023u));  // [2][3][ROWS]
    T *scr = stage0 + 6 * ROWS;
    const int64_t KK = int64_t(1) << A.K;
    auto slot_of = [&](int64_t it) -> int64_t {  // groups walked last-first (the split wrote them last)
        const int64_t g = cid + it * ncl;
        return g < ngroups ? (ngroups - 1 - g) * G + rank : -1;
    };
    auto ld_ws = [&](T *dst, const CUtensorMap *map, int64_t slot, uint64_t *bar) {
        if constexpr ((TDS_L2HINT & 1) != 0)
            tma_load_lines_hint(dst, map, 0, int(slot), bar, l2_evict_first());
        else
            tma_load_lines(dst, map, 0, int(slot), bar);
    };
    auto issue_cd = [&](int64_t it, int s) {  // thread 0; announces all three arrays
        const int64_t sl = slot_of(it);
        if (sl < 0) return;
        mbar_expect_tx(&full_bar[s], 3 * uint32_t(ROWS) * sizeof(T));
        T *dst = stage0 + size_t(s) * 3 * ROWS;
        ld_ws(dst + ROWS, &tm.m[1], sl, &full_bar[s]);
        ld_ws(dst + 2 * ROWS, &tm.m[2], sl, &full_bar[s]);
    };
    auto issue_a = [&](int64_t it, int s) {  // thread 0
        const int64_t sl = slot_of(it);
        if (sl >= 0) ld_ws(stage0 + size_t(s) * 3 * ROWS, &tm.m[0], sl, &full_bar[s]);
    };
    pdl_wait();  // the split pass is complete before any global access
    if (t == 0) {
        mbar_init(&full_bar[0], 1);
        mbar_init(&full_bar[1], 1);
        mbar_init(&x_full, 1);
#pragma unroll
        for (int q = 0; q < G; ++q) mbar_init(&ready[q], 1);
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
        issue_cd(0, 0);
        issue_a(0, 0);
        issue_cd(1, 1);
        issue_a(1, 1);
    }
    cg::this_cluster().sync();  // every CTA runs (mbarriers initialised) before any DSMEM access
    const int own = (t * R) / SEG;  // CTA storing this thread's rows
    const uint32_t r_xfull = cluster_addr(&x_full, own);
    const uint32_t r_ready = t < G ? cluster_addr(&ready[rank], t) : 0u;

    for (int64_t it = 0;; ++it) {
        const int64_t sigma = slot_of(it);
        if (sigma < 0) break;
        const int s = int(it & 1);
        const uint32_t ph = uint32_t(it & 1);
        if (t == 0) mbar_expect_tx(&x_full, uint32_t(ROWS) * sizeof(T));
        mbar_wait(&full_bar[s], uint32_t((it >> 1) & 1));
        T *sb = stage0 + size_t(s) * 3 * ROWS;
        if (A.l2_discard) {  // c', d' of this slot are dead once in shared memory
            const int nl = ROWS / ELINE;
            for (int li = t; li < 2 * nl; li += NT)
                l2_discard_line((li < nl ? A.c : A.d) + sigma * A.slot + int64_t(li < nl ? li : li - nl) * ELINE);
        }
        T ra[R], rc[R], rd[R];
        lds_rows_sw<T, R>(sb, t * R, ra);
        lds_rows_sw<T, R>(sb + ROWS, t * R, rc);
        lds_rows_sw<T, R>(sb + 2 * ROWS, t * R, rd);
        __syncthreads();  // stage s consumed: its a-region now takes this item's x runs
        if (t == 0) issue_cd(it + 2, s);
        if (t < G) mbar_arrive_remote(r_ready);  // relaxed: the stage's reads are complete (barrier above)
        // the previous item's x store (stage 1-s) has read its region before the a-refill
        auto refill_a = [&]() {
            if (t == 0 && it > 0) {
                bulk_wait_read0();
                issue_a(it + 1, 1 - s);
            }
        };
        solve_item_warp<T, R>(ra, rc, rd, scr, lane, warp, nwarps, refill_a);
        // push rows tR .. tR+R-1 of class rank+r0 to CTA `own`, block [G][SEG]
        mbar_wait(&ready[own], ph);  // CTA scope: no L1 invalidation (CCTL.IVALL) per item
        const uint32_t dst = cluster_addr(sb + rank * SEG + (t * R - own * SEG), own);
#pragma unroll
        for (int q = 0; q < R / E16; ++q) st_async16(dst + 16 * q, rd + q * E16, r_xfull);
        mbar_wait(&x_full, ph);  // the G classes' runs of this CTA's segment (st.async complete_tx)
        T v[PER][G];
#pragma unroll
        for (int i = 0; i < PER; ++i)
#pragma unroll
            for (int q = 0; q < G; ++q) v[i][q] = sb[q * SEG + t + i * NT];
        __syncthreads();  // in place: every read precedes every write
#pragma unroll
        for (int i = 0; i < PER; ++i) {
            T *row = sb + (t + i * NT) * G;
#pragma unroll
            for (int q = 0; q < G; q += E16) {
                if constexpr (sizeof(T) == 4)
                    *reinterpret_cast<float4 *>(row + q) = make_float4(v[i][q], v[i][q + 1], v[i][q + 2], v[i][q + 3]);
                else
                    *reinterpret_cast<double2 *>(row + q) = make_double2(v[i][q], v[i][q + 1]);
            }
        }
        fence_proxy_async_smem();
        __syncthreads();
        if (t == 0) {
            const int sys = int(sigma >> A.K), r0 = int((sigma & (KK - 1)) - rank);
            for (int b = 0; b * box_rows < SEG; ++b)
                tma_store_box3(&tmx.m[0], sb + size_t(b) * box_rows * G, r0, rank * SEG + b * box_rows, sys);
            bulk_commit();
        }
    }
    if (t == 0) bulk_wait_all();
    cg::this_cluster().sync();  // no CTA leaves while a peer may still push into it
}

// ---- the paper's strided base-kernel variant (plan strided = 1):
// the split pass left the 2^K subsystems interleaved in place (row i of
// system s at a'[s * stride + i]), so subsystem (s, r) is gathered with
// stride 2^K straight into registers (scalar loads; a warp's loads touch 32
// different sectors) and its x is scattered the same way into the caller's
// array -- no de-interleave, no x slots, no placement kernel, no TMA (the
// rows of one subsystem are not contiguous).  Same arithmetic as the warp
// form of the pipe kernel (solve_item_warp), so x is bit-identical to the
// de-interleaved path under the same plan.  Persistent, one subsystem per CTA
// at a time.
template <typename T, int R>
__global__ void __launch_bounds__(512, 1)
    onchip_strided_kernel(const OnchipArgs<T> A, int64_t nslots, int64_t ws_stride) {
    extern __shared__ __align__(16) unsigned char smem_raw[];
    T *scr = reinterpret_cast<T *>(smem_raw);
    const int NT = blockDim.x, t = threadIdx.x, lane = t & 31, warp = t >> 5, nwarps = NT >> 5;
    const int64_t KK = int64_t(1) << A.K;
    pdl_wait();  // the split pass is complete before any global access
    for (int64_t q = blockIdx.x; q < nslots; q += gridDim.x) {
        const int64_t sys = q >> A.K, r = q & (KK - 1);
        const int64_t L = r < A.n ? (A.n - r + KK - 1) >> A.K : 0;
        if (L == 0) continue;  // CTA-uniform
        const int64_t jt = int64_t(t) * R, g0 = sys * ws_stride + r;
        T ra[R], rc[R], rd[R];
#pragma unroll
        for (int v = 0; v < R; ++v) {
            const bool in = jt + v < L;  // rows past the subsystem: identity (0, 1, 0, 0)
            const int64_t g = g0 + (jt + v) * KK;
            ra[v] = in ? __ldcs(A.a + g) : T(0);
            rc[v] = in ? __ldcs(A.c + g) : T(0);
            rd[v] = in ? __ldcs(A.d + g) : T(0);
        }
        solve_item_warp<T, R>(ra, rc, rd, scr, lane, warp, nwarps, [] {});
        T *x = A.x + sys * A.batch_stride + r;
#pragma unroll
        for (int v = 0; v < R; ++v)
            if (jt + v < L) x[(jt + v) * KK] = rd[v];
    }
}

template <typename T>
cudaError_t launch_onchip_strided(const OnchipArgs<T> &A, int64_t nslots, int threads, int64_t ws_stride,
                                  cudaStream_t st) {
    constexpr int R = 64 / int(sizeof(T));
    if (threads % 32 || threads > 512 || nslots > 0x7fffffffLL) return cudaErrorInvalidConfiguration;
    const int nw = threads / 32;
    const size_t smem = size_t(nw * (3 * ilog2c(R) + 30) + 128) * sizeof(T);
    auto kern = onchip_strided_kernel<T, R>;
    int occ = 1;
    cudaError_t e = kernel_setup((const void *)kern, threads, smem, 1, &occ);
    if (e != cudaSuccess) return e;
    const int64_t grid = std::min<int64_t>(nslots, int64_t(std::max(occ, 1)) * sm_count_current());
    e = launch_pdl(kern, dim3(unsigned(std::max<int64_t>(grid, 1))), dim3(threads), smem, st, 1, A, nslots,
                   ws_stride);
    if (e != cudaSuccess) return e;
    return cudaGetLastError();
}

template cudaError_t launch_onchip_strided<float>(const OnchipArgs<float> &, int64_t, int, int64_t, cudaStream_t);
template cudaError_t launch_onchip_strided<double>(const OnchipArgs<double> &, int64_t, int, int64_t, cudaStream_t);

size_t onchip_gpipe_smem_bytes(int32_t dtype, int32_t threads) {
    const int64_t R = 64 / dsize(dtype), nw = threads / 32;
    return 1024 + size_t((6 * int64_t(threads) * R + nw * (3 * ilog2c(int(R)) + 30) + 128 + 8) * dsize(dtype));
}

template <typename T>
cudaError_t launch_onchip_gpipe(const OnchipArgs<T> &A, int64_t nslots, int threads, int sm_count, cudaStream_t st) {
    constexpr int R = 64 / int(sizeof(T)), ELINE = 128 / int(sizeof(T));
    (void)sm_count;
    const int G = A.x_group;
    const int64_t rows = int64_t(threads) * R, L = A.n >> A.K;
    if ((G != 2 && G != 4 && G != 8) || G * int(sizeof(T)) < 16 || L != rows || rows % (G * ELINE) || nslots % G ||
        threads % 32 || threads > 512)
        return cudaErrorInvalidConfiguration;
    const int64_t seg = rows / G;
    const int box_rows = int(std::min<int64_t>(seg, 256));
    if (seg % box_rows || nslots > 0x7fffffffLL || A.m_systems > 0x7fffffffLL || A.K > 30)
        return cudaErrorInvalidConfiguration;
    const size_t smem = onchip_gpipe_smem_bytes(sizeof(T) == 4 ? TDS_F32 : TDS_F64, threads);
    void (*kern)(const OnchipArgs<T>, int64_t, const TmapSet, const TmapSet, int32_t) = nullptr;
    if (G == 8) kern = onchip_gpipe_kernel<T, R, 8>;
    else if (G == 4) kern = onchip_gpipe_kernel<T, R, 4>;
    else if constexpr (sizeof(T) == 8) kern = onchip_gpipe_kernel<T, R, 2>;
    if (!kern) return cudaErrorInvalidConfiguration;
    int occ = 1;  // resident clusters per device
    cudaError_t e = kernel_setup((const void *)kern, threads, smem, G, &occ);
    if (e != cudaSuccess) return e;
    TmapSet tm{}, tmx{};
    const T *arrs[3] = {A.a, A.c, A.d};
    for (int q = 0; q < 3; ++q)
        if (!encode_rows_tmap(&tm.m[q], arrs[q], int(sizeof(T)), rows / ELINE, nslots, A.slot, int(rows / ELINE)))
            return cudaErrorInvalidValue;
    const uint64_t dims[3] = {uint64_t(1) << A.K, uint64_t(L), uint64_t(A.m_systems)};
    const uint64_t strides[2] = {(uint64_t(1) << A.K) * sizeof(T), uint64_t(A.batch_stride) * sizeof(T)};
    const uint32_t box[3] = {uint32_t(G), uint32_t(box_rows), 1};
    if (!encode_box3_tmap_plain(&tmx.m[0], A.x, int(sizeof(T)), dims, strides, box)) return cudaErrorInvalidValue;
    const int64_t ngroups = nslots / G;
    const int64_t ncl = std::min<int64_t>(std::max(occ, 1), ngroups);
    e = launch_pdl(kern, dim3(unsigned(ncl * G)), dim3(threads), smem, st, G, A, ngroups, tm, tmx,
                   int32_t(box_rows));
    if (e != cudaSuccess) return e;
    return cudaGetLastError();
}

template cudaError_t launch_onchip_gpipe<float>(const OnchipArgs<float> &, int64_t, int, int, cudaStream_t);
template cudaError_t launch_onchip_gpipe<double>(const OnchipArgs<double> &, int64_t, int, int, cudaStream_t);

size_t onchip_pipe_smem_bytes(int32_t dtype, int32_t threads, int32_t R, int32_t tl_levels) {
    const int64_t rows = int64_t(threads) * R;
    return 1024 + size_t((6 * rows + 3 * (threads >> tl_levels) + 4 * int64_t(threads) + 6 * (threads / 32) + 8) *
                         dsize(dtype));
}

template <typename T>
cudaError_t launch_onchip_pipe(const OnchipArgs<T> &A, int64_t nslots, int threads, int cr_levels, int sm_count,
                               size_t smem, cudaStream_t st) {
    // tl_levels == 5 (CR across all 32 lanes) selects the warp-level shuffle path
    constexpr int RW = 64 / int(sizeof(T)), RN = 32 / int(sizeof(T));
    const bool wide = (1 << cr_levels) == RW;
    auto kern = wide ? (A.tl_levels == 5 ? onchip_pipe_kernel<T, RW, true> : onchip_pipe_kernel<T, RW, false>)
                     : (A.tl_levels == 5 ? onchip_pipe_kernel<T, RN, true> : onchip_pipe_kernel<T, RN, false>);
    int occ = 1;  // smaller subsystems fit two or more persistent CTAs per SM
    cudaError_t e = kernel_setup((const void *)kern, threads, smem, 1, &occ);
    if (e != cudaSuccess) return e;
    const int64_t grid = std::min<int64_t>(nslots, int64_t(std::max(occ, 1)) * sm_count);
    // every slot holds at least n >> K rows: that many whole 128-byte lines go by TMA
    constexpr int ELINE = 128 / int(sizeof(T));
    const int64_t rows = int64_t(threads) * (wide ? RW : RN);
    const int64_t tma_lines = std::min<int64_t>((A.n >> A.K) / ELINE, rows / ELINE);
    if (nslots > 0x7fffffffLL) return cudaErrorInvalidConfiguration;
    TmapSet tm{};
    if (tma_lines > 0) {
        const T *arrs[3] = {A.a, A.c, A.d};
        for (int q = 0; q < 3; ++q)
            if (!encode_rows_tmap(&tm.m[q], arrs[q], int(sizeof(T)), tma_lines, nslots, A.slot, int(rows / ELINE)))
                return cudaErrorInvalidValue;
    }
#ifdef TDS_ONCHIP_ABLATION
    {
        const char *ab = std::getenv("TDS_ONCHIP_ABLATION");
        const int v = ab ? std::atoi(ab) : 0;
        cudaMemcpyToSymbolAsync(tds_onchip_ablation, &v, sizeof(int), 0, cudaMemcpyHostToDevice, st);
    }
#endif
    cudaError_t le = launch_pdl(kern, dim3(unsigned(grid)), dim3(threads), smem, st, 1, A, nslots, tm,
                                int32_t(tma_lines));
    if (le != cudaSuccess) return le;
    return cudaGetLastError();
}

template cudaError_t launch_onchip_pipe<float>(const OnchipArgs<float> &, int64_t, int, int, int, size_t,
                                               cudaStream_t);
template cudaError_t launch_onchip_pipe<double>(const OnchipArgs<double> &, int64_t, int, int, int, size_t,
                                                cudaStream_t);

}  // namespace tds
