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
#include <cstdlib>

namespace tds {

// Ablation build (-DTDS_SPLIT_ABLATION, diagnostics only -- results are wrong
// when a bit is set): env TDS_SPLIT_ABLATION = 1 skip the PCR levels, 2 skip
// the TMA loads, 4 skip the TMA stores.  Product builds compile TDS_ABL to false.
#ifdef TDS_SPLIT_ABLATION
__constant__ int tds_split_ablation;
#define TDS_ABL(bit) ((tds_split_ablation & (bit)) != 0)
#else
#define TDS_ABL(bit) false
#endif

// Experiment switch (-DTDS_SPLIT_STG=1): the tile's outputs leave by vector
// STG from registers instead of shared-memory staging + TMA tensor stores.
#ifndef TDS_SPLIT_STG
#define TDS_SPLIT_STG 0
#endif
// NB is rounded so a residue's positions per tile are whole 16-byte TMA store
// rows for every CTA size (256-thread k_p = 8: 13 -> 12 B-blocks, so fp64 and
// 256-thread fp32 tiles leave by TMA tensor stores instead of per-residue
// scalar STG with 64-bit address arithmetic: config 3 fp64 split 0.285 ->
// 0.269 ms, gpurun_out/r02i).  -DTDS_SPLIT_NBQ_ALL=0 restores the old rule.
#ifndef TDS_SPLIT_NBQ_ALL
#define TDS_SPLIT_NBQ_ALL 1
#endif
// fp64 class transpose in ONE round for the three arrays (class-major
// [3][16][AV] buffer, XOR-swizzled 16-byte chunks, 92 KB) instead of three
// rounds through one buffer (6 barriers per tile): 252 -> 212 registers,
// config 3 fp64 split 0.277 -> 0.268 ms (gpurun_out/r02j).
// -DTDS_SPLIT_TRC64=0 restores the three-round transpose.
#ifndef TDS_SPLIT_TRC64
#define TDS_SPLIT_TRC64 1
#endif
// fp32 512-thread and fp64 256-thread tiles: the bank-conflict-free sub-row class
// transpose (split_reg.cuh, Tr34); -DTDS_SPLIT_TR34=0 restores the swizzled [rho][m] rows.
#ifndef TDS_SPLIT_TR34
#define TDS_SPLIT_TR34 1
#endif
// Experiment switch (-DTDS_SPLIT_WSTORE=1), fp32 512-thread sub-row tiles: every warp
// (one residue class rho mod 16) stages its outputs in its own class rows of the
// transpose buffer and stores them by its own 5-D TMA tensor store -- no CTA barrier
// between the layout-B levels and the stores.  Correct (300 split / coupling / fuzz GPU
// tests) but slower: config 3 split 101.5 vs 97.0 us (48 stores of 1.8 KB per tile
// instead of 3 of 28 KB; gpurun_out/r02b22, profiles/r02b22/).  Default off.
#ifndef TDS_SPLIT_WSTORE
#define TDS_SPLIT_WSTORE 0
#endif

template <int KP, int NT_>
struct SplitShape {
    static constexpr int R = kRegSplitRows;
    static constexpr int NT = NT_;                      // 256 (2 CTAs/SM) or 512 (1 CTA/SM, less halo)
    static constexpr int CH = NT / 16;                  // lanes per layout-B chain (shuffle width)
    static constexpr int NW = NT / 32;
    static constexpr int AV = 30 * NW;          // valid A-blocks per window
    static constexpr int ROWS = (AV + 2) * R;   // window rows (A-blocks 0 .. AV+1)
    static constexpr int KQ = KP > 4 ? KP - 4 : 0;
    // B halo members before the output (>= 2^KQ - 1 rows of garbage reach; a
    // multiple of 4 so layout-B reads are whole 16-byte chunks)
    static constexpr int LEFT = KP > 4 ? ((1 << KQ) > 4 ? (1 << KQ) : 4) : 0;
    static constexpr int NBMAX = KP > 4 ? (AV + 1 - LEFT - (1 << KQ)) / 16 : 0;
    // B blocks stored; with 512 threads rounded so a residue's positions per tile
    // (NB * 256 / 2^KP) stay a 16-byte multiple (TMA store rows)
    static constexpr int NBQ = (KP >= 8 ? 4 : KP == 7 ? 2 : 1);
    static constexpr int NB = ((NT == 512 || TDS_SPLIT_NBQ_ALL) && !TDS_SPLIT_STG) ? NBMAX - NBMAX % NBQ : NBMAX;
    static constexpr int TV = KP > 4 ? NB * 16 * R : AV * R;              // output rows per tile
    static constexpr int HEAD = R + LEFT * R;                             // window rows before the tile
    static_assert(TV % (1 << KP) == 0, "tile must hold whole residue periods");
    // TMA view: the tensor starts TOFF rows into each slot so that every
    // window starts on a 128-byte line (then the 8 lanes of a quarter-warp read
    // 4 whole swizzled lines: no bank conflict); rows [0, TOFF) come by LDG.
    template <typename T>
    __host__ __device__ static constexpr int toff() {
        return (128 / int(sizeof(T)) - HEAD % (128 / int(sizeof(T)))) % (128 / int(sizeof(T)));
    }
    template <typename T>
    __host__ __device__ static constexpr int box_lines() { return ROWS / (128 / int(sizeof(T))); }
    template <typename T>
    __host__ __device__ static constexpr int stage_elems() { return (box_lines<T>() * 128 + 1023) / 1024 * 1024 / int(sizeof(T)); }
    // output staging for the TMA tensor store: [array][residue][position], PT
    // positions per residue per tile (rows of PT * sizeof(T) bytes, a 16-byte multiple)
    static constexpr int PT = TV >> KP;
    static constexpr int BOXP = PT <= 256 ? PT : 240;  // TMA box dims are <= 256: KP <= 3 stores PT / 240 boxes
    static constexpr int NBOX = PT / BOXP;
    static_assert(PT % BOXP == 0, "whole boxes");
    template <typename T>
    __host__ __device__ static constexpr bool tstore() { return !TDS_SPLIT_STG && (PT * int(sizeof(T))) % 16 == 0; }
    template <typename T>
    __host__ __device__ static constexpr bool tr34() {
        return TDS_SPLIT_TR34 && KP > 4 && ((sizeof(T) == 4 && NT == 512) || (sizeof(T) == 8 && NT == 256));
    }
    template <typename T>
    __host__ __device__ static constexpr bool wstore() {
        return TDS_SPLIT_WSTORE && tr34<T>() && sizeof(T) == 4 && tstore<T>() && NBOX == 1;
    }
    template <typename T>
    __host__ __device__ static constexpr int tbuf_elems() {
        const int tr = !(KP > 4)  ? 0
                       : tr34<T>() ? 3 * 16 * Tr34<T>::C + Tr34<T>::SLACK
                                   : ((sizeof(T) == 4 || TDS_SPLIT_TRC64) ? 3 : 1) * AV * 16;
        const int so = tstore<T>() ? 3 * TV : 0;
        return tr > so ? tr : so;
    }
    // the transpose / staging buffer follows the last array's window (the stages are
    // 1024-byte aligned for the swizzled TMA boxes; the buffer only needs 128 bytes)
    template <typename T>
    __host__ __device__ static constexpr int tbuf_off(int na) {
        return tr34<T>() ? (na - 1) * stage_elems<T>() + ROWS : na * stage_elems<T>();
    }
    template <typename T>
    static constexpr size_t smem_bytes(bool raw) {
        return 1024 + (size_t(tbuf_off<T>(raw ? 4 : 3)) + size_t(tbuf_elems<T>())) * sizeof(T);
    }
};

template <typename T, int KP, bool RAW, int NT, bool SC>
__global__ void __launch_bounds__(NT, (sizeof(T) == 4 && NT == 256) ? 2 : 1)
    split_pipe_kernel(const SplitArgs<T> A, int64_t tps, int64_t nitems, const __grid_constant__ TmapSet tm,
                      int32_t tma_lines, const __grid_constant__ TmapSet tmo, const CUtensorMap *__restrict__ tms) {
    using S = SplitShape<KP, NT>;
    constexpr int R = S::R, AV = S::AV, TV = S::TV, HEAD = S::HEAD, ROWS = S::ROWS, CH = S::CH;
    constexpr int TOFF = S::template toff<T>(), BL = S::template box_lines<T>(), ELINE = 128 / int(sizeof(T));
    static_assert(ROWS % ELINE == 0, "window of whole lines");
    constexpr int STG = S::template stage_elems<T>();          // elements per array stage (1024-byte multiple)
    constexpr int NA = RAW ? 4 : 3;                            // arrays streamed
    constexpr int NTR = KP > 4 ? ((sizeof(T) == 4 || TDS_SPLIT_TRC64) ? 3 : 1) : 0;  // arrays per transpose round
    extern __shared__ __align__(1024) unsigned char smem_raw[];
    T *stage = reinterpret_cast<T *>(smem_raw + ((1024u - (smem_u32(smem_raw) & 1023u)) & 1023u));  // 1024-aligned
    T *tbuf = stage + S::template tbuf_off<T>(NA);  // [NTR][AV * 16] transpose buffer / [3][TV] output staging
    static_assert((ROWS * sizeof(T)) % 128 == 0, "128-byte aligned transpose / staging buffer");
    constexpr bool TSTORE = S::template tstore<T>();
    constexpr bool WST = S::template wstore<T>() && !SC;  // per-warp staging and stores (fp32 512-thread sub-row tiles)
    constexpr int PT = S::PT, BOXP = S::BOXP, NBOX = S::NBOX, NRES = 1 << KP;
    // staging index of (residue rr, tile position p): [box][residue][BOXP]
    auto sidx = [](int rr, int p) { return (p / BOXP) * (NRES * BOXP) + rr * BOXP + p % BOXP; };
    __shared__ __align__(8) uint64_t bar;
    const int t = threadIdx.x, lane = t & 31, warp = t >> 5;
    const int ablk = 30 * warp + lane;  // A-block of this thread
    const int kprev = RAW ? 0 : pass_levels(A.geom.npass, A.geom.kpass);
    const bool small_items = nitems < (int64_t(1) << 31);
    const int64_t tma_end = TOFF + int64_t(tma_lines) * ELINE;  // rows [TOFF, tma_end) of every slot are TMA lines

    auto slot_len = [&](int64_t sigma) -> int64_t {
        if (RAW) return A.n;
        const int64_t r = sigma & ((int64_t(1) << kprev) - 1);
        return r < A.n ? (A.n - r + (int64_t(1) << kprev) - 1) >> kprev : 0;
    };
    // window rows [ws, ws + ROWS); rows [g0, gt) come from the TMA box, the rest by LDG / identity
    auto item_rows = [&](int64_t w, int64_t &sigma, int64_t &t0, int64_t &L, int64_t &g0, int64_t &gt) {
        if (small_items) {
            const uint32_t q = uint32_t(w) / uint32_t(tps);
            sigma = q;
            t0 = int64_t(uint32_t(w) - q * uint32_t(tps)) * TV;
        } else {
            sigma = w / tps;
            t0 = (w % tps) * TV;
        }
        L = slot_len(sigma);
        g0 = t0 - HEAD < TOFF ? TOFF : t0 - HEAD;
        gt = t0 - HEAD + ROWS < tma_end ? t0 - HEAD + ROWS : tma_end;
    };
    auto issue = [&](int64_t w) {  // thread 0 only
        if (w >= nitems || TDS_ABL(2)) return;
        if (tma_lines == 0) {  // slots shorter than one line: everything by LDG
            mbar_expect_tx(&bar, 0);
            return;
        }
        int64_t sigma, t0, L, g0, gt;
        item_rows(w, sigma, t0, L, g0, gt);
        mbar_expect_tx(&bar, NA * BL * 128);
        const int line0 = int((t0 - HEAD - TOFF) / ELINE);  // exact: TV and HEAD + TOFF are whole lines
#pragma unroll
        for (int q = 0; q < NA; ++q) {
            if constexpr ((TDS_L2HINT & 8) != 0)
                tma_load_lines_hint(stage + q * STG, &tm.m[q], line0, int(sigma), &bar, l2_evict_first());
            else
                tma_load_lines(stage + q * STG, &tm.m[q], line0, int(sigma), &bar);
        }
    };
    // the tile's outputs, staged in tbuf as [array][residue][position], leave by one
    // TMA tensor store per array: box {PT positions, 1, 2^KP residues, 1} of the
    // output view {position, r < 2^kprev, rho < 2^KP, system}
    auto tma_store_tile = [&](int64_t sigma, int64_t t0, int kp_prev) {
        fence_proxy_async_smem();  // generic-proxy smem writes -> visible to the TMA
        __syncthreads();
        // fused all-to-all: residues [h q, (h+1) q) of the tile go straight to destination
        // h's residue systems ({position, residue} view, positions shifted by -sc_first;
        // the TMA unit drops the positions past the window).  A TMA tensor STORE with a
        // negative start coordinate is an illegal instruction on sm_100a (measured:
        // scripts/probes/tma_store_probe.cu), so the boxes that start before the window --
        // the first tile's, holding the left halo -- leave by plain stores of the window
        // part (CTA-uniform branch; one tile of each system).
        const int64_t jw = SC ? (t0 >> KP) - A.sc_first : 0;  // window position of the tile's first position
        if (SC && jw < 0) {
            for (int bx = 0; bx < NBOX && jw + int64_t(bx) * BOXP < 0; ++bx)
                for (int e = t; e < 3 * NRES * BOXP; e += S::NT) {
                    const int q = e / (NRES * BOXP), rr = (e / BOXP) % NRES, p = e % BOXP;
                    const int64_t j = jw + int64_t(bx) * BOXP + p;
                    if (j < 0 || j >= A.sc_num) continue;
                    const int h = rr / A.sc_q, rl = rr % A.sc_q;
                    A.sc_dst[q][h][int64_t(rl) * A.sc_stride + j] = tbuf[q * TV + bx * NRES * BOXP + rr * BOXP + p];
                }
        }
        if (SC && t == 0 && !TDS_ABL(4)) {
            // (the [array][destination] maps live in global memory: tds_split_scatter
            // copies them there on the stream before the launch)
#pragma unroll
            for (int q = 0; q < 3; ++q)
#pragma unroll
                for (int bx = 0; bx < NBOX; ++bx)
#pragma unroll
                    for (int h = 0; h < 8; ++h)
                        if (h < A.sc_groups && jw + int64_t(bx) * BOXP >= 0)
                            tma_store_box3(tms + q * 8 + h, tbuf + q * TV + bx * NRES * BOXP + h * A.sc_q * BOXP,
                                           int(jw + int64_t(bx) * BOXP), 0, 0);
            bulk_commit();
        } else if (t == 0 && !TDS_ABL(4)) {
            const int j0 = int(t0 >> KP), r = int(sigma & ((int64_t(1) << kp_prev) - 1)), sys = int(sigma >> kp_prev);
#pragma unroll
            for (int q = 0; q < 3; ++q)
#pragma unroll
                for (int bx = 0; bx < NBOX; ++bx)
                    if constexpr ((TDS_L2HINT & 16) != 0)
                        tma_store_4d_hint(&tmo.m[q], tbuf + q * TV + bx * NRES * BOXP, j0 + bx * BOXP, r, 0, sys,
                                          l2_evict_last());
                    else
                        tma_store_4d(&tmo.m[q], tbuf + q * TV + bx * NRES * BOXP, j0 + bx * BOXP, r, 0, sys);
            bulk_commit();
        }
    };
    pdl_wait();  // the previous kernel on the stream is complete before any global access
    if (t == 0) {
        mbar_init(&bar, 1);
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
        issue(blockIdx.x);
    }
    __syncthreads();

    for (int64_t it = 0;; ++it) {
        const int64_t w = int64_t(blockIdx.x) + it * gridDim.x;
        if (w >= nitems) break;
        pdl_trigger_if_last(w + gridDim.x >= nitems);
        int64_t sigma, t0, L, g0, gt;
        item_rows(w, sigma, t0, L, g0, gt);
        if (!TDS_ABL(2)) mbar_wait(&bar, uint32_t(it & 1));
        const int64_t ws = t0 - HEAD;  // window start row
        if (!TDS_ABL(2) && (ws <= 0 || ws + ROWS >= L || g0 > ws || gt < ws + ROWS)) {
            // CTA-uniform: patch the stage where the window leaves the TMA range --
            // identity rows outside [0, L), the tail rows by LDG, and (first pass)
            // a_0 = c_{n-1} = 0 -- so the register loads below need no branch
            for (int s = t; s < ROWS; s += S::NT) {
                const int64_t row = ws + s;
                const bool ident = row < 0 || row >= L, tail = !ident && (row < g0 || row >= gt);
                if (!(ident || tail || (RAW && (row == 0 || row == L - 1)))) continue;
                const int o = sw_off<T>(s);
                T va = stage[o], vc = stage[STG + o], vd = stage[2 * STG + o], vb = RAW ? stage[3 * STG + o] : T(1);
                if (ident) {
                    va = vc = vd = T(0);
                    vb = T(1);
                } else if (tail) {
                    const int64_t g = sigma * A.in_stride + row;
                    va = A.a[g];
                    vc = A.c[g];
                    vd = A.d[g];
                    if constexpr (RAW) vb = A.b[g];
                }
                if (RAW && row == 0) va = T(0);
                if (RAW && row == L - 1) vc = T(0);
                stage[o] = va;
                stage[STG + o] = vc;
                stage[2 * STG + o] = vd;
                if constexpr (RAW) stage[3 * STG + o] = vb;
            }
            asm volatile("fence.proxy.async.shared::cta;" ::: "memory");  // before the next TMA refill
            __syncthreads();
        }
        const int64_t i0 = ws + int64_t(ablk) * R;  // first row of this thread (layout A)
        T ra[R], rc[R], rd[R];
        lds_rows_sw<T, R>(stage + 0 * STG, ablk * R, ra);
        lds_rows_sw<T, R>(stage + 1 * STG, ablk * R, rc);
        lds_rows_sw<T, R>(stage + 2 * STG, ablk * R, rd);
        if constexpr (RAW) {
            T rb[R];
            lds_rows_sw<T, R>(stage + 3 * STG, ablk * R, rb);
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
        __syncthreads();  // the stage is consumed: prefetch the next tile
        if (t == 0) issue(w + gridDim.x);
        if (!TDS_ABL(1)) {
        if constexpr (KP >= 1) reg_level_w<T, R, 1, 32>(ra, rc, rd);
        if constexpr (KP >= 2) reg_level_w<T, R, 2, 32>(ra, rc, rd);
        if constexpr (KP >= 3) reg_level_w<T, R, 4, 32>(ra, rc, rd);
        if constexpr (KP >= 4) reg_level_w<T, R, 8, 32>(ra, rc, rd);
        }
        if constexpr (TSTORE) {  // tbuf is written next: the previous tile's TMA store must have read it
            if (WST ? lane == 0 : t == 0) bulk_wait_read0();  // WST: each warp's own stores
            __syncthreads();
        }
        if constexpr (KP <= 4) {
            if (A.natural) {  // strided variant: rows stay in original order (no de-interleave)
                if (lane >= 1 && lane <= 30 && i0 < L) {
                    const int64_t o = sigma * A.out_slot + i0;
                    if (i0 + R <= L) {
                        store_run<T, R>(A.oa + o, ra);
                        store_run<T, R>(A.oc + o, rc);
                        store_run<T, R>(A.od + o, rd);
                    } else {
#pragma unroll
                        for (int v = 0; v < R; ++v)
                            if (i0 + v < L) {
                                A.oa[o + v] = ra[v];
                                A.oc[o + v] = rc[v];
                                A.od[o + v] = rd[v];
                            }
                    }
                }
                continue;
            }
        }
        if constexpr (KP <= 4 && TSTORE) {
            constexpr int NR = 1 << KP, G = R >> KP;
            if (lane >= 1 && lane <= 30) {  // residue rr, positions 16(a-1)/2^KP + u
                const int p0 = (16 * (ablk - 1)) >> KP;
#pragma unroll
                for (int rr = 0; rr < NR; ++rr) {
                    T va[G], vc[G], vd[G];
#pragma unroll
                    for (int u = 0; u < G; ++u) {
                        va[u] = ra[rr + NR * u];
                        vc[u] = rc[rr + NR * u];
                        vd[u] = rd[rr + NR * u];
                    }
                    const int o = sidx(rr, p0);  // G | BOXP: a run never crosses a box
                    store_run<T, G>(tbuf + o, va);
                    store_run<T, G>(tbuf + TV + o, vc);
                    store_run<T, G>(tbuf + 2 * TV + o, vd);
                }
            }
            tma_store_tile(sigma, t0, kprev);
        } else if constexpr (KP <= 4) {
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
            const int rho = t / CH, b = t % CH;
            const int mb = LEFT - 16 + 16 * b;  // member of u = 0
            const bool wr = lane >= 1 && lane <= 30;
            if constexpr (S::template tr34<T>()) {  // conflict-free sub-row transpose (fp32 512 / fp64 256 threads)
                constexpr int CW = Tr34<T>::C, AW = 16 * CW;  // class row / array strides
                if (wr) {
                    const int pm = tr34_phys<T>(ablk - 1);
                    trc_write<T, R, CW>(ra, tbuf + pm);
                    trc_write<T, R, CW>(rc, tbuf + AW + pm);
                    trc_write<T, R, CW>(rd, tbuf + 2 * AW + pm);
                }
                __syncthreads();
                const T *rp = tbuf + rho * CW + b - 1;
                tr34_read<R, LEFT>(ra, rp);
                tr34_read<R, LEFT>(rc, rp + AW);
                tr34_read<R, LEFT>(rd, rp + 2 * AW);
            } else if constexpr (NTR == 3 && sizeof(T) == 4) {  // fp32, one round: 3 class-major buffers [rho][m]
                if (wr) {
                    const int pm = trc_phys(ablk - 1);
                    trc_write<T, R, AV>(ra, tbuf + pm);
                    trc_write<T, R, AV>(rc, tbuf + AV * 16 + pm);
                    trc_write<T, R, AV>(rd, tbuf + 2 * AV * 16 + pm);
                }
                __syncthreads();
                int ch[R / 4];
                trc_read_chunks<R, AV>(mb, ch);
                trc_read<R>(ra, tbuf + rho * AV, ch);
                trc_read<R>(rc, tbuf + AV * 16 + rho * AV, ch);
                trc_read<R>(rd, tbuf + 2 * AV * 16 + rho * AV, ch);
            } else if constexpr (NTR == 3) {  // fp64, one round (TDS_SPLIT_TRC64)
                if (wr) {
                    const int pm = trc_phys64(ablk - 1);
                    trc_write<T, R, AV>(ra, tbuf + pm);
                    trc_write<T, R, AV>(rc, tbuf + AV * 16 + pm);
                    trc_write<T, R, AV>(rd, tbuf + 2 * AV * 16 + pm);
                }
                __syncthreads();
                int ch[R / 2];
                trc_read_chunks64<R, AV>(mb, ch);
                trc_read64<R>(ra, tbuf + rho * AV, ch);
                trc_read64<R>(rc, tbuf + AV * 16 + rho * AV, ch);
                trc_read64<R>(rd, tbuf + 2 * AV * 16 + rho * AV, ch);
            } else {
                int ad[R];
                tr_read_addrs<R, AV, (LEFT - 16) & 15>(mb, rho, ad);  // three rounds through one buffer
                if (wr) tr_write<T, R>(ra, tbuf, ablk - 1);
                __syncthreads();
                tr_read<T, R>(ra, tbuf, ad);
                __syncthreads();
                if (wr) tr_write<T, R>(rc, tbuf, ablk - 1);
                __syncthreads();
                tr_read<T, R>(rc, tbuf, ad);
                __syncthreads();
                if (wr) tr_write<T, R>(rd, tbuf, ablk - 1);
                __syncthreads();
                tr_read<T, R>(rd, tbuf, ad);
            }
            if (!TDS_ABL(1)) {
            if constexpr (KQ >= 1) reg_level_w<T, R, 1, CH>(ra, rc, rd);
            if constexpr (KQ >= 2) reg_level_w<T, R, 2, CH>(ra, rc, rd);
            if constexpr (KQ >= 3) reg_level_w<T, R, 4, CH>(ra, rc, rd);
            if constexpr (KQ >= 4) reg_level_w<T, R, 8, CH>(ra, rc, rd);
            }
            // member LEFT + 16(b-1) + u is row t0 + 16(16(b-1) + u) + rho
            if constexpr (WST) {
                // this warp's outputs (residues rho + 16 mu, mu < NQ, positions 0..PT) into its
                // own class rows ([mu][PT] from the first 128-byte boundary of row rho: only this
                // warp reads these rows, apart from halo lanes whose values are discarded), then
                // one 5-D tensor store per array by lane 0 -- no CTA barrier
                constexpr int CW = Tr34<T>::C, AW = 16 * CW, PT = S::PT;
                static_assert(NQ * PT + 31 <= CW, "a warp's staging fits its class row");
                T *wb = tbuf + ((rho * CW + 31) & ~31);
                if (b >= 1 && b <= NB) {
#pragma unroll
                    for (int mu = 0; mu < NQ; ++mu) {  // residue rho + 16 mu, positions G(b-1) + q
                        T va[G], vc[G], vd[G];
#pragma unroll
                        for (int q = 0; q < G; ++q) {
                            va[q] = ra[mu + NQ * q];
                            vc[q] = rc[mu + NQ * q];
                            vd[q] = rd[mu + NQ * q];
                        }
                        const int o = mu * PT + G * (b - 1);
                        store_run<T, G>(wb + o, va);
                        store_run<T, G>(wb + AW + o, vc);
                        store_run<T, G>(wb + 2 * AW + o, vd);
                    }
                }
                fence_proxy_async_smem();  // generic-proxy smem writes -> visible to the TMA
                __syncwarp();
                if (lane == 0 && !TDS_ABL(4)) {
                    const int j0 = int(t0 >> KP), r = int(sigma & ((int64_t(1) << kprev) - 1)),
                              sys = int(sigma >> kprev);
#pragma unroll
                    for (int q = 0; q < 3; ++q) tma_store_5d(&tmo.m[q], wb + q * AW, j0, r, rho, 0, sys);
                    bulk_commit();
                }
                continue;
            }
            if constexpr (TSTORE) {
                __syncthreads();  // every layout-B read of tbuf is done: reuse it as the staging buffer
                if (b >= 1 && b <= NB) {
#pragma unroll
                    for (int mu = 0; mu < NQ; ++mu) {  // residue rho + 16 mu, positions G(b-1) + q
                        T va[G], vc[G], vd[G];
#pragma unroll
                        for (int q = 0; q < G; ++q) {
                            va[q] = ra[mu + NQ * q];
                            vc[q] = rc[mu + NQ * q];
                            vd[q] = rd[mu + NQ * q];
                        }
                        const int o = sidx(rho + 16 * mu, G * (b - 1));
                        store_run<T, G>(tbuf + o, va);
                        store_run<T, G>(tbuf + TV + o, vc);
                        store_run<T, G>(tbuf + 2 * TV + o, vd);
                    }
                }
                tma_store_tile(sigma, t0, kprev);
                continue;
            }
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
    if constexpr (TSTORE) {
        if (WST ? lane == 0 : t == 0) bulk_wait_all();
    }
}

template <typename T, int KP, bool RAW, int NT>
static cudaError_t launch_sp(const SplitArgs<T> &A, int64_t m_in, int64_t max_len, cudaStream_t st,
                             const ScatterHost *sc) {
    using S = SplitShape<KP, NT>;
    // the fused split + all-to-all is its own instantiation (first pass only): the product
    // kernels keep their code and registers
    auto kern = (RAW && sc) ? split_pipe_kernel<T, KP, RAW, NT, RAW> : split_pipe_kernel<T, KP, RAW, NT, false>;
    const size_t smem = S::template smem_bytes<T>(RAW);
    int occ = 1;
    cudaError_t e = kernel_setup((const void *)kern, S::NT, smem, 1, &occ);
    if (e != cudaSuccess) return e;
    const int64_t tps = (max_len + S::TV - 1) / S::TV;
    const int64_t nitems = m_in * tps;
    if (nitems <= 0) return cudaSuccess;
    // every input slot holds at least n >> kprev rows: that many full lines go by TMA
    const int kprev = RAW ? 0 : [&] {
        int k = 0;
        for (int p = 0; p < A.geom.npass; ++p) k += A.geom.kpass[p];
        return k;
    }();
    constexpr int TOFF = S::template toff<T>();
    const int64_t lmin = A.n >> kprev;
    const int64_t tma_lines = lmin > TOFF ? (lmin - TOFF) / (128 / int64_t(sizeof(T))) : 0;
    if (tma_lines > 0x7fffffffLL || m_in > 0x7fffffffLL) return cudaErrorInvalidConfiguration;
    TmapSet tm{};
    if (tma_lines > 0) {
        const T *arrs[4] = {A.a, A.c, A.d, A.b};
        for (int q = 0; q < (RAW ? 4 : 3); ++q)
            if (!encode_rows_tmap(&tm.m[q], arrs[q] + TOFF, int(sizeof(T)), tma_lines, m_in, A.in_stride,
                                  S::template box_lines<T>()))
                return cudaErrorInvalidValue;
    }
    TmapSet tmo{};
    TmapSet24 tms{};
    SplitArgs<T> B = A;
    B.sc_groups = 0;
    if (sc) {  // fused split + all-to-all: one {position, residue} view per destination and array
        if constexpr (!S::template tstore<T>() || !RAW) {
            return cudaErrorNotSupported;
        } else {
            if (sc->groups < 1 || sc->groups > 8 || sc->q * sc->groups != (1 << KP) || m_in != 1)
                return cudaErrorInvalidValue;
            for (int q = 0; q < 3; ++q)
                for (int h = 0; h < sc->groups; ++h) {
                    const uint64_t dims[3] = {uint64_t(sc->num_pos), uint64_t(sc->q), 1};
                    const uint64_t strides[2] = {uint64_t(sc->dst_stride) * sizeof(T),
                                                 uint64_t(sc->dst_stride) * sizeof(T) * uint64_t(sc->q)};
                    const uint32_t box[3] = {uint32_t(S::BOXP), uint32_t(sc->q), 1};
                    if (!encode_box3_tmap_plain(&tms.m[q * 8 + h], sc->dst[q][h], int(sizeof(T)), dims, strides,
                                                box))
                        return cudaErrorInvalidValue;
                }
            B.sc_groups = sc->groups;
            B.sc_q = sc->q;
            B.sc_first = sc->first_pos;
            B.sc_num = sc->num_pos;
            B.sc_stride = sc->dst_stride;
            for (int q = 0; q < 3; ++q)
                for (int h = 0; h < sc->groups; ++h) B.sc_dst[q][h] = static_cast<T *>(sc->dst[q][h]);
        }
    } else if constexpr (S::template tstore<T>()) {  // output view {position, r, rho, system}
        T *outs[3] = {A.oa, A.oc, A.od};
        const int64_t msys = m_in >> kprev;
        for (int q = 0; q < 3; ++q) {
            const bool ok = S::template wstore<T>()  // {position, r, rho mod 16, rho / 16, system}: one warp's box
                                ? encode_out5_tmap(&tmo.m[q], outs[q], int(sizeof(T)), A.out_slot, int64_t(1) << kprev,
                                                   int64_t(1) << KP, msys, S::BOXP)
                                : encode_out_tmap(&tmo.m[q], outs[q], int(sizeof(T)), A.out_slot, int64_t(1) << kprev,
                                                  int64_t(1) << KP, msys, S::BOXP);
            if (!ok) return cudaErrorInvalidValue;
        }
    }
    const int64_t grid = std::min<int64_t>(nitems, int64_t(std::max(occ, 1)) * sm_count_current());
#ifdef TDS_SPLIT_ABLATION
    {
        const char *ab = std::getenv("TDS_SPLIT_ABLATION");
        const int v = ab ? std::atoi(ab) : 0;
        cudaMemcpyToSymbolAsync(tds_split_ablation, &v, sizeof(int), 0, cudaMemcpyHostToDevice, st);
    }
#endif
    // scatter maps: to global memory, stream-ordered (allocated and freed around the launch)
    CUtensorMap *dmaps = nullptr;
    if (B.sc_groups > 0) {
        cudaError_t e2 = cudaMallocAsync(reinterpret_cast<void **>(&dmaps), sizeof(tms), st);
        if (e2 == cudaSuccess) e2 = cudaMemcpyAsync(dmaps, &tms, sizeof(tms), cudaMemcpyHostToDevice, st);
        if (e2 != cudaSuccess) return e2;
    }
    cudaError_t le = launch_pdl(kern, dim3(unsigned(grid)), dim3(S::NT), smem, st, 1, B, tps, nitems, tm,
                                int32_t(tma_lines), tmo, (const CUtensorMap *)dmaps);
    if (dmaps) {
        const cudaError_t e3 = cudaFreeAsync(dmaps, st);
        if (le == cudaSuccess) le = e3;
    }
    if (le != cudaSuccess) return le;
    return cudaGetLastError();
}

template <typename T>
cudaError_t launch_split_pipe(const SplitArgs<T> &A, bool raw, int64_t m_in, int64_t max_len, int threads,
                              cudaStream_t st, const ScatterHost *sc) {
    // fp32: 512 threads (1 CTA/SM, 7.7K-row windows, less halo) when split_threads >= 512; fp64 always 256
    constexpr int NTW = sizeof(T) == 4 ? 512 : 256;
    const bool wide = threads >= 512;
#define TDS_SP(KPV)                                                                                       \
    case KPV:                                                                                             \
        if (wide)                                                                                         \
            return raw ? launch_sp<T, KPV, true, NTW>(A, m_in, max_len, st, sc)                           \
                       : launch_sp<T, KPV, false, NTW>(A, m_in, max_len, st, sc);                         \
        return raw ? launch_sp<T, KPV, true, 256>(A, m_in, max_len, st, sc)                                \
                   : launch_sp<T, KPV, false, 256>(A, m_in, max_len, st, sc)
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

template cudaError_t launch_split_pipe<float>(const SplitArgs<float> &, bool, int64_t, int64_t, int, cudaStream_t,
                                              const ScatterHost *);
template cudaError_t launch_split_pipe<double>(const SplitArgs<double> &, bool, int64_t, int64_t, int, cudaStream_t,
                                               const ScatterHost *);

}  // namespace tds
