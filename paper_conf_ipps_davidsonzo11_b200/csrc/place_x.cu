// place_x.cu -- A4 "x placement": put the per-subsystem solutions back in the
// original row order, x[s][r + 2^K j] = xs[slot(s, r)][j].
//
// PCR splitting leaves 2^K interleaved subsystems (residue classes mod 2^K,
// PAPER.md Fig. 3a); the on-chip kernel writes each subsystem's x
// contiguously into its workspace slot.  Writing x straight to original rows
// from there would be a stride-2^K scatter (one 4-byte sector per element).
// Here thread t gathers 16 CONSECUTIVE original rows (the mirror image of the
// register split kernel's de-interleaved store): for K <= 4 the 16 >> K rows
// of one residue have consecutive j and are one vector load, and across the
// warp every residue run is a coalesced read; the 16 rows leave as contiguous
// 16-byte vector stores.
#include <algorithm>

#include "pipe.cuh"

namespace tds {

template <typename T>
struct PlaceArgs {
    const T *xs;         // per-subsystem solutions, slot sigma at xs[sigma * slot + j]
    T *x;                // output, original layout
    int64_t n, batch_stride, slot;
    int32_t K;           // total split levels
    int32_t vec;         // x rows may be written with 16-byte vector stores
    PassGeom geom;       // slot -> residue map
};

constexpr int kPlaceRows = 16;
constexpr int kPlaceThreads = 256;

template <typename T, int KK>  // KK = min(K, 4)
__global__ void __launch_bounds__(kPlaceThreads) place_x_kernel(const PlaceArgs<T> A) {
    constexpr int R = kPlaceRows;
    constexpr int NRK = 1 << KK;  // residues among 16 consecutive rows
    constexpr int G = R >> KK;    // rows per residue per thread
    constexpr int W = 16 / int(sizeof(T));
    const int64_t NR = int64_t(1) << A.K;
    const int64_t tiles = (A.n + R * kPlaceThreads - 1) / (R * kPlaceThreads);
    const int64_t sys = blockIdx.x / tiles;
    const int64_t i0 = ((blockIdx.x % tiles) * kPlaceThreads + threadIdx.x) * R;
    if (i0 >= A.n) return;
    const int64_t sys_slots = sys << A.K;
    const bool full = i0 + R <= A.n;
    T v[R];
#pragma unroll
    for (int rho = 0; rho < NRK; ++rho) {
        const int64_t row = i0 + rho;           // first of this residue's G rows
        const int64_t r = row & (NR - 1), j = row >> A.K;
        const T *src = A.xs + (sys_slots + r) * A.slot + j;  // slots are in canonical residue order
        constexpr bool kVec = (G * sizeof(T) >= 16) || (sizeof(T) == 4 && G == 2);
        if (kVec && full) {
            if constexpr (G * sizeof(T) >= 16) {
#pragma unroll
                for (int q = 0; q < G / W; ++q) {
                    if constexpr (sizeof(T) == 4) {
                        const float4 f = __ldcs(reinterpret_cast<const float4 *>(src) + q);
                        v[rho + NRK * (4 * q)] = f.x;
                        v[rho + NRK * (4 * q + 1)] = f.y;
                        v[rho + NRK * (4 * q + 2)] = f.z;
                        v[rho + NRK * (4 * q + 3)] = f.w;
                    } else {
                        const double2 f = __ldcs(reinterpret_cast<const double2 *>(src) + q);
                        v[rho + NRK * (2 * q)] = f.x;
                        v[rho + NRK * (2 * q + 1)] = f.y;
                    }
                }
            } else if constexpr (sizeof(T) == 4 && G == 2) {
                const float2 f = __ldcs(reinterpret_cast<const float2 *>(src));
                v[rho] = f.x;
                v[rho + NRK] = f.y;
            }
        } else {
#pragma unroll
            for (int u = 0; u < G; ++u)
                v[rho + NRK * u] = (row + NRK * u < A.n) ? __ldcs(src + u) : T(0);
        }
    }
    T *dst = A.x + sys * A.batch_stride + i0;
    if (full && A.vec) {
#pragma unroll
        for (int q = 0; q < R / W; ++q) {
            if constexpr (sizeof(T) == 4)
                __stcs(reinterpret_cast<float4 *>(dst) + q, make_float4(v[4 * q], v[4 * q + 1], v[4 * q + 2], v[4 * q + 3]));
            else
                __stcs(reinterpret_cast<double2 *>(dst) + q, make_double2(v[2 * q], v[2 * q + 1]));
        }
    } else {
#pragma unroll
        for (int u = 0; u < R; ++u)
            if (i0 + u < A.n) dst[u] = v[u];
    }
}

// K >= 5: 32 residues x 128 positions per CTA through a shared-memory tile.
// Reads are 32 runs of 128 consecutive positions (one per slot, 16-byte
// vectors), writes are 128 runs of 32 consecutive original rows; the padded
// tile (stride 33) keeps both shared-memory sides at most 2-way conflicted.
constexpr int kTileRes = 32, kTileJ = 128;

template <typename T>
__global__ void __launch_bounds__(kPlaceThreads) place_x_tile_kernel(const PlaceArgs<T> A, int64_t jtiles,
                                                                    int64_t lmax) {
    constexpr int E = 16 / int(sizeof(T));                 // elements per 16-byte vector
    constexpr int NRD = kTileRes * kTileJ / E / kPlaceThreads;  // vector reads per thread
    constexpr int LPR = kTileJ / E;                        // lanes per residue run (read side)
    constexpr int LPW = kTileRes / E;                      // lanes per row run (write side)
    __shared__ T tile[kTileJ][kTileRes + 1];
    const int t = threadIdx.x;
    const uint32_t rtiles = uint32_t((int64_t(1) << A.K) / kTileRes);
    uint32_t b = blockIdx.x;  // grid < 2^31: 32-bit index arithmetic
    const uint32_t jt = b % uint32_t(jtiles);
    b /= uint32_t(jtiles);
    const int64_t rt = b % rtiles, sys = b / rtiles;
    const int64_t j0 = jt * kTileJ, r0 = rt * kTileRes;
    const T *src = A.xs + ((sys << A.K) + r0) * A.slot + j0;
#pragma unroll
    for (int q = 0; q < NRD; ++q) {
        const int e = q * kPlaceThreads + t;
        const int rl = e / LPR, jj = (e % LPR) * E;
        T v[E];
        if (j0 + jj + E <= A.slot) {
            if constexpr (sizeof(T) == 4) {
                const float4 f = __ldcs(reinterpret_cast<const float4 *>(src + rl * A.slot + jj));
                v[0] = f.x;
                v[1] = f.y;
                v[2] = f.z;
                v[3] = f.w;
            } else {
                const double2 f = __ldcs(reinterpret_cast<const double2 *>(src + rl * A.slot + jj));
                v[0] = f.x;
                v[1] = f.y;
            }
        } else {
#pragma unroll
            for (int u = 0; u < E; ++u) v[u] = j0 + jj + u < A.slot ? src[rl * A.slot + jj + u] : T(0);
        }
#pragma unroll
        for (int u = 0; u < E; ++u) tile[jj + u][rl] = v[u];
    }
    __syncthreads();
    T *dst = A.x + sys * A.batch_stride + r0;
#pragma unroll
    for (int q = 0; q < NRD; ++q) {
        const int e = q * kPlaceThreads + t;
        const int jj = e / LPW, rl = (e % LPW) * E;
        const int64_t j = j0 + jj;
        if (j >= lmax) continue;
        const int64_t row = (j << A.K) + r0 + rl;  // original row of residue r0 + rl
        T v[E];
#pragma unroll
        for (int u = 0; u < E; ++u) v[u] = tile[jj][rl + u];
        T *p = dst + (j << A.K) + rl;
        if (A.vec && row + E <= A.n) {
            if constexpr (sizeof(T) == 4)
                __stcs(reinterpret_cast<float4 *>(p), make_float4(v[0], v[1], v[2], v[3]));
            else
                __stcs(reinterpret_cast<double2 *>(p), make_double2(v[0], v[1]));
        } else {
#pragma unroll
            for (int u = 0; u < E; ++u)
                if (row + u < A.n) p[u] = v[u];
        }
    }
}

// K >= 5 (fp32) / 4 (fp64), 16-byte aligned rows: a persistent TMA transposer.
// A box is E x E elements (E = 128 bytes / sizeof(T)): E positions of E
// consecutive residue slots in (tensor view {positions, slots} of xs), E
// residues of E consecutive j out (view {2^K, floor(n / 2^K), m} of x), both
// with the 128-byte swizzle so the shared-memory transpose (one LDS.128 of a
// slot's chunk, CH scalar STS into the j rows) is conflict-free.  NBX boxes
// along j per tile; loads run two tiles ahead; stores are TMA tensor stores.
// Rows past floor(n / 2^K) * 2^K (fewer than 2^K per system) are copied last
// with plain loads and stores.
// Tile shape of the TMA transposer: 2 boxes per tile, 128 threads (~25 KB, 9 CTAs per
// SM) measured fastest on config 3 (place_x 22.4 -> 20.8 us, gpurun_out/r02b9, r02b10):
// more, smaller CTAs beat deeper pipelines (3-4 input stages or double-buffered
// output boxes: 24-29 us) and 4-box / 256- or 512-thread tiles (22.3-22.8 us).
#ifndef TDS_TP_BOXES
#define TDS_TP_BOXES 2
#endif
#ifndef TDS_TP_THREADS
#define TDS_TP_THREADS 128
#endif
constexpr int kTpBoxes = TDS_TP_BOXES, kTpThreads = TDS_TP_THREADS;
// pipeline depth of the TMA transposer: input stages in flight, output boxes in flight
#ifndef TDS_TP_STAGES
#define TDS_TP_STAGES 2
#endif
#ifndef TDS_TP_OUTBUF
#define TDS_TP_OUTBUF 1
#endif
constexpr int kTpStages = TDS_TP_STAGES, kTpOut = TDS_TP_OUTBUF;

template <typename T, bool XS>
__global__ void __launch_bounds__(kTpThreads) place_x_tma_kernel(const PlaceArgs<T> A, const __grid_constant__ TmapSet tm,
                                                                int64_t ntiles, int64_t jtiles, int64_t lfull,
                                                                int64_t msys, int32_t l2_discard,
                                                                const CUtensorMap *__restrict__ xmaps, int64_t jb) {
    constexpr int E = 128 / int(sizeof(T)), CH = 16 / int(sizeof(T)), NBX = kTpBoxes;
    constexpr int BOX = E * E;  // elements per box
    extern __shared__ __align__(1024) unsigned char smem_raw[];
    T *base = reinterpret_cast<T *>(smem_raw + ((1024u - (smem_u32(smem_raw) & 1023u)) & 1023u));
    constexpr int NS = kTpStages, NO = kTpOut;
    T *sin = base;                    // [NS][NBX][E slots][E positions]
    T *sout0 = base + NS * NBX * BOX;  // [NO][NBX][E j][E residues]
    __shared__ __align__(8) uint64_t full[NS];
    const int t = threadIdx.x;
    const int64_t rtiles = (int64_t(1) << A.K) / E;
    auto coords = [&](int64_t w, int64_t &sys, int64_t &rt, int64_t &jt) {
        jt = w % jtiles;
        const int64_t q = w / jtiles;
        rt = q % rtiles;
        sys = q / rtiles;
    };
    auto issue = [&](int64_t w, int s) {  // thread 0
        if (w >= ntiles) return;
        int64_t sys, rt, jt;
        coords(w, sys, rt, jt);
        mbar_expect_tx(&full[s], NBX * BOX * sizeof(T));
        const int slot0 = int((sys << A.K) + rt * E);
#pragma unroll
        for (int bx = 0; bx < NBX; ++bx)
            if constexpr ((TDS_L2HINT & 4) != 0)
                tma_load_box3_hint(sin + (s * NBX + bx) * BOX, &tm.m[0], int((jt * NBX + bx) * E), slot0, 0, &full[s],
                                   l2_evict_first());
            else
                tma_load_box3(sin + (s * NBX + bx) * BOX, &tm.m[0], int((jt * NBX + bx) * E), slot0, 0, &full[s]);
    };
    pdl_wait();  // the previous kernel on the stream is complete before any global access
    if (t == 0) {
#pragma unroll
        for (int q = 0; q < NS; ++q) mbar_init(&full[q], 1);
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
#pragma unroll
        for (int q = 0; q < NS; ++q) issue(int64_t(blockIdx.x) + q * int64_t(gridDim.x), q);
    }
    __syncthreads();
    for (int64_t it = 0;; ++it) {
        const int64_t w = int64_t(blockIdx.x) + it * gridDim.x;
        if (w >= ntiles) break;
        pdl_trigger_if_last(w + gridDim.x >= ntiles);
        const int s = int(it % NS);
        T *sout = sout0 + int(it % NO) * NBX * BOX;
        mbar_wait(&full[s], uint32_t((it / NS) & 1));
        if (l2_discard && t < NBX * E) {  // the x-slot lines of this tile are dead once in shared memory
            int64_t sys, rt, jt;
            coords(w, sys, rt, jt);
            const int64_t pos = (jt * NBX + t / E) * E;
            if (pos + E <= lfull) l2_discard_line(A.xs + ((sys << A.K) + rt * E + t % E) * A.slot + pos);
        }
        if (t == 0) bulk_wait_read<NO - 1>();  // the stores of tile it - NO have read this sout
        __syncthreads();
        // transpose: task = (box, slot r, chunk jq); LDS.128 of slot r's chunk jq,
        // CH scalar stores into rows j = jq*CH + e of the output box
        for (int task = t; task < NBX * E * 8; task += kTpThreads) {
            const int bx = task / (E * 8), rem = task % (E * 8), r = rem % E, jq = rem / E;
            const T *in = sin + (s * NBX + bx) * BOX + r * E + ((jq ^ (r & 7)) * CH);
            T v[CH];
            if constexpr (sizeof(T) == 4) {
                const float4 f = *reinterpret_cast<const float4 *>(in);
                v[0] = f.x;
                v[1] = f.y;
                v[2] = f.z;
                v[3] = f.w;
            } else {
                const double2 f = *reinterpret_cast<const double2 *>(in);
                v[0] = f.x;
                v[1] = f.y;
            }
            T *out = sout + bx * BOX;
#pragma unroll
            for (int e = 0; e < CH; ++e) {
                const int j = jq * CH + e;
                out[j * E + (((r / CH) ^ (j & 7)) * CH) + r % CH] = v[e];
            }
        }
        fence_proxy_async_smem();
        __syncthreads();
        if (t == 0) {
            int64_t sys, rt, jt;
            coords(w, sys, rt, jt);
#pragma unroll
            for (int bx = 0; bx < NBX; ++bx) {
                const int64_t J = (jt * NBX + bx) * E;
                if constexpr (XS) {  // x scatter: the box's rows belong to destination J / jb (boxes never straddle)
                    const int64_t h = J / jb;
                    if (J < lfull) tma_store_box3(xmaps + h, sout + bx * BOX, int(rt * E), int(J - h * jb), int(sys));
                } else {
                    tma_store_box3(&tm.m[1], sout + bx * BOX, int(rt * E), int(J), int(sys));
                }
            }
            bulk_commit();
            issue(w + NS * int64_t(gridDim.x), s);  // stage s is free: every thread passed the barrier
        }
    }
    if (t == 0) bulk_wait_all();
    // rows [lfull * 2^K, n) of every system (fewer than 2^K): position lfull of slot r
    const int64_t tail = A.n - (lfull << A.K);
    for (int64_t idx = int64_t(blockIdx.x) * kTpThreads + t; idx < msys * tail;
         idx += int64_t(gridDim.x) * kTpThreads) {
        const int64_t sys = idx / tail, r = idx % tail;
        A.x[sys * A.batch_stride + (lfull << A.K) + r] = A.xs[((sys << A.K) + r) * A.slot + lfull];
    }
}

template <typename T>
cudaError_t launch_place_x(const T *xs, T *x, int64_t n, int64_t m, int64_t batch_stride, int64_t slot, int K,
                           int vec, const PassGeom &geom, cudaStream_t st, bool xs_scratch, const XScatterHost *xsc) {
    PlaceArgs<T> A{};
    A.xs = xs;
    A.x = x;
    A.n = n;
    A.batch_stride = batch_stride;
    A.slot = slot;
    A.K = K;
    A.vec = vec;
    A.geom = geom;
    constexpr int E = 128 / int(sizeof(T));
    const int64_t lfull = n >> K;  // whole j rows of 2^K residues
    if (xsc) {  // x scatter: only the TMA transposer, whole j rows, boxes inside one destination
        const int64_t jb = xsc->rows_per_group >> K;
        if (!((int64_t(1) << K) >= E && (lfull << K) == n && xsc->rows_per_group % (int64_t(1) << K) == 0 &&
              jb % (kTpBoxes * E) == 0 && jb * xsc->groups == lfull && (m << K) < (int64_t(1) << 31)))
            return cudaErrorNotSupported;
        TmapSet tm{};
        TmapSet24 xm{};
        const uint64_t din[3] = {uint64_t(slot), uint64_t(m << K), 1};
        const uint64_t sin_[2] = {uint64_t(slot) * sizeof(T), uint64_t(slot) * sizeof(T) * uint64_t(m << K)};
        const uint32_t bin[3] = {uint32_t(E), uint32_t(E), 1};
        if (!encode_box3_tmap(&tm.m[0], xs, int(sizeof(T)), din, sin_, bin)) return cudaErrorInvalidValue;
        for (int h = 0; h < xsc->groups; ++h) {  // destination h: {2^K residues, jb j, m systems}
            const uint64_t dout[3] = {uint64_t(1) << K, uint64_t(jb), uint64_t(m)};
            const uint64_t sout_[2] = {(uint64_t(1) << K) * sizeof(T), uint64_t(xsc->dst_system_stride) * sizeof(T)};
            const uint32_t bout[3] = {uint32_t(E), uint32_t(E), 1};
            if (!encode_box3_tmap(&xm.m[h], xsc->dst[h], int(sizeof(T)), dout, sout_, bout)) return cudaErrorInvalidValue;
        }
        const int64_t rtiles = (int64_t(1) << K) / E;
        const int64_t jtiles = lfull / (kTpBoxes * E);
        const int64_t ntiles = m * rtiles * jtiles;
        const size_t smem = 1024 + size_t((kTpStages + kTpOut) * kTpBoxes * E * E) * sizeof(T);
        auto kern = place_x_tma_kernel<T, true>;
        int occ = 1;
        cudaError_t e = kernel_setup((const void *)kern, kTpThreads, smem, 1, &occ);
        if (e != cudaSuccess) return e;
        CUtensorMap *dmaps = nullptr;  // the destination maps in global memory, stream-ordered
        e = cudaMallocAsync(reinterpret_cast<void **>(&dmaps), sizeof(xm), st);
        if (e == cudaSuccess) e = cudaMemcpyAsync(dmaps, &xm, sizeof(xm), cudaMemcpyHostToDevice, st);
        if (e != cudaSuccess) return e;
        const int64_t grid =
            std::max<int64_t>(1, std::min<int64_t>(ntiles, int64_t(std::max(occ, 1)) * sm_count_current()));
        const int32_t disc = xs_scratch && (slot * int64_t(sizeof(T))) % 128 == 0 && uintptr_t(xs) % 128 == 0;
        e = launch_pdl(kern, dim3(unsigned(grid)), dim3(kTpThreads), smem, st, 1, A, tm, ntiles, jtiles, lfull, m, disc,
                       (const CUtensorMap *)dmaps, jb);
        const cudaError_t e3 = cudaFreeAsync(dmaps, st);
        if (e != cudaSuccess) return e;
        if (e3 != cudaSuccess) return e3;
        return cudaGetLastError();
    }
    if ((int64_t(1) << K) >= E && vec && lfull > 0 && n > 0 && m > 0) {
        const int64_t rtiles = (int64_t(1) << K) / E;
        const int64_t jtiles = (lfull + kTpBoxes * E - 1) / (kTpBoxes * E);
        const int64_t ntiles = m * rtiles * jtiles;
        TmapSet tm{};
        // xs: {positions, slots, 1}, box {E positions, E slots, 1}
        const uint64_t din[3] = {uint64_t(slot), uint64_t(m << K), 1};
        const uint64_t sin_[2] = {uint64_t(slot) * sizeof(T), uint64_t(slot) * sizeof(T) * uint64_t(m << K)};
        const uint32_t bin[3] = {uint32_t(E), uint32_t(E), 1};
        // x: {2^K residues, lfull j, m systems}, box {E residues, E j, 1}
        const uint64_t dout[3] = {uint64_t(1) << K, uint64_t(lfull), uint64_t(m)};
        const uint64_t sout_[2] = {(uint64_t(1) << K) * sizeof(T), uint64_t(batch_stride) * sizeof(T)};
        const uint32_t bout[3] = {uint32_t(E), uint32_t(E), 1};
        if ((m << K) < (int64_t(1) << 31) &&
            encode_box3_tmap(&tm.m[0], xs, int(sizeof(T)), din, sin_, bin) &&
            encode_box3_tmap(&tm.m[1], x, int(sizeof(T)), dout, sout_, bout)) {
            const size_t smem = 1024 + size_t((kTpStages + kTpOut) * kTpBoxes * E * E) * sizeof(T);
            auto kern = place_x_tma_kernel<T, false>;
            int occ = 1;
            cudaError_t e = kernel_setup((const void *)kern, kTpThreads, smem, 1, &occ);
            if (e != cudaSuccess) return e;
            const int64_t grid =
                std::max<int64_t>(1, std::min<int64_t>(ntiles, int64_t(std::max(occ, 1)) * sm_count_current()));
            // x slots are scratch whose last reader is this kernel: drop their lines from L2 once loaded
            const int32_t disc = xs_scratch && (slot * int64_t(sizeof(T))) % 128 == 0 && uintptr_t(xs) % 128 == 0;
            e = launch_pdl(kern, dim3(unsigned(grid)), dim3(kTpThreads), smem, st, 1, A, tm, ntiles, jtiles, lfull, m,
                           disc, (const CUtensorMap *)nullptr, int64_t(0));
            if (e != cudaSuccess) return e;
            return cudaGetLastError();
        }
    }
    if (K >= 5) {
        const int64_t lmax = (n + (int64_t(1) << K) - 1) >> K;
        const int64_t jtiles = (lmax + kTileJ - 1) / kTileJ;
        const int64_t grid = m * ((int64_t(1) << K) / kTileRes) * jtiles;
        if (grid > 0x7fffffffLL) return cudaErrorInvalidConfiguration;
        place_x_tile_kernel<T><<<(unsigned)grid, kPlaceThreads, 0, st>>>(A, jtiles, lmax);
        return cudaGetLastError();
    }
    const int64_t tiles = (n + kPlaceRows * kPlaceThreads - 1) / (kPlaceRows * kPlaceThreads);
    const int64_t grid = m * tiles;
    if (grid > 0x7fffffffLL) return cudaErrorInvalidConfiguration;
    switch (K >= 4 ? 4 : K) {
        case 1: place_x_kernel<T, 1><<<(unsigned)grid, kPlaceThreads, 0, st>>>(A); break;
        case 2: place_x_kernel<T, 2><<<(unsigned)grid, kPlaceThreads, 0, st>>>(A); break;
        case 3: place_x_kernel<T, 3><<<(unsigned)grid, kPlaceThreads, 0, st>>>(A); break;
        default: place_x_kernel<T, 4><<<(unsigned)grid, kPlaceThreads, 0, st>>>(A); break;
    }
    return cudaGetLastError();
}

template cudaError_t launch_place_x<float>(const float *, float *, int64_t, int64_t, int64_t, int64_t, int, int,
                                           const PassGeom &, cudaStream_t, bool, const XScatterHost *);
template cudaError_t launch_place_x<double>(const double *, double *, int64_t, int64_t, int64_t, int64_t, int, int,
                                            const PassGeom &, cudaStream_t, bool, const XScatterHost *);

}  // namespace tds
