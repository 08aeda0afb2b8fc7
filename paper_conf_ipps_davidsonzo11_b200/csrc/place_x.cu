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
#include "common.cuh"

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

template <typename T>
cudaError_t launch_place_x(const T *xs, T *x, int64_t n, int64_t m, int64_t batch_stride, int64_t slot, int K,
                           int vec, const PassGeom &geom, cudaStream_t st) {
    PlaceArgs<T> A{};
    A.xs = xs;
    A.x = x;
    A.n = n;
    A.batch_stride = batch_stride;
    A.slot = slot;
    A.K = K;
    A.vec = vec;
    A.geom = geom;
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
                                           const PassGeom &, cudaStream_t);
template cudaError_t launch_place_x<double>(const double *, double *, int64_t, int64_t, int64_t, int64_t, int, int,
                                            const PassGeom &, cudaStream_t);

}  // namespace tds
