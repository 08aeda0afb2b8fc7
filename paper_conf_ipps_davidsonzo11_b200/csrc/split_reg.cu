// split_reg.cu -- G1, register-resident form for k_p <= 4 fused PCR levels.
//
// Same contract as split_pass.cu (one HBM pass of k_p global PCR splitting
// levels, §III-B/C P:L296-303; output de-interleaved so
// each subsystem is contiguous), but with no shared-memory tile:
//   * thread t owns 16 CONSECUTIVE rows in registers (16-byte vector loads);
//   * level l (stride s = 2^l <= 8) needs the last / first s rows of threads
//     t-1 / t+1: warp shuffles, plus shared memory only for the two warp-edge
//     lanes;  the first and last thread of the CTA are the tile's halo
//     (16 >= 2^k_p - 1 rows per side), so a tile yields 16*(NT-2) rows;
//   * after k_p levels row v of the thread belongs to residue v mod 2^k_p and
//     the 16 >> k_p rows of one residue have consecutive positions j, so the
//     de-interleaved store is a vector store per residue, coalesced across
//     the warp (consecutive threads -> consecutive j).
// Per row and level: one normalised row update (9 FMA-pipe ops + 1 MUFU.RCP).
#include "split_reg.cuh"

namespace tds {

template <typename T, int KP, bool RAW>
__global__ void __launch_bounds__(kRegSplitThreads, 2) split_reg_kernel(const SplitArgs<T> A) {
    constexpr int R = kRegSplitRows;
    constexpr int NT = kRegSplitThreads;
    constexpr int NW = NT / 32;
    constexpr int SM = 1 << (KP - 1);  // largest stride
    constexpr int NR = 1 << KP;        // residues produced
    constexpr int G = R >> KP;         // rows per residue per thread
    constexpr int W = 16 / int(sizeof(T));
    __shared__ T eL[2][3][NW][SM];  // lane 0's first s rows  -> previous warp's lane 31
    __shared__ T eR[2][3][NW][SM];  // lane 31's last s rows  -> next warp's lane 0
    const int t = threadIdx.x, lane = t & 31, warp = t >> 5;
    constexpr int TV = NT * R - 2 * R;  // valid rows per tile

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
    const int64_t ntiles = (L + TV - 1) / TV;
    const int64_t t_begin = g * ntiles / A.segs;
    const int64_t t_end = (g + 1) * ntiles / A.segs;

    for (int64_t ti = t_begin; ti < t_end; ++ti) {
        const int64_t i0 = ti * TV - R + int64_t(t) * R;  // first row of this thread
        T ra[R], rc[R], rd[R];
        if (A.vec && i0 >= 0 && i0 + R <= L) {
            const int64_t o = in_base + i0;
#pragma unroll
            for (int q = 0; q < R / W; ++q) {
                if constexpr (sizeof(T) == 4) {
                    const float4 fa = __ldcs(reinterpret_cast<const float4 *>(A.a + o) + q);
                    const float4 fc = __ldcs(reinterpret_cast<const float4 *>(A.c + o) + q);
                    const float4 fd = __ldcs(reinterpret_cast<const float4 *>(A.d + o) + q);
                    ra[4 * q] = fa.x; ra[4 * q + 1] = fa.y; ra[4 * q + 2] = fa.z; ra[4 * q + 3] = fa.w;
                    rc[4 * q] = fc.x; rc[4 * q + 1] = fc.y; rc[4 * q + 2] = fc.z; rc[4 * q + 3] = fc.w;
                    rd[4 * q] = fd.x; rd[4 * q + 1] = fd.y; rd[4 * q + 2] = fd.z; rd[4 * q + 3] = fd.w;
                } else {
                    const double2 fa = __ldcs(reinterpret_cast<const double2 *>(A.a + o) + q);
                    const double2 fc = __ldcs(reinterpret_cast<const double2 *>(A.c + o) + q);
                    const double2 fd = __ldcs(reinterpret_cast<const double2 *>(A.d + o) + q);
                    ra[2 * q] = fa.x; ra[2 * q + 1] = fa.y;
                    rc[2 * q] = fc.x; rc[2 * q + 1] = fc.y;
                    rd[2 * q] = fd.x; rd[2 * q + 1] = fd.y;
                }
            }
            if (RAW) {
                T rb[R];
#pragma unroll
                for (int q = 0; q < R / W; ++q) {
                    if constexpr (sizeof(T) == 4) {
                        const float4 fb = __ldcs(reinterpret_cast<const float4 *>(A.b + o) + q);
                        rb[4 * q] = fb.x; rb[4 * q + 1] = fb.y; rb[4 * q + 2] = fb.z; rb[4 * q + 3] = fb.w;
                    } else {
                        const double2 fb = __ldcs(reinterpret_cast<const double2 *>(A.b + o) + q);
                        rb[2 * q] = fb.x; rb[2 * q + 1] = fb.y;
                    }
                }
#pragma unroll
                for (int v = 0; v < R; ++v) {
                    const T inv = rcp(rb[v]);
                    ra[v] = (i0 + v > 0 ? ra[v] : T(0)) * inv;
                    rc[v] = (i0 + v < L - 1 ? rc[v] : T(0)) * inv;
                    rd[v] = rd[v] * inv;
                }
            }
        } else {
#pragma unroll
            for (int v = 0; v < R; ++v) {
                const int64_t row = i0 + v;
                ra[v] = T(0);
                rc[v] = T(0);
                rd[v] = T(0);
                if (row >= 0 && row < L) {
                    const int64_t o = in_base + row;
                    if (RAW) {
                        const T inv = rcp(A.b[o]);
                        ra[v] = (row > 0 ? A.a[o] : T(0)) * inv;
                        rc[v] = (row < L - 1 ? A.c[o] : T(0)) * inv;
                        rd[v] = A.d[o] * inv;
                    } else {
                        ra[v] = A.a[o];
                        rc[v] = A.c[o];
                        rd[v] = A.d[o];
                    }
                }
            }
        }

        T *el = &eL[0][0][0][0], *er = &eR[0][0][0][0];
        if constexpr (KP >= 1) reg_level<T, R, 1, NW, SM>(ra, rc, rd, el, er, 0, lane, warp);
        if constexpr (KP >= 2) reg_level<T, R, 2, NW, SM>(ra, rc, rd, el, er, 1, lane, warp);
        if constexpr (KP >= 3) reg_level<T, R, 4, NW, SM>(ra, rc, rd, el, er, 0, lane, warp);
        if constexpr (KP >= 4) reg_level<T, R, 8, NW, SM>(ra, rc, rd, el, er, 1, lane, warp);

        // ---- de-interleaved store: residue rho gets rows rho + NR*u, u < G, positions (i0 >> KP) + u
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
        __syncthreads();  // edge buffers are reused by the next tile
    }
}

template <typename T, int KP>
static cudaError_t launch_kp(const SplitArgs<T> &A, bool raw, int64_t grid, cudaStream_t st) {
    if (raw)
        split_reg_kernel<T, KP, true><<<(unsigned)grid, kRegSplitThreads, 0, st>>>(A);
    else
        split_reg_kernel<T, KP, false><<<(unsigned)grid, kRegSplitThreads, 0, st>>>(A);
    return cudaGetLastError();
}

template <typename T>
cudaError_t launch_split_reg(const SplitArgs<T> &A, bool raw, int64_t grid, cudaStream_t st) {
    switch (A.kp) {
        case 1: return launch_kp<T, 1>(A, raw, grid, st);
        case 2: return launch_kp<T, 2>(A, raw, grid, st);
        case 3: return launch_kp<T, 3>(A, raw, grid, st);
        case 4: return launch_kp<T, 4>(A, raw, grid, st);
        default: return cudaErrorInvalidConfiguration;
    }
}

template cudaError_t launch_split_reg<float>(const SplitArgs<float> &, bool, int64_t, cudaStream_t);
template cudaError_t launch_split_reg<double>(const SplitArgs<double> &, bool, int64_t, cudaStream_t);

}  // namespace tds
