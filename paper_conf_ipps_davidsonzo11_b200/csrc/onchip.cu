// onchip.cu -- G2: the on-chip hybrid CR/PCR-Thomas solver, one subsystem per
// CTA or per thread-block CLUSTER.
//
// Paper: the base kernel is a hybrid PCR-Thomas solver that fetches each
// system into shared memory, splits it with PCR until there are enough
// independent subsystems, then solves each with the Thomas algorithm in one
// thread (§III-A, Fig. 3b; stages 3 and 4, §III-D
// P:L505-512).  The north_star asks for a hybrid CR/PCR solver; Zhang et
// al.'s CR-PCR hybrid is the paper's comparison point.  Stage 1
// (several processors cooperating on one system, §III-C) maps to a
// thread-block cluster on B200: C CTAs on C SMs share one subsystem through
// distributed shared memory, so a subsystem may hold C x the rows one SM can.
//
// B200 form: thread t of cluster-CTA q owns R = 2^c
// CONSECUTIVE rows (q*NT + t)*R ... +R-1 in registers.
//   A.  LDG.128 loads, normalise (b = 1); rows beyond the subsystem are identity;
//   B1. c CR forward levels in registers.  Level l (stride s = 2^(l-1))
//       updates rows v = 2^l-1 (mod 2^l); only row R-1 needs a row of thread
//       t+1 (its row s-1): warp shuffle, shared memory across warps, DSMEM
//       across CTAs -> one reduced row per thread (stride R);
//   B2. c2 more CR levels ACROSS threads in shared memory (stride 2^(l-1)
//       threads), leaving NT / 2^c2 rows per CTA.  The CTA's last row is kept
//       at every level and is the only one that reaches into the next CTA:
//       its chain is deferred until one cluster barrier delivers the values
//       the next CTA published (its rows s-1, which depend on nothing beyond
//       its own first 2s-1 rows);
//   C.  the C * NT / 2^c2 remaining rows are gathered into the leader CTA's
//       shared memory (DSMEM stores); the leader runs log2(T) PCR levels until
//       T independent chains and Thomas on each chain (the paper's stage 3 -> 4
//       switch point T);
//   D.  the x values come back (DSMEM loads), CR back substitution across
//       threads (c2 levels) and then in registers (c levels); x is written to
//       original rows r + 2^K j (index placement A4).
// c = c2 = 0, C = 1 (R = 1) is exactly the paper's PCR-Thomas base kernel.
#include <cooperative_groups.h>

#include "common.cuh"

namespace cg = cooperative_groups;

namespace tds {

// 16-byte streaming loads/stores of N consecutive elements.
template <typename T, int N>
__device__ __forceinline__ void ld16(const T *__restrict__ p, T *v) {
    if constexpr (sizeof(T) == 4) {
#pragma unroll
        for (int q = 0; q < N / 4; ++q) {
            const float4 f = __ldcs(reinterpret_cast<const float4 *>(p) + q);
            v[4 * q] = f.x;
            v[4 * q + 1] = f.y;
            v[4 * q + 2] = f.z;
            v[4 * q + 3] = f.w;
        }
    } else {
#pragma unroll
        for (int q = 0; q < N / 2; ++q) {
            const double2 f = __ldcs(reinterpret_cast<const double2 *>(p) + q);
            v[2 * q] = f.x;
            v[2 * q + 1] = f.y;
        }
    }
}

template <typename T, int N>
__device__ __forceinline__ void st16(T *p, const T *v) {
    if constexpr (sizeof(T) == 4) {
#pragma unroll
        for (int q = 0; q < N / 4; ++q)
            __stcs(reinterpret_cast<float4 *>(p) + q, make_float4(v[4 * q], v[4 * q + 1], v[4 * q + 2], v[4 * q + 3]));
    } else {
#pragma unroll
        for (int q = 0; q < N / 2; ++q)
            __stcs(reinterpret_cast<double2 *>(p) + q, make_double2(v[2 * q], v[2 * q + 1]));
    }
}

// Stage C on the leader CTA: PCR until 2^log2T chains, then Thomas per chain.
// z = [a | c | d] of Z <= ZR * NT normalised rows; x overwrites d.
template <typename T, int ZR>
__device__ __forceinline__ void reduced_solve(T *z, int Z, int NT, int t, int log2T) {
    T *za = z, *zc = z + Z, *zd = z + 2 * Z;
    for (int j = 0; j < log2T; ++j) {
        const int s = 1 << j;
        T na[ZR], nc[ZR], nd[ZR];
#pragma unroll
        for (int q = 0; q < ZR; ++q) {
            const int i = t + q * NT;
            if (i < Z) {
                T a = za[i], c = zc[i], d = zd[i];
                const bool hl = i >= s, hr = i + s < Z && !TDS_MUT(5, s >= 4);
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
        // Thomas on rows ch, ch+TC, ... (b = 1): c'_i = c_i / (1 - a_i c'_{i-1}), ...
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

template <int C>
__device__ __forceinline__ void cluster_or_cta_sync() {
    if constexpr (C > 1) cg::this_cluster().sync(); else __syncthreads();
}

template <typename T, int R, int C, bool RAW>
__global__ void __launch_bounds__(R * sizeof(T) >= 64 ? 512 : 1024) onchip_kernel(const OnchipArgs<T> A) {
    extern __shared__ __align__(16) unsigned char smem_raw[];
    constexpr int CR = ilog2c(R);
    constexpr int W = 16 / int(sizeof(T));  // elements per 16-byte vector
    const int NT = blockDim.x;
    const int t = threadIdx.x, lane = t & 31, warp = t >> 5, nwarps = NT >> 5;
    const int c2 = A.tl_levels;              // CR levels across threads
    const int G = NT >> c2;                  // rows per CTA left for the leader
    const int Z = C * G;                     // leader's reduced system
    T *z = reinterpret_cast<T *>(smem_raw);  // [3][Z] reduced system (leader)
    T *ya = z + 3 * Z;                       // [4][NT] thread-level rows (a, c, d, x)
    T *yc = ya + NT, *yd = yc + NT, *yx = yd + NT;
    T *edge = yx + NT;                       // [2][3][nwarps] warp-edge exchange
    T *ghost = edge + 6 * nwarps;            // [CR][3] register-level rows from the next CTA
    T *tghost = ghost + 3 * 4;               // [c2][3] thread-level rows from the next CTA
    T *xprev = tghost + 3 * 10;              // x of the previous CTA's last row

    const int64_t sigma = blockIdx.x / C;
    const int crank = (C > 1) ? int(blockIdx.x % C) : 0;
    int64_t sys, r, L, in_base;
    if (RAW) {
        sys = sigma;
        r = 0;
        L = A.n;
        in_base = sys * A.batch_stride;
    } else {
        sys = sigma >> A.K;
        r = sigma & ((int64_t(1) << A.K) - 1);
        if (r >= A.n) return;  // empty slot (2^K > n): uniform across the cluster
        L = (A.n - r + (int64_t(1) << A.K) - 1) >> A.K;
        in_base = sigma * A.slot;
    }
    const int64_t out_base = sys * A.batch_stride + r;
    const int64_t jt = int64_t(crank * NT + t) * R;  // first row owned by this thread
    // DSMEM may only be touched once every CTA of the cluster runs: arrive now,
    // wait after the loads are in flight.
    if constexpr (C > 1) cg::this_cluster().barrier_arrive();

    // ---- A. load R consecutive rows, normalise (b = 1)
    T ra[R], rc[R], rd[R];
    if (R >= W && A.vec && jt + R <= L) {
        ld16<T, R>(A.a + in_base + jt, ra);
        ld16<T, R>(A.c + in_base + jt, rc);
        ld16<T, R>(A.d + in_base + jt, rd);
        if (RAW) {
            T rb[R];
            ld16<T, R>(A.b + in_base + jt, rb);
#pragma unroll
            for (int v = 0; v < R; ++v) {
                const T inv = rcp(rb[v]);
                ra[v] = (jt + v > 0 ? ra[v] : T(0)) * inv;
                rc[v] = (jt + v < L - 1 ? rc[v] : T(0)) * inv;
                rd[v] = rd[v] * inv;
            }
        }
    } else {
#pragma unroll
        for (int v = 0; v < R; ++v) {
            const int64_t j = jt + v;
            ra[v] = T(0);
            rc[v] = T(0);
            rd[v] = T(0);
            if (j < L) {
                const int64_t o = in_base + j;
                if (RAW) {
                    const T inv = rcp(A.b[o]);
                    ra[v] = (j > 0 ? A.a[o] : T(0)) * inv;
                    rc[v] = (j < L - 1 ? A.c[o] : T(0)) * inv;
                    rd[v] = A.d[o] * inv;
                } else {
                    ra[v] = A.a[o];
                    rc[v] = A.c[o];
                    rd[v] = A.d[o];
                }
            }
        }
    }

    // ---- B1. CR forward levels in registers
    if constexpr (C > 1) cg::this_cluster().barrier_wait();
    const bool defer = (C > 1) && (t == NT - 1) && (crank < C - 1);
#pragma unroll
    for (int l = 1; l <= CR; ++l) {
        const int s = 1 << (l - 1);
        const T pa = ra[s - 1], pc = rc[s - 1], pd = rd[s - 1];  // row s-1 (level l-1), wanted by thread t-1
        T na = __shfl_down_sync(0xffffffffu, pa, 1);
        T nc = __shfl_down_sync(0xffffffffu, pc, 1);
        T nd = __shfl_down_sync(0xffffffffu, pd, 1);
        T *eb = edge + (l & 1) * 3 * nwarps;
        if (lane == 0) {
            eb[warp] = pa;
            eb[nwarps + warp] = pc;
            eb[2 * nwarps + warp] = pd;
        }
        if constexpr (C > 1) {
            if (t == 0 && crank > 0) {
                T *g = cg::this_cluster().map_shared_rank(ghost, crank - 1);
                g[3 * (l - 1)] = pa;
                g[3 * (l - 1) + 1] = pc;
                g[3 * (l - 1) + 2] = pd;
            }
        }
        __syncthreads();
        if (lane == 31) {
            if (warp + 1 < nwarps) {
                na = eb[warp + 1];
                nc = eb[nwarps + warp + 1];
                nd = eb[2 * nwarps + warp + 1];
            } else {
                na = T(0);
                nc = T(0);
                nd = T(0);
            }
        }
#pragma unroll
        for (int v = (1 << l) - 1; v < R; v += (1 << l)) {
            const bool last = (v == R - 1);  // only row R-1 reaches into thread t+1
            const T ar = last ? na : ra[(v + s) % R];
            const T cr = last ? nc : rc[(v + s) % R];
            const T dr = last ? nd : rd[(v + s) % R];
            if (!(last && defer)) row_update(ra[v], rc[v], rd[v], ra[v - s], rc[v - s], rd[v - s], ar, cr, dr);
        }
    }

    // ---- B2. c2 CR levels across threads (shared memory, in place)
    ya[t] = ra[R - 1];
    yc[t] = rc[R - 1];
    yd[t] = rd[R - 1];
    for (int l = 1; l <= c2; ++l) {
        const int s = 1 << (l - 1);
        __syncthreads();
        if constexpr (C > 1) {
            if (t == s - 1 && crank > 0) {  // row s-1 is final after level l-1: publish for the previous CTA
                T *g = cg::this_cluster().map_shared_rank(tghost, crank - 1);
                g[3 * (l - 1)] = ya[t];
                g[3 * (l - 1) + 1] = yc[t];
                g[3 * (l - 1) + 2] = yd[t];
            }
        }
        if ((t & ((1 << l) - 1)) == (1 << l) - 1 && !(t == NT - 1 && defer)) {
            T a = ya[t], c = yc[t], d = yd[t];
            const bool hr = t + s < NT;  // only t = NT-1 lacks a right neighbour: identity
            row_update(a, c, d, ya[t - s], yc[t - s], yd[t - s], hr ? ya[t + s] : T(0), hr ? yc[t + s] : T(0),
                       hr ? yd[t + s] : T(0));
            ya[t] = a;
            yc[t] = c;
            yd[t] = d;
        }
    }

    // ---- C. deferred chain, gather the remaining rows on the leader, solve there
    T *zl = z;
    if constexpr (C > 1) {
        cg::cluster_group cl = cg::this_cluster();
        cl.sync();  // ghosts from the next CTA are visible (also orders B2's last level)
        if (defer) {
#pragma unroll
            for (int l = 1; l <= CR; ++l) {
                const int s = 1 << (l - 1);
                const bool g = !TDS_MUT(6, crank + 1 < C);
                row_update(ra[R - 1], rc[R - 1], rd[R - 1], ra[R - 1 - s], rc[R - 1 - s], rd[R - 1 - s],
                           g ? ghost[3 * (l - 1)] : T(0), g ? ghost[3 * (l - 1) + 1] : T(0),
                           g ? ghost[3 * (l - 1) + 2] : T(0));
            }
            T a = ra[R - 1], c = rc[R - 1], d = rd[R - 1];
            for (int l = 1; l <= c2; ++l) {
                const int s = 1 << (l - 1);
                row_update(a, c, d, ya[t - s], yc[t - s], yd[t - s], tghost[3 * (l - 1)], tghost[3 * (l - 1) + 1],
                           tghost[3 * (l - 1) + 2]);
            }
            ya[t] = a;
            yc[t] = c;
            yd[t] = d;
        }
        zl = cl.map_shared_rank(z, 0);
    } else {
        __syncthreads();
    }
    const bool top = (t & ((1 << c2) - 1)) == (1 << c2) - 1;  // row kept through all c2 levels
    const int zi = crank * G + (t >> c2);
    if (top) {
        zl[zi] = ya[t];
        zl[Z + zi] = yc[t];
        zl[2 * Z + zi] = yd[t];
    }
    cluster_or_cta_sync<C>();
    if (crank == 0) reduced_solve<T, C>(z, Z, NT, t, A.log2T);
    if constexpr (C > 1) cg::this_cluster().sync();
    if (top) yx[t] = zl[2 * Z + zi];
    if (t == 0) xprev[0] = crank > 0 ? zl[2 * Z + crank * G - 1] : T(0);
    if constexpr (C > 1) cg::this_cluster().barrier_arrive();  // done reading the leader's memory

    // ---- D. back substitution across threads (c2 levels), then in registers
    for (int l = c2; l >= 1; --l) {
        const int s = 1 << (l - 1);
        __syncthreads();
        if ((t & ((1 << l) - 1)) == s - 1) {
            const T xl = t >= s ? yx[t - s] : xprev[0];
            yx[t] = yd[t] - ya[t] * xl - yc[t] * yx[t + s];
        }
    }
    __syncthreads();
    rd[R - 1] = yx[t];
    const T xleft = t > 0 ? yx[t - 1] : xprev[0];
#pragma unroll
    for (int l = CR; l >= 1; --l) {
        const int s = 1 << (l - 1);
#pragma unroll
        for (int v = s - 1; v < R - 1; v += 2 * s) {
            const T xlv = (v >= s) ? rd[(v - s + R) % R] : xleft;
            rd[v] = rd[v] - ra[v] * xlv - rc[v] * rd[(v + s) % R];
        }
    }
    // x of this subsystem is written contiguously: straight to x when K == 0, else
    // to its workspace slot (the placement kernel restores the original order).
    T *dst = A.K == 0 ? A.x + out_base : A.xs + sigma * A.slot;
    const bool dvec = A.K == 0 ? (A.vec != 0) : true;
    if (R >= W && dvec && jt + R <= L) {
        st16<T, R>(dst + jt, rd);
    } else {
#pragma unroll
        for (int v = 0; v < R; ++v) {
            const int64_t j = jt + v;
            if (j < L) __stcs(dst + j, rd[v]);
        }
    }
    if constexpr (C > 1) cg::this_cluster().barrier_wait();  // keep shared memory alive for the readers
}

template <typename T, int R, int C>
static cudaError_t launch_rc(const OnchipArgs<T> &A, bool raw, int64_t grid, int threads, size_t smem,
                             cudaStream_t st) {
    auto kern = raw ? onchip_kernel<T, R, C, true> : onchip_kernel<T, R, C, false>;
    cudaError_t e = cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    if (e != cudaSuccess) return e;
    if constexpr (C > 8) {
        e = cudaFuncSetAttribute(kern, cudaFuncAttributeNonPortableClusterSizeAllowed, 1);
        if (e != cudaSuccess) return e;
    }
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = dim3((unsigned)grid);
    cfg.blockDim = dim3(threads);
    cfg.dynamicSmemBytes = smem;
    cfg.stream = st;
    cudaLaunchAttribute attr[1];
    if constexpr (C > 1) {
        attr[0].id = cudaLaunchAttributeClusterDimension;
        attr[0].val.clusterDim.x = C;
        attr[0].val.clusterDim.y = 1;
        attr[0].val.clusterDim.z = 1;
        cfg.attrs = attr;
        cfg.numAttrs = 1;
    }
    e = cudaLaunchKernelEx(&cfg, kern, A);
    if (e != cudaSuccess) return e;
    return cudaGetLastError();
}

template <typename T, int R>
static cudaError_t launch_r(const OnchipArgs<T> &A, int C, bool raw, int64_t grid, int threads, size_t smem,
                            cudaStream_t st) {
    switch (C) {
        case 1: return launch_rc<T, R, 1>(A, raw, grid, threads, smem, st);
        case 2: if constexpr (R >= 8) return launch_rc<T, R, 2>(A, raw, grid, threads, smem, st); break;
        case 4: if constexpr (R >= 8) return launch_rc<T, R, 4>(A, raw, grid, threads, smem, st); break;
        case 8: if constexpr (R >= 8) return launch_rc<T, R, 8>(A, raw, grid, threads, smem, st); break;
        case 16: if constexpr (R >= 8) return launch_rc<T, R, 16>(A, raw, grid, threads, smem, st); break;
        default: break;
    }
    return cudaErrorInvalidConfiguration;
}

template <typename T>
cudaError_t launch_onchip(const OnchipArgs<T> &A, int cr_levels, bool raw, int64_t grid, int threads,
                          size_t smem, cudaStream_t st) {
    const int C = A.cluster;
    switch (cr_levels) {
        case 0: return C == 1 ? launch_r<T, 1>(A, C, raw, grid, threads, smem, st) : cudaErrorInvalidConfiguration;
        case 1: return C == 1 ? launch_r<T, 2>(A, C, raw, grid, threads, smem, st) : cudaErrorInvalidConfiguration;
        case 2: return C == 1 ? launch_r<T, 4>(A, C, raw, grid, threads, smem, st) : cudaErrorInvalidConfiguration;
        case 3: return launch_r<T, 8>(A, C, raw, grid, threads, smem, st);
        case 4:
            if constexpr (sizeof(T) == 4) return launch_r<T, 16>(A, C, raw, grid, threads, smem, st);
            return cudaErrorInvalidConfiguration;
        default: return cudaErrorInvalidConfiguration;
    }
}

template cudaError_t launch_onchip<float>(const OnchipArgs<float> &, int, bool, int64_t, int, size_t, cudaStream_t);
template cudaError_t launch_onchip<double>(const OnchipArgs<double> &, int, bool, int64_t, int, size_t, cudaStream_t);

}  // namespace tds
