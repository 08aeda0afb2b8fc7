// common.cuh -- device helpers shared by the libtds kernels (not by the oracle).
#pragma once
#include <cuda_runtime.h>
#include <stdint.h>

#include <algorithm>

#include "tds_internal.h"

namespace tds {

constexpr int kMaxPasses = TDS_MAX_PASSES;

// Mutation-test builds only (scripts/mutation_check.sh, -DTDS_MUTATE=k):
// site k drops one long-range coupling term so the coupling tests
// (tests/test_coupling.py) can be shown to fail.  Product builds: 0, every
// site compiles away.
//   1 warp-form top PCR (onchip_pipe solve_item_warp): warps >= 2 apart
//   2 cpipe: the last warp's chain loses the next CTA's rows (DSMEM hand-off)
//   3 cpipe: the cluster's all-gathered top system, strides >= 4
//   4 pipe shared-memory form: reduced PCR, strides >= 4
//   5 onchip (generic / cluster) leader PCR, strides >= 4
//   6 onchip cluster: the deferred chain loses the next CTA's ghost rows
//   7 onchip_coalesced: PCR levels, strides >= 4
#ifndef TDS_MUTATE
#define TDS_MUTATE 0
#endif
#define TDS_MUT(k, cond) (TDS_MUTATE == (k) && (cond))

// Reciprocal.  fp32: the SFU approximation (MUFU.RCP, <= 1 ulp) -- the
// north_star's fp32 tolerance (1e-4 error, 1e-5 residual) leaves room for it
// (reading R16).  fp64: the SFU seed (MUFU.RCP64H) refined by one
// cubic step (relative error <= 2 ulp, R16, below) instead of IEEE
// division, whose special-case slow path costs a call per row update.
__device__ __forceinline__ float rcp(float x) {
    float r;
    asm("rcp.approx.ftz.f32 %0, %1;" : "=f"(r) : "f"(x));
    return r;
}
// fp64 refinement: with e = 1 - x r0, 1/x = r0 / (1 - e) = r0 (1 + e + e^2
// + ...); r0 (1 + e + e^2) = fma(r0, fma(e, e, e), r0) leaves a relative
// error ~e^3 (seed <= 9.9e-7 ~ 2^-20 -> 2^-60) plus rounding: <= 2 ulp over
// 2^26 inputs, in 3 dependent DFMA instead of the two Newton steps' 4 (0 ulp
// measured; -DTDS_RCP64_CUBIC=0): config 3 fp64 step -3 %
// (scripts/probes/rcp64_probe.cu, profiles/r02am_rcp64.md).
#ifndef TDS_RCP64_CUBIC
#define TDS_RCP64_CUBIC 1
#endif
__device__ __forceinline__ double rcp(double x) {
    double r;
    asm("rcp.approx.ftz.f64 %0, %1;" : "=d"(r) : "d"(x));
#if TDS_RCP64_CUBIC
    const double e = fma(-x, r, 1.0);
    return fma(r, fma(e, e, e), r);
#else
    double e = fma(-x, r, 1.0);
    r = fma(r, e, r);
    e = fma(-x, r, 1.0);
    return fma(r, e, r);
#endif
}

// The same update with the other operation order: the products a_i a_{i-s},
// c_i c_{i+s} and the numerator d_i - a_i d_{i-s} - c_i d_{i+s} do not depend
// on r, so they are formed while the reciprocal is in flight and each output
// is ONE multiply after it (1 dependent op after MUFU.RCP instead of 3).
// Equal in exact arithmetic; measured faster in the k = 0 cluster kernel
// (config 2 -3 %, config 4 -4 %), slower in the k > 0 pipe kernel, neutral in
// the split, so only onchip_cpipe.cu uses it.
template <typename T>
__device__ __forceinline__ void row_update_early(T &a, T &c, T &d, T al, T cl, T dl, T ar, T cr, T dr) {
    const T den = fma(-c, ar, fma(-a, cl, T(1)));
    const T r = rcp(den);
    const T pa = a * al;
    const T pc = c * cr;
    const T num = fma(-c, dr, fma(-a, dl, d));
    a = -pa * r;
    c = -pc * r;
    d = num * r;
}

// One PCR/CR row update in NORMALISED form (every row scaled so b = 1).
// With the textbook update (Hockney & Jesshope [11], cited
// PAPER.md P:L199-200) applied to normalised rows and the result rescaled
// by 1/b':
//   r  = 1 / (1 - a_i c_{i-s} - c_i a_{i+s})
//   a' = -a_i a_{i-s} r,  c' = -c_i c_{i+s} r,  d' = (d_i - a_i d_{i-s} - c_i d_{i+s}) r
// Identity neighbours (outside the system) are (a, c, d) = (0, 0, 0).
#ifndef TDS_FP64_EARLY
#define TDS_FP64_EARLY 0
#endif
template <typename T>
__device__ __forceinline__ void row_update(T &a, T &c, T &d, T al, T cl, T dl, T ar, T cr, T dr) {
    if constexpr (TDS_FP64_EARLY && sizeof(T) == 8) {  // experiment: fp64 in the early order (below)
        row_update_early(a, c, d, al, cl, dl, ar, cr, dr);
        return;
    }
    const T den = fma(-c, ar, fma(-a, cl, T(1)));
    const T r = rcp(den);
    const T ma = -a * r;
    const T mc = -c * r;
    const T nd = fma(ma, dl, fma(mc, dr, d * r));
    a = ma * al;
    c = mc * cr;
    d = nd;
}

// The same update on two independent rows at once with the packed fp32x2
// instructions of sm_100 (FFMA2 / FMUL2): per lane bit-identical to
// row_update<float> (same fused operations, same rounding), half the issue slots.
__device__ __forceinline__ float2 neg2(float2 a) { return make_float2(-a.x, -a.y); }
__device__ __forceinline__ void row_update2(float2 &a, float2 &c, float2 &d, float2 al, float2 cl, float2 dl, float2 ar,
                                            float2 cr, float2 dr) {
    const float2 den = __ffma2_rn(neg2(c), ar, __ffma2_rn(neg2(a), cl, make_float2(1.f, 1.f)));
    const float2 r = make_float2(rcp(den.x), rcp(den.y));
    const float2 ma = __fmul2_rn(neg2(a), r);
    const float2 mc = __fmul2_rn(neg2(c), r);
    const float2 nd = __ffma2_rn(ma, dl, __ffma2_rn(mc, dr, __fmul2_rn(d, r)));
    a = __fmul2_rn(ma, al);
    c = __fmul2_rn(mc, cr);
    d = nd;
}

// Workspace slots are kept in CANONICAL residue order: after K cumulative
// levels, slot (s << K) + r holds the residue-r subsystem of system s.  Each
// pass writes the new residue digit rho of input slot sigma (levels kprev
// before it, kp in it) to residue r + (rho << kprev).
__device__ __forceinline__ int64_t out_slot_index(int64_t sigma, int kprev, int kp, int64_t rho) {
    const int64_t sys = sigma >> kprev, r = sigma & ((int64_t(1) << kprev) - 1);
    return (sys << (kprev + kp)) + r + (rho << kprev);
}

__device__ __forceinline__ int pass_levels(int npass, const int32_t *kpass) {
    int k = 0;
#pragma unroll
    for (int p = 0; p < TDS_MAX_PASSES; ++p)
        if (p < npass) k += kpass[p];
    return k;
}

struct PassGeom {
    int32_t npass;                 // passes already applied to the input
    int32_t kpass[kMaxPasses];     // their level counts
};


template <typename T>
struct SplitArgs {
    const T *a, *b, *c, *d;  // input (RAW: original a,b,c,d; else normalised a,c,d slots)
    int64_t in_stride;       // RAW: batch_stride; else input slot capacity
    int64_t n;               // original system size
    T *oa, *oc, *od;         // output slots (normalised)
    int64_t out_slot;        // output slot capacity
    int32_t kp;              // levels fused in this pass
    int32_t tile;            // TILE rows (power of two, >= 2^kp)
    int32_t segs;            // CTAs per input slot
    int32_t ep;              // padded shared-memory length per array
    int32_t vec;             // input rows may be read with 16-byte vector loads
    PassGeom geom;           // passes applied to the input
    int32_t natural;         // output rows in original order (strided variant; first pass, k_p <= 4)
    // fused split + all-to-all (tds_split_scatter): > 0 destinations; residues
    // [h q, (h+1) q) of the tile go to destination h, positions shifted by -sc_first
    int32_t sc_groups, sc_q;
    int64_t sc_first, sc_num, sc_stride;
    T *sc_dst[3][8];  // the destinations again, for the boxes a TMA store cannot take (see split_pipe.cu)
};

// Host description of a scatter (tds_split_scatter): per destination h and
// array t a base pointer; the destination is a [q][dst_stride] block of which
// positions [0, num_pos) of every residue row are written.
struct ScatterHost {
    int32_t groups, q;
    int64_t first_pos, num_pos, dst_stride;
    void *dst[3][8];
};

template <typename T>
struct OnchipArgs {
    const T *a, *b, *c, *d;  // RAW (K == 0): original arrays; else normalised a,c,d slots
    T *x;                    // K == 0: the solution, original layout
    T *xs;                   // K > 0: per-subsystem solutions (workspace slots, aliasing a)
    int64_t n;
    int64_t batch_stride;    // original layout (input when RAW, always for x)
    int64_t slot;            // workspace slot capacity (K > 0)
    int64_t m_systems;       // number of systems (K == 0 persistent kernel)
    int32_t K;               // total split levels
    int32_t log2T;           // PCR levels on the reduced system (T = 2^log2T chains)
    int32_t cluster;         // CTAs per subsystem (thread-block cluster size)
    int32_t tl_levels;       // CR levels across threads before the leader's solve
    int32_t vec;             // 16-byte vector loads/stores allowed
    PassGeom geom;           // passes applied (for the slot -> residue map)
    int32_t l2_discard;      // K > 0: slots are 128-byte aligned, c/d lines may be discarded once loaded
    int32_t x_group;         // K > 0: CTAs (one cluster) storing x of adjacent residue classes together
};

__host__ __device__ constexpr int ilog2c(int v) { return v <= 1 ? 0 : 1 + ilog2c(v / 2); }

template <typename T>
cudaError_t launch_split_pass(const SplitArgs<T> &A, bool raw, int64_t grid, int threads, size_t smem,
                              cudaStream_t st);
template <typename T>
cudaError_t launch_split_reg(const SplitArgs<T> &A, bool raw, int64_t grid, cudaStream_t st);
template <typename T>
cudaError_t launch_split_pipe(const SplitArgs<T> &A, bool raw, int64_t m_in, int64_t max_len, int threads,
                              cudaStream_t st, const ScatterHost *sc = nullptr);
template <typename T>
cudaError_t launch_onchip_pipe(const OnchipArgs<T> &A, int64_t nslots, int threads, int cr_levels, int sm_count,
                               size_t smem, cudaStream_t st);
size_t onchip_pipe_smem_bytes(int32_t dtype, int32_t threads, int32_t R, int32_t tl_levels);

// The persistent TMA-pipelined on-chip kernel applies to split plans (k > 0) on
// one CTA per subsystem whose threads hold 64 bytes of rows per array (fp32
// c = 4, fp64 c = 3; up to 512 threads) or 32 bytes (fp32 c = 3, fp64 c = 2;
// up to 1024 threads).
// in: rows x cols row-major -> out: cols x rows, `narrays` (1 or 4) arrays (interleave.cu)
template <typename T>
cudaError_t launch_transpose(const T *const *in, T *const *out, int narrays, int64_t rows, int64_t cols,
                             cudaStream_t st);

template <typename T>
cudaError_t launch_onchip_strided(const OnchipArgs<T> &A, int64_t nslots, int threads, int64_t ws_stride,
                                  cudaStream_t st);

template <typename T>
cudaError_t launch_onchip_coalesced(T *const wa[2], T *const wc[2], T *const wd[2], T *x, int64_t n, int64_t m,
                                    int64_t batch_stride, int64_t ws_stride, int K, int log2T, int64_t smem_budget,
                                    cudaStream_t st);

template <typename T>
cudaError_t launch_onchip_gpipe(const OnchipArgs<T> &A, int64_t nslots, int threads, int sm_count, cudaStream_t st);

inline bool onchip_pipe_ok(const tds_plan_info &I) {
    const tds_params &P = I.params;
    if (P.k == 0 || P.cluster != 1) return false;
    const int rb = (1 << P.cr_levels) * dsize(I.dtype);
    if (rb != 64 && rb != 32) return false;
    return onchip_pipe_smem_bytes(I.dtype, I.onchip_threads, 1 << P.cr_levels, P.tl_levels) + kSmemReserve + 16 <=
           size_t(232448);
}

template <typename T>
cudaError_t launch_onchip_cpipe(const OnchipArgs<T> &A, int threads, int sm_count, cudaStream_t st);
size_t onchip_cpipe_smem_bytes(int32_t dtype, int32_t threads, int32_t cluster);

// k = 0 systems on chip straight from a, b, c, d: persistent TMA kernel, warp
// form, one CTA or a cluster of 2, 4 or 8 CTAs per system, 64 bytes of rows
// per thread.
inline bool onchip_cpipe_ok(const tds_plan_info &I) {
    const tds_params &P = I.params;
    const int C = P.cluster;
    if (P.k != 0 || (C != 1 && C != 2 && C != 4 && C != 8) || P.tl_levels != 5) return false;
    if ((1 << P.cr_levels) * dsize(I.dtype) != 64) return false;
    const int nw = I.onchip_threads / 32;
    if (I.onchip_threads % 32 || I.onchip_threads > 512) return false;
    if (C * nw > 32 && I.onchip_threads < C * 16) return false;  // CTA 0 solves the C*nw top rows
    return onchip_cpipe_smem_bytes(I.dtype, I.onchip_threads, C) + kSmemReserve + 16 <= size_t(232448);
}

// Host description of an x scatter (tds_solve_normalized_xscatter): rows
// [h rows_per_group, (h+1) rows_per_group) of system s go to
// dst[h] + s * dst_system_stride (+ row - h rows_per_group).
struct XScatterHost {
    int32_t groups;
    int64_t rows_per_group, dst_system_stride;
    void *dst[8];
};

template <typename T>
cudaError_t launch_place_x(const T *xs, T *x, int64_t n, int64_t m, int64_t batch_stride, int64_t slot, int K,
                           int vec, const PassGeom &geom, cudaStream_t st, bool xs_scratch = true,
                           const XScatterHost *xsc = nullptr);
template <typename T>
cudaError_t launch_onchip(const OnchipArgs<T> &A, int cr_levels, bool raw, int64_t grid, int threads,
                          size_t smem, cudaStream_t st);

// G4 seeded input generator (gen.cu), bit-identical to inputs.py's "dd" family.
template <typename T>
cudaError_t launch_generate(T *a, T *b, T *c, T *d, int64_t n, int64_t m, int64_t stride, uint64_t seed,
                            int64_t first_system, double mu, cudaStream_t st);

}  // namespace tds
