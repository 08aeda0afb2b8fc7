// api.cu -- the solve half of the C ABI: device query, argument validation,
// the stream-ordered launch sequence (split passes, then the on-chip kernel)
// and the diagnostic split-only entry point.  See include/tds.h.
#include <algorithm>
#include <cstring>
#include <string>

#include "common.cuh"
#include "pipe.cuh"

namespace tds {

static bool overlaps(const void *p, size_t pb, const void *q, size_t qb) {
    const char *a = static_cast<const char *>(p), *b = static_cast<const char *>(q);
    return a < b + qb && b < a + pb;
}

static tds_status cuda_fail(cudaError_t e, const char *what) {
    return fail(TDS_ERR_CUDA, std::string(what) + ": " + cudaGetErrorString(e));
}

static tds_status check_device(const tds_plan_st *plan) {
    int dev = -1;
    cudaError_t e = cudaGetDevice(&dev);
    if (e != cudaSuccess) return cuda_fail(e, "cudaGetDevice");
    if (plan->info.device < 0 || dev != plan->info.device)
        return fail(TDS_ERR_DEVICE_MISMATCH, "current device " + std::to_string(dev) + " != plan device " +
                                                 std::to_string(plan->info.device));
    return TDS_OK;
}

static tds_status check_workspace(const tds_plan_info &I, const void *ws, size_t ws_bytes) {
    if (I.workspace_bytes == 0) return TDS_OK;
    if (!ws) return fail(TDS_ERR_WORKSPACE, "workspace is NULL");
    if (ws_bytes < I.workspace_bytes)
        return fail(TDS_ERR_WORKSPACE, "workspace " + std::to_string(ws_bytes) + " < required " +
                                           std::to_string(I.workspace_bytes));
    if (reinterpret_cast<uintptr_t>(ws) % 256) return fail(TDS_ERR_WORKSPACE, "workspace not 256-byte aligned");
    return TDS_OK;
}

// 16-byte vector access to the caller's arrays: every system start must be aligned.
static int vec_ok(const tds_plan_info &I, std::initializer_list<const void *> ptrs) {
    const int64_t es = dsize(I.dtype);
    if ((I.batch_stride * es) % 16) return 0;
    for (const void *p : ptrs)
        if (reinterpret_cast<uintptr_t>(p) % 16) return 0;
    return 1;
}

// Workspace buffer i holds normalised (a, c, d) arrays of E elements each.
template <typename T>
struct WsBufs {
    T *a[2], *c[2], *d[2];
};

template <typename T>
static WsBufs<T> ws_bufs(const tds_plan_info &I, void *ws) {
    WsBufs<T> w{};
    const int nbuf = I.params.passes >= 2 || I.params.strided == 2 ? 2 : 1;
    const int64_t E = int64_t(I.workspace_bytes / (size_t(nbuf) * 3 * sizeof(T)));
    T *base = static_cast<T *>(ws);
    for (int i = 0; i < nbuf; ++i) {
        w.a[i] = base + (3 * i + 0) * E;
        w.c[i] = base + (3 * i + 1) * E;
        w.d[i] = base + (3 * i + 2) * E;
    }
    if (nbuf == 1) {
        w.a[1] = w.a[0];
        w.c[1] = w.c[0];
        w.d[1] = w.d[0];
    }
    return w;
}

// Per-system stride of the in-place (natural order) split output of the
// strided variants: whole 32-byte sectors, so a coalesced group of
// 32 / sizeof(T) residues is one aligned sector (onchip_coalesced.cu).
template <typename T>
static int64_t natural_stride(int64_t n) {
    return round_up(n, 32 / int64_t(sizeof(T)));
}

// Launch the P split passes; returns the index of the buffer holding the result.
template <typename T>
static tds_status run_split(const tds_plan_info &I, const T *a, const T *b, const T *c, const T *d,
                            const WsBufs<T> &w, cudaStream_t st, int *out_buf, int first = 0,
                            int last = 1 << 30, bool natural = false, const ScatterHost *sc = nullptr) {
    const tds_params &P = I.params;
    int kprev = 0;
    for (int p = 0; p < P.passes; ++p) {
        const int kp = P.k_pass[p];
        if (p < first || p > last) {
            kprev += kp;
            continue;
        }
        SplitArgs<T> A{};
        const bool raw = (p == 0 && b != nullptr);  // b == nullptr: normalised input (b = 1, tds_solve_normalized)
        if (p == 0) {
            A.a = a;
            A.b = b;
            A.c = c;
            A.d = d;
            A.in_stride = I.batch_stride;
        } else {
            const int ib = (p - 1) & 1;
            A.a = w.a[ib];
            A.b = nullptr;
            A.c = w.c[ib];
            A.d = w.d[ib];
            A.in_stride = slot_rows(I.n, kprev, I.dtype);
        }
        const int ob = p & 1;
        A.oa = w.a[ob];
        A.oc = w.c[ob];
        A.od = w.d[ob];
        A.n = I.n;
        A.out_slot = slot_rows(I.n, kprev + kp, I.dtype);
        A.kp = kp;
        A.tile = P.split_tile_rows;
        A.geom.npass = p;
        for (int q = 0; q < kMaxPasses; ++q) A.geom.kpass[q] = q < p ? P.k_pass[q] : 0;
        const int64_t m_in = I.m << kprev;
        const int64_t len_in = cdiv(I.n, int64_t(1) << kprev);
        A.segs = split_segments(m_in, cdiv(len_in, split_tile_eff(P, p)), P.theta);
        const int64_t e = P.split_tile_rows + 2 * ((int64_t(1) << kp) - 1);
        A.ep = int32_t(e + (e >> std::max(kp, 5)) + 1);
        A.vec = p == 0 ? (raw ? vec_ok(I, {a, b, c, d}) : vec_ok(I, {a, c, d})) : 1;
        if (natural) {  // strided variant: one pass, rows kept in original order (per system stride)
            A.natural = 1;
            A.out_slot = natural_stride<T>(I.n);
        }
        const int64_t grid = m_in * A.segs;
        if (grid > 0x7fffffffLL) return fail(TDS_ERR_UNSUPPORTED, "split grid exceeds 2^31-1 CTAs");
        cudaError_t err;
        if (sc && !(kp <= kPipeSplitMaxKp && A.vec))
            return fail(TDS_ERR_UNSUPPORTED, "a scatter needs the TMA split kernel (k <= 8, 16-byte aligned rows)");
        if (kp <= kPipeSplitMaxKp && A.vec) {
            // persistent, TMA-prefetched register kernel (16-byte aligned rows)
            err = launch_split_pipe<T>(A, raw, m_in, len_in, I.params.split_threads, st, sc);
        } else if (kp <= kRegSplitMaxKp) {
            err = launch_split_reg<T>(A, raw, grid, st);
        } else {
            const size_t smem = split_smem_bytes(I.dtype, P.split_tile_rows, kp);
            err = launch_split_pass<T>(A, raw, grid, P.split_threads, smem, st);
        }
        if (err != cudaSuccess) return cuda_fail(err, "split_pass launch");
        kprev += kp;
    }
    *out_buf = (P.passes - 1) & 1;
    return TDS_OK;
}

template <typename T>
static tds_status solve_impl(const tds_plan_info &I, const T *a, const T *b, const T *c, const T *d, T *x,
                             void *ws, cudaStream_t st, int first = 0, int last = 1 << 30,
                             const XScatterHost *xsc = nullptr) {
    const tds_params &P = I.params;
    OnchipArgs<T> A{};
    A.x = x;
    A.n = I.n;
    A.batch_stride = I.batch_stride;
    A.K = P.k;
    A.m_systems = I.m;
    int t = P.thomas_chains, l2 = 0;
    while ((1 << l2) < t) ++l2;
    A.log2T = l2;
    A.cluster = P.cluster;
    A.tl_levels = P.tl_levels;
    A.x_group = P.x_group;
    // strided variant (the paper's in-place subsystems): needs the TMA split kernel (16-byte aligned input)
    const bool strided_ok = P.strided && P.k > 0 && vec_ok(I, {a, b, c, d});
    if (P.strided == 2 && !strided_ok)  // no de-interleaved fallback: the plan's CTA size is the coalesced kernel's
        return fail(TDS_ERR_UNSUPPORTED, "strided 2 needs 16-byte aligned a, b, c, d and batch_stride");
    int64_t grid;
    if (P.k == 0) {
        A.a = a;
        A.b = b;
        A.c = c;
        A.d = d;
        A.vec = vec_ok(I, {a, b, c, d, x});
        grid = I.m * P.cluster;
    } else {
        A.vec = 1;
        WsBufs<T> w = ws_bufs<T>(I, ws);
        int ob = 0;
        tds_status s = run_split<T>(I, a, b, c, d, w, st, &ob, first, last, strided_ok);
        if (s != TDS_OK) return s;
        A.a = w.a[ob];
        A.b = nullptr;
        A.c = w.c[ob];
        A.d = w.d[ob];
        A.xs = w.a[ob];  // per-subsystem x overwrites a (each CTA reads its rows before writing them)
        A.slot = I.slot_rows;
        // the on-chip kernel is the last reader of c', d': their whole 128-byte
        // lines are dropped from L2 once loaded (no write-back of dead scratch)
        A.l2_discard = (I.slot_rows * int64_t(sizeof(T))) % 128 == 0 && uintptr_t(A.c) % 128 == 0 &&
                       uintptr_t(A.d) % 128 == 0;
        A.geom.npass = P.passes;
        for (int q = 0; q < kMaxPasses; ++q) A.geom.kpass[q] = P.k_pass[q];
        grid = (I.m << P.k) * P.cluster;
    }
    if (P.passes >= first && P.passes <= last) {
        if (grid > 0x7fffffffLL) return fail(TDS_ERR_UNSUPPORTED, "on-chip grid exceeds 2^31-1 CTAs");
        cudaError_t err;
        if (strided_ok && P.strided == 2) {
            // coalesced 32-byte sectors of G adjacent residues, rows beyond shared memory in the workspace
            WsBufs<T> w = ws_bufs<T>(I, ws);
            int l2t = 0;
            while ((1 << l2t) < P.thomas_chains) ++l2t;
            const int64_t smem_budget = int64_t(smem_optin_current()) - kSmemReserve;
            err = launch_onchip_coalesced<T>(w.a, w.c, w.d, x, I.n, I.m, I.batch_stride, natural_stride<T>(I.n), P.k,
                                             l2t, smem_budget, st);
        } else if (strided_ok) {
            // gather residue classes with stride 2^k from the in-place split output, x scattered in place
            A.x = x;
            err = launch_onchip_strided<T>(A, I.m << P.k, I.onchip_threads, natural_stride<T>(I.n), st);
        } else if (P.k == 0 && onchip_cpipe_ok(I) && A.vec) {
            // persistent, TMA-fed warp-form kernel on one CTA or a 2-CTA cluster per system
            err = launch_onchip_cpipe<T>(A, I.onchip_threads, sm_count_current(), st);
        } else if (P.x_group > 0 && uintptr_t(x) % 16 == 0) {
            // cluster of x_group CTAs on adjacent residue classes, x stored in place (no placement kernel)
            err = launch_onchip_gpipe<T>(A, I.m << P.k, I.onchip_threads, sm_count_current(), st);
        } else if (onchip_pipe_ok(I)) {
            // persistent, TMA-pipelined form (cluster == 1, 64 bytes of rows per thread)
            const int sms = sm_count_current();
            const size_t smem = onchip_pipe_smem_bytes(I.dtype, I.onchip_threads, 1 << P.cr_levels, P.tl_levels);
            err = launch_onchip_pipe<T>(A, I.m << P.k, I.onchip_threads, P.cr_levels, sms, smem, st);
        } else {
            const size_t smem = onchip_smem_bytes(I.dtype, I.onchip_threads, P.cluster, P.tl_levels);
            err = launch_onchip<T>(A, P.cr_levels, P.k == 0, grid, I.onchip_threads, smem, st);
        }
        if (err != cudaSuccess) return cuda_fail(err, "onchip launch");
    }
    // x_group plans place x inside the on-chip stage (a misaligned x falls back
    // to the slot kernel + placement, both counted as that one stage)
    const bool fused = P.x_group > 0 || P.strided;
    const bool fused_ok = P.strided ? strided_ok : uintptr_t(x) % 16 == 0;
    const bool place = !fused ? P.passes + 1 >= first && P.passes + 1 <= last
                              : !fused_ok && P.passes >= first && P.passes <= last;
    if (P.k > 0 && place) {
        cudaError_t err = launch_place_x<T>(A.xs, x, I.n, I.m, I.batch_stride, I.slot_rows, P.k,
                                            xsc ? 1 : vec_ok(I, {(const void *)x}), A.geom, st, true, xsc);
        if (err != cudaSuccess) return cuda_fail(err, "place_x launch");
    }
    return TDS_OK;
}

int32_t onchip_form_of(const tds_plan_info &I) {
    const tds_params &P = I.params;
    bool warp;
    if (P.strided == 2) warp = false;  // onchip_coalesced: PCR levels + Thomas per chain
    else if (P.strided || P.x_group > 0) warp = true;  // onchip_strided / onchip_gpipe: solve_item_warp
    else if (P.k == 0) warp = onchip_cpipe_ok(I);
    else warp = onchip_pipe_ok(I) && P.tl_levels == 5;
    return warp ? TDS_FORM_WARP_CR : TDS_FORM_PCR_THOMAS;
}

// Gather workspace slots into the canonical order (diagnostic path only).
template <typename T>
__global__ void gather_canonical_kernel(const T *sa, const T *sc, const T *sd, T *oa, T *oc, T *od, int64_t n,
                                        int32_t K, int64_t slot, PassGeom geom) {
    const int64_t sigma = blockIdx.x;
    const int64_t sys = sigma >> K;
    const int64_t r = sigma & ((int64_t(1) << K) - 1);
    if (r >= n) return;
    const int64_t L = (n - r + (int64_t(1) << K) - 1) >> K;
    const int64_t q = n >> K, rem = n & ((int64_t(1) << K) - 1);
    const int64_t off = r * q + (r < rem ? r : rem);
    for (int64_t j = threadIdx.x; j < L; j += blockDim.x) {
        const int64_t i = sigma * slot + j, o = sys * n + off + j;
        oa[o] = sa[i];
        oc[o] = sc[i];
        od[o] = sd[i];
    }
}

template <typename T>
static tds_status split_impl(const tds_plan_info &I, const T *a, const T *b, const T *c, const T *d, T *oa,
                             T *oc, T *od, void *ws, cudaStream_t st) {
    WsBufs<T> w = ws_bufs<T>(I, ws);
    int ob = 0;
    tds_status s = run_split<T>(I, a, b, c, d, w, st, &ob);
    if (s != TDS_OK) return s;
    PassGeom g{};
    g.npass = I.params.passes;
    for (int q = 0; q < kMaxPasses; ++q) g.kpass[q] = I.params.k_pass[q];
    const int64_t grid = I.m << I.params.k;
    if (grid > 0x7fffffffLL) return fail(TDS_ERR_UNSUPPORTED, "grid too large");
    gather_canonical_kernel<T><<<(unsigned)grid, 256, 0, st>>>(w.a[ob], w.c[ob], w.d[ob], oa, oc, od, I.n,
                                                                 I.params.k, I.slot_rows, g);
    cudaError_t err = cudaGetLastError();
    if (err != cudaSuccess) return cuda_fail(err, "gather launch");
    return TDS_OK;
}

// Run launches [first, last] of the chunked sequence: for each chunk of
// chunk_systems systems, S = passes + 1 + (k > 0 && x_group == 0 && strided == 0) kernels.  Chunks reuse one
// workspace, so a chunk's split output is still in L2 when its on-chip kernel
// and x placement read it.
template <typename T>
static tds_status solve_chunks(const tds_plan_info &I, const T *a, const T *b, const T *c, const T *d, T *x,
                               void *ws, cudaStream_t st, int first, int last) {
    const int S = I.params.passes + 1 + (I.params.k > 0 && I.params.x_group == 0 && !I.params.strided ? 1 : 0);
    const int64_t mc = chunk_m(I.params, I.m);
    for (int64_t ch = 0; ch * mc < I.m; ++ch) {
        const int lf = std::max<int64_t>(first - ch * S, 0);
        const int ll = (int)std::min<int64_t>(last - ch * S, S - 1);
        if (lf > ll) continue;
        tds_plan_info Ic = I;
        Ic.m = std::min<int64_t>(mc, I.m - ch * mc);
        const int64_t off = ch * mc * I.batch_stride;
        tds_status s = solve_impl<T>(Ic, a + off, b + off, c + off, d + off, x + off, ws, st, lf, ll);
        if (s != TDS_OK) return s;
    }
    return TDS_OK;
}

template <typename T>
static tds_status split_chunks(const tds_plan_info &I, const T *a, const T *b, const T *c, const T *d, T *oa,
                               T *oc, T *od, void *ws, cudaStream_t st) {
    const int64_t mc = chunk_m(I.params, I.m);
    for (int64_t ch = 0; ch * mc < I.m; ++ch) {
        tds_plan_info Ic = I;
        Ic.m = std::min<int64_t>(mc, I.m - ch * mc);
        const int64_t off = ch * mc * I.batch_stride, oo = ch * mc * I.n;
        tds_status s = split_impl<T>(Ic, a + off, b + off, c + off, d + off, oa + oo, oc + oo, od + oo, ws, st);
        if (s != TDS_OK) return s;
    }
    return TDS_OK;
}

// Interleaved layout (tds_solve_interleaved): the plan's workspace, then the
// four transposed (system-major) arrays, each rounded to 256 bytes; x is
// solved in place over the transposed d.
static size_t interleaved_array_bytes(const tds_plan_info &I) {
    return size_t(round_up(I.m * I.n * dsize(I.dtype), 256));
}
static tds_status interleaved_plan_ok(const tds_plan_st *plan) {
    if (!plan) return fail(TDS_ERR_INVALID_ARG, "plan is NULL");
    if (plan->info.params.split_only) return fail(TDS_ERR_UNSUPPORTED, "split-only plan: use tds_split_batched");
    if (plan->info.batch_stride != plan->info.n)
        return fail(TDS_ERR_UNSUPPORTED, "interleaved layout needs a dense plan (batch_stride == n)");
    return TDS_OK;
}

template <typename T>
static tds_status solve_interleaved_impl(const tds_plan_info &I, const T *a, const T *b, const T *c, const T *d,
                                         T *x, void *ws, cudaStream_t st) {
    char *base = static_cast<char *>(ws) + round_up(int64_t(I.workspace_bytes), 256);
    const size_t ab = interleaved_array_bytes(I);
    T *sys[4];
    for (int q = 0; q < 4; ++q) sys[q] = reinterpret_cast<T *>(base + q * ab);
    const T *in[4] = {a, b, c, d};
    cudaError_t e = launch_transpose<T>(in, sys, 4, I.n, I.m, st);  // n x m -> m x n
    if (e != cudaSuccess) return cuda_fail(e, "interleave transpose launch");
    tds_status s = solve_chunks<T>(I, sys[0], sys[1], sys[2], sys[3], sys[3], ws, st, 0, I.launches - 1);
    if (s != TDS_OK) return s;
    const T *xin[1] = {sys[3]};
    T *xout[1] = {x};
    e = launch_transpose<T>(xin, xout, 1, I.m, I.n, st);  // m x n -> n x m
    if (e != cudaSuccess) return cuda_fail(e, "interleave transpose launch");
    return TDS_OK;
}

// Launch geometry of every kernel of a solve, checked before the first launch
// (so an UNSUPPORTED never leaves earlier launches of the same call enqueued).
static tds_status check_geometry(const tds_plan_info &I) {
    const tds_params &P = I.params;
    const int64_t mc = chunk_m(P, I.m);  // the largest chunk
    int kprev = 0;
    for (int p = 0; p < P.passes; ++p) {
        const int64_t m_in = mc << kprev;
        const int64_t len_in = cdiv(I.n, int64_t(1) << kprev);
        const int64_t segs = split_segments(m_in, cdiv(len_in, split_tile_eff(P, p)), P.theta);
        if (m_in * segs > 0x7fffffffLL) return fail(TDS_ERR_UNSUPPORTED, "split grid exceeds 2^31-1 CTAs");
        kprev += P.k_pass[p];
    }
    const int64_t grid = P.k == 0 ? mc * P.cluster : (mc << P.k) * P.cluster;
    if (!P.split_only && grid > 0x7fffffffLL) return fail(TDS_ERR_UNSUPPORTED, "on-chip grid exceeds 2^31-1 CTAs");
    return TDS_OK;
}

static tds_status check_arrays(const tds_plan_info &I, std::initializer_list<const void *> ptrs) {
    const size_t es = size_t(dsize(I.dtype));
    for (const void *p : ptrs) {
        if (!p) return fail(TDS_ERR_INVALID_ARG, "NULL array pointer");
        if (reinterpret_cast<uintptr_t>(p) % es) return fail(TDS_ERR_INVALID_ARG, "array not aligned to sizeof(T)");
    }
    return TDS_OK;
}

}  // namespace tds

using namespace tds;

extern "C" {

tds_status tds_device_props_query(int device, tds_device_props *out) {
    if (!out) return fail(TDS_ERR_INVALID_ARG, "out is NULL");
    cudaDeviceProp p;
    cudaError_t e = cudaGetDeviceProperties(&p, device);
    if (e != cudaSuccess) return cuda_fail(e, "cudaGetDeviceProperties");
    int optin = 0;
    e = cudaDeviceGetAttribute(&optin, cudaDevAttrMaxSharedMemoryPerBlockOptin, device);
    if (e != cudaSuccess) return cuda_fail(e, "cudaDeviceGetAttribute");
    std::memset(out, 0, sizeof(*out));
    out->sm_count = p.multiProcessorCount;
    out->smem_optin_bytes = optin;
    out->smem_per_sm_bytes = (int32_t)p.sharedMemPerMultiprocessor;
    out->regs_per_sm = p.regsPerMultiprocessor;
    out->max_threads_per_block = p.maxThreadsPerBlock;
    out->warp_size = p.warpSize;
    out->cc_major = p.major;
    out->cc_minor = p.minor;
    out->l2_bytes = p.l2CacheSize;
    out->global_mem_bytes = (int64_t)p.totalGlobalMem;
    return TDS_OK;
}

tds_status tds_solve_batched(const tds_plan_t plan, const void *a, const void *b, const void *c, const void *d,
                             void *x, void *workspace, size_t workspace_bytes, void *cuda_stream) {
    if (!plan) return fail(TDS_ERR_INVALID_ARG, "plan is NULL");
    return tds_solve_stages(plan, a, b, c, d, x, workspace, workspace_bytes, cuda_stream, 0,
                            plan->info.launches - 1);
}

tds_status tds_solve_stages(const tds_plan_t plan, const void *a, const void *b, const void *c, const void *d,
                            void *x, void *workspace, size_t workspace_bytes, void *cuda_stream,
                            int32_t first_stage, int32_t last_stage) {
    if (!plan) return fail(TDS_ERR_INVALID_ARG, "plan is NULL");
    const tds_plan_info &I = plan->info;
    if (I.params.split_only) return fail(TDS_ERR_UNSUPPORTED, "split-only plan: use tds_split_batched");
    if (first_stage < 0 || last_stage >= I.launches || first_stage > last_stage)
        return fail(TDS_ERR_INVALID_ARG, "launch range outside [0, info.launches)");
    tds_status s = check_arrays(I, {a, b, c, d, x});
    if (s != TDS_OK) return s;
    const size_t bytes = size_t(((I.m - 1) * I.batch_stride + I.n) * dsize(I.dtype));
    for (const void *p : {a, b, c})
        if (overlaps(x, bytes, p, bytes)) return fail(TDS_ERR_INVALID_ARG, "x overlaps a, b or c");
    if (x != d && overlaps(x, bytes, d, bytes))
        return fail(TDS_ERR_INVALID_ARG, "x partially overlaps d (only x == d is allowed)");
    if ((s = check_workspace(I, workspace, workspace_bytes)) != TDS_OK) return s;
    if (workspace && I.workspace_bytes)
        for (const void *p : {a, b, c, d, (const void *)x})
            if (overlaps(workspace, I.workspace_bytes, p, bytes))
                return fail(TDS_ERR_INVALID_ARG, "workspace overlaps an array");
    if ((s = check_geometry(I)) != TDS_OK) return s;
    if ((s = check_device(plan)) != TDS_OK) return s;
    cudaStream_t st = static_cast<cudaStream_t>(cuda_stream);
    s = I.dtype == TDS_F32
            ? solve_chunks<float>(I, (const float *)a, (const float *)b, (const float *)c, (const float *)d,
                                  (float *)x, workspace, st, first_stage, last_stage)
            : solve_chunks<double>(I, (const double *)a, (const double *)b, (const double *)c,
                                   (const double *)d, (double *)x, workspace, st, first_stage, last_stage);
    if (s == TDS_OK) clear_error();
    return s;
}

tds_status tds_split_batched(const tds_plan_t plan, const void *a, const void *b, const void *c, const void *d,
                             void *a_out, void *c_out, void *d_out, void *workspace, size_t workspace_bytes,
                             void *cuda_stream) {
    if (!plan) return fail(TDS_ERR_INVALID_ARG, "plan is NULL");
    const tds_plan_info &I = plan->info;
    if (I.params.k < 1) return fail(TDS_ERR_INVALID_ARG, "tds_split_batched needs k >= 1");
    tds_status s = check_arrays(I, {a, b, c, d, a_out, c_out, d_out});
    if (s != TDS_OK) return s;
    if ((s = check_workspace(I, workspace, workspace_bytes)) != TDS_OK) return s;
    if ((s = check_device(plan)) != TDS_OK) return s;
    cudaStream_t st = static_cast<cudaStream_t>(cuda_stream);
    s = I.dtype == TDS_F32
            ? split_chunks<float>(I, (const float *)a, (const float *)b, (const float *)c, (const float *)d,
                                  (float *)a_out, (float *)c_out, (float *)d_out, workspace, st)
            : split_chunks<double>(I, (const double *)a, (const double *)b, (const double *)c,
                                   (const double *)d, (double *)a_out, (double *)c_out, (double *)d_out, workspace,
                                   st);
    if (s == TDS_OK) clear_error();
    return s;
}

static tds_status check_solve_args(const tds_plan_info &I, const void *a, const void *b, const void *c,
                                   const void *d, void *x, void *workspace, size_t workspace_bytes) {
    tds_status s = b ? check_arrays(I, {a, b, c, d, x}) : check_arrays(I, {a, c, d, x});
    if (s != TDS_OK) return s;
    const size_t bytes = size_t(((I.m - 1) * I.batch_stride + I.n) * dsize(I.dtype));
    for (const void *p : {a, b, c})
        if (p && overlaps(x, bytes, p, bytes)) return fail(TDS_ERR_INVALID_ARG, "x overlaps a, b or c");
    if (x != d && overlaps(x, bytes, d, bytes))
        return fail(TDS_ERR_INVALID_ARG, "x partially overlaps d (only x == d is allowed)");
    if ((s = check_workspace(I, workspace, workspace_bytes)) != TDS_OK) return s;
    if (workspace && I.workspace_bytes)
        for (const void *p : {a, b, c, d, (const void *)x})
            if (p && overlaps(workspace, I.workspace_bytes, p, bytes))
                return fail(TDS_ERR_INVALID_ARG, "workspace overlaps an array");
    return TDS_OK;
}

tds_status tds_solve_normalized(const tds_plan_t plan, const void *a, const void *c, const void *d, void *x,
                                void *workspace, size_t workspace_bytes, void *cuda_stream) {
    if (!plan) return fail(TDS_ERR_INVALID_ARG, "plan is NULL");
    const tds_plan_info &I = plan->info;
    if (I.params.split_only) return fail(TDS_ERR_UNSUPPORTED, "split-only plan");
    if (I.params.k < 1 || I.params.strided)
        return fail(TDS_ERR_UNSUPPORTED, "normalised input needs a plan with k >= 1 split levels and strided = 0");
    tds_status s = check_solve_args(I, a, nullptr, c, d, x, workspace, workspace_bytes);
    if (s != TDS_OK) return s;
    if ((s = check_geometry(I)) != TDS_OK) return s;
    if ((s = check_device(plan)) != TDS_OK) return s;
    cudaStream_t st = static_cast<cudaStream_t>(cuda_stream);
    s = I.dtype == TDS_F32
            ? solve_chunks<float>(I, (const float *)a, nullptr, (const float *)c, (const float *)d, (float *)x,
                                  workspace, st, 0, I.launches - 1)
            : solve_chunks<double>(I, (const double *)a, nullptr, (const double *)c, (const double *)d, (double *)x,
                                   workspace, st, 0, I.launches - 1);
    if (s == TDS_OK) clear_error();
    return s;
}

tds_status tds_solve_normalized_xscatter(const tds_plan_t plan, const void *a, const void *c, const void *d,
                                         const tds_xscatter *spec, void *workspace, size_t workspace_bytes,
                                         void *cuda_stream) {
    if (!plan || !spec) return fail(TDS_ERR_INVALID_ARG, "NULL argument");
    const tds_plan_info &I = plan->info;
    const tds_params &P = I.params;
    if (P.split_only || P.k < 5 || P.strided || P.x_group || I.chunks != 1)
        return fail(TDS_ERR_UNSUPPORTED, "an x scatter needs k >= 5, no chunking, strided 0, x_group 0 (the TMA "
                                         "placement)");
    const int64_t es = dsize(I.dtype);
    const int64_t KK = int64_t(1) << P.k, E = 128 / es;
    const int64_t jb = spec->rows_per_group / KK;
    if (spec->groups < 1 || spec->groups > 8 || spec->rows_per_group * spec->groups != I.n || I.n % KK ||
        spec->rows_per_group % KK || jb % (4 * E) || spec->dst_system_stride < spec->rows_per_group ||
        (spec->dst_system_stride * es) % 16)
        return fail(TDS_ERR_INVALID_ARG, "groups in [1, 8] with groups * rows_per_group == n; rows_per_group a "
                                         "multiple of 2^k * 4 * 128 bytes / sizeof(T); dst_system_stride >= "
                                         "rows_per_group in 16-byte units");
    tds_status s = check_solve_args(I, a, nullptr, c, d, const_cast<void *>(d), workspace, workspace_bytes);
    if (s != TDS_OK) return s;
    XScatterHost xsc{};
    xsc.groups = spec->groups;
    xsc.rows_per_group = spec->rows_per_group;
    xsc.dst_system_stride = spec->dst_system_stride;
    const size_t in_bytes = size_t(((I.m - 1) * I.batch_stride + I.n) * es);
    const size_t dbytes = size_t(((I.m - 1) * spec->dst_system_stride + spec->rows_per_group) * es);
    for (int h = 0; h < spec->groups; ++h) {
        const void *p = spec->dst[h];
        if (!p || reinterpret_cast<uintptr_t>(p) % 16) return fail(TDS_ERR_INVALID_ARG, "NULL or misaligned dst");
        for (const void *q : {a, c, d})
            if (overlaps(p, dbytes, q, in_bytes)) return fail(TDS_ERR_INVALID_ARG, "dst overlaps an input");
        if (workspace && overlaps(p, dbytes, workspace, I.workspace_bytes))
            return fail(TDS_ERR_INVALID_ARG, "dst overlaps the workspace");
        xsc.dst[h] = spec->dst[h];
    }
    if ((s = check_geometry(I)) != TDS_OK) return s;
    if ((s = check_device(plan)) != TDS_OK) return s;
    cudaStream_t st = static_cast<cudaStream_t>(cuda_stream);
    s = I.dtype == TDS_F32
            ? solve_impl<float>(I, (const float *)a, nullptr, (const float *)c, (const float *)d, nullptr, workspace,
                                st, 0, 1 << 30, &xsc)
            : solve_impl<double>(I, (const double *)a, nullptr, (const double *)c, (const double *)d, nullptr,
                                 workspace, st, 0, 1 << 30, &xsc);
    if (s == TDS_OK) clear_error();
    return s;
}

tds_status tds_plan_slots_layout(const tds_plan_t plan, tds_slots_layout *out) {
    if (!plan || !out) return fail(TDS_ERR_INVALID_ARG, "NULL argument");
    const tds_plan_info &I = plan->info;
    if (I.params.k < 1 || I.params.strided) return fail(TDS_ERR_UNSUPPORTED, "slots need k >= 1 and strided = 0");
    if (I.chunks != 1) return fail(TDS_ERR_UNSUPPORTED, "slots of a chunked plan are reused per chunk");
    const int nbuf = I.params.passes >= 2 || I.params.strided == 2 ? 2 : 1;
    const int64_t E = int64_t(I.workspace_bytes / (size_t(nbuf) * 3 * size_t(dsize(I.dtype))));
    const int ob = (I.params.passes - 1) & 1;
    out->a_offset = (3 * ob + 0) * E;
    out->c_offset = (3 * ob + 1) * E;
    out->d_offset = (3 * ob + 2) * E;
    out->slot_rows = I.slot_rows;
    out->num_slots = I.m << I.params.k;
    return TDS_OK;
}

tds_status tds_split_slots(const tds_plan_t plan, const void *a, const void *b, const void *c, const void *d,
                           void *workspace, size_t workspace_bytes, void *cuda_stream) {
    tds_slots_layout L;
    tds_status s = tds_plan_slots_layout(plan, &L);
    if (s != TDS_OK) return s;
    const tds_plan_info &I = plan->info;
    if ((s = check_arrays(I, {a, b, c, d})) != TDS_OK) return s;
    if ((s = check_workspace(I, workspace, workspace_bytes)) != TDS_OK) return s;
    const size_t bytes = size_t(((I.m - 1) * I.batch_stride + I.n) * dsize(I.dtype));
    for (const void *p : {a, b, c, d})
        if (overlaps(workspace, I.workspace_bytes, p, bytes)) return fail(TDS_ERR_INVALID_ARG, "workspace overlaps an array");
    if ((s = check_geometry(I)) != TDS_OK) return s;
    if ((s = check_device(plan)) != TDS_OK) return s;
    cudaStream_t st = static_cast<cudaStream_t>(cuda_stream);
    int ob = 0;
    if (I.dtype == TDS_F32) {
        WsBufs<float> w = ws_bufs<float>(I, workspace);
        s = run_split<float>(I, (const float *)a, (const float *)b, (const float *)c, (const float *)d, w, st, &ob);
    } else {
        WsBufs<double> w = ws_bufs<double>(I, workspace);
        s = run_split<double>(I, (const double *)a, (const double *)b, (const double *)c, (const double *)d, w, st,
                              &ob);
    }
    if (s == TDS_OK) clear_error();
    return s;
}

tds_status tds_split_scatter(const tds_plan_t plan, const void *a, const void *b, const void *c, const void *d,
                             const tds_scatter *spec, void *cuda_stream) {
    if (!plan || !spec) return fail(TDS_ERR_INVALID_ARG, "NULL argument");
    const tds_plan_info &I = plan->info;
    const tds_params &P = I.params;
    if (P.passes != 1 || P.k_pass[0] > kPipeSplitMaxKp || I.m != 1 || P.strided || I.chunks != 1)
        return fail(TDS_ERR_UNSUPPORTED, "a scatter needs one system (m = 1) split in ONE pass of <= 8 levels");
    const int64_t NR = int64_t(1) << P.k;
    if (spec->groups < 1 || spec->groups > 8 || int64_t(spec->residues_per_group) * spec->groups != NR)
        return fail(TDS_ERR_INVALID_ARG, "groups in [1, 8] and groups * residues_per_group == 2^k");
    const int64_t es = dsize(I.dtype);
    // (TMA tensor stores need 16-byte aligned box starts: the tiles' store coordinates
    // are whole 16-byte runs after the shift by first_pos only if first_pos is)
    if (spec->first_pos < 0 || spec->num_pos < 1 || spec->first_pos + spec->num_pos > I.n / NR ||
        spec->dst_stride < spec->num_pos || (spec->dst_stride * es) % 16 || (spec->first_pos * es) % 16 ||
        (spec->num_pos * es) % 16)
        return fail(TDS_ERR_INVALID_ARG, "positions [first_pos, first_pos + num_pos) within floor(n / 2^k); "
                                         "first_pos, num_pos and dst_stride (>= num_pos) in 16-byte units");
    tds_status s = check_arrays(I, {a, b, c, d});
    if (s != TDS_OK) return s;
    if (!vec_ok(I, {a, b, c, d})) return fail(TDS_ERR_UNSUPPORTED, "a scatter needs 16-byte aligned a, b, c, d");
    ScatterHost sc{};
    sc.groups = spec->groups;
    sc.q = spec->residues_per_group;
    sc.first_pos = spec->first_pos;
    sc.num_pos = spec->num_pos;
    sc.dst_stride = spec->dst_stride;
    const size_t bytes = size_t(((I.m - 1) * I.batch_stride + I.n) * es);
    const size_t dbytes = size_t((int64_t(sc.q - 1) * spec->dst_stride + spec->num_pos) * es);
    for (int t = 0; t < 3; ++t)
        for (int h = 0; h < sc.groups; ++h) {
            const void *p = spec->dst[t][h];
            if (!p || reinterpret_cast<uintptr_t>(p) % 16) return fail(TDS_ERR_INVALID_ARG, "NULL or misaligned dst");
            for (const void *q : {a, b, c, d})
                if (overlaps(p, dbytes, q, bytes)) return fail(TDS_ERR_INVALID_ARG, "dst overlaps an input");
            sc.dst[t][h] = spec->dst[t][h];
        }
    if ((s = check_geometry(I)) != TDS_OK) return s;
    if ((s = check_device(plan)) != TDS_OK) return s;
    cudaStream_t st = static_cast<cudaStream_t>(cuda_stream);
    int ob = 0;
    if (I.dtype == TDS_F32) {
        WsBufs<float> w{};
        s = run_split<float>(I, (const float *)a, (const float *)b, (const float *)c, (const float *)d, w, st, &ob, 0,
                             1 << 30, false, &sc);
    } else {
        WsBufs<double> w{};
        s = run_split<double>(I, (const double *)a, (const double *)b, (const double *)c, (const double *)d, w, st,
                              &ob, 0, 1 << 30, false, &sc);
    }
    if (s == TDS_OK) clear_error();
    return s;
}

tds_status tds_unpack_residues(tds_dtype dtype, int64_t n, int64_t m, int32_t k, int64_t slot_rows, const void *xs,
                               void *x, int64_t batch_stride, void *cuda_stream) {
    if (dtype != TDS_F32 && dtype != TDS_F64) return fail(TDS_ERR_INVALID_ARG, "dtype");
    if (n < 1 || m < 1 || k < 1 || k > 30) return fail(TDS_ERR_INVALID_ARG, "n, m >= 1 and 1 <= k <= 30");
    if (batch_stride == 0) batch_stride = n;
    if (batch_stride < n) return fail(TDS_ERR_INVALID_ARG, "batch_stride < n");
    const int64_t es = dsize(dtype);
    if (slot_rows < cdiv(n, int64_t(1) << k)) return fail(TDS_ERR_INVALID_ARG, "slot_rows < ceil(n / 2^k)");
    if (!xs || !x || reinterpret_cast<uintptr_t>(xs) % es || reinterpret_cast<uintptr_t>(x) % es)
        return fail(TDS_ERR_INVALID_ARG, "NULL or misaligned array");
    const size_t xb = size_t(((m - 1) * batch_stride + n) * es), sb = size_t((m << k) * slot_rows * es);
    if (overlaps(xs, sb, x, xb)) return fail(TDS_ERR_INVALID_ARG, "x overlaps xs");
    PassGeom g{};
    g.npass = 1;
    g.kpass[0] = k;
    cudaStream_t st = static_cast<cudaStream_t>(cuda_stream);
    tds_plan_info I{};
    I.dtype = dtype;
    I.batch_stride = batch_stride;
    const int vec = vec_ok(I, {x});
    // place_x's TMA transposer needs whole 16-byte slot rows
    const int64_t vslot = (slot_rows * es) % 16 == 0 && reinterpret_cast<uintptr_t>(xs) % 16 == 0 ? vec : 0;
    const cudaError_t e = dtype == TDS_F32
                              ? launch_place_x<float>((const float *)xs, (float *)x, n, m, batch_stride, slot_rows, k,
                                                      int(vslot), g, st, false)
                              : launch_place_x<double>((const double *)xs, (double *)x, n, m, batch_stride, slot_rows,
                                                       k, int(vslot), g, st, false);
    if (e != cudaSuccess) return cuda_fail(e, "unpack launch");
    clear_error();
    return TDS_OK;
}

tds_status tds_interleaved_workspace_bytes(const tds_plan_t plan, size_t *bytes) {
    tds_status s = interleaved_plan_ok(plan);
    if (s != TDS_OK) return s;
    if (!bytes) return fail(TDS_ERR_INVALID_ARG, "bytes is NULL");
    *bytes = size_t(round_up(int64_t(plan->info.workspace_bytes), 256)) + 4 * interleaved_array_bytes(plan->info);
    clear_error();
    return TDS_OK;
}

tds_status tds_solve_interleaved(const tds_plan_t plan, const void *a, const void *b, const void *c, const void *d,
                                 void *x, void *workspace, size_t workspace_bytes, void *cuda_stream) {
    tds_status s = interleaved_plan_ok(plan);
    if (s != TDS_OK) return s;
    const tds_plan_info &I = plan->info;
    if ((s = check_arrays(I, {a, b, c, d, x})) != TDS_OK) return s;
    const size_t bytes = size_t(I.m * I.n * dsize(I.dtype));
    for (const void *p : {a, b, c})
        if (overlaps(x, bytes, p, bytes)) return fail(TDS_ERR_INVALID_ARG, "x overlaps a, b or c");
    if (x != d && overlaps(x, bytes, d, bytes))
        return fail(TDS_ERR_INVALID_ARG, "x partially overlaps d (only x == d is allowed)");
    size_t need = 0;
    tds_interleaved_workspace_bytes(plan, &need);
    if (!workspace) return fail(TDS_ERR_WORKSPACE, "workspace is NULL");
    if (workspace_bytes < need)
        return fail(TDS_ERR_WORKSPACE, "workspace " + std::to_string(workspace_bytes) + " < required " +
                                           std::to_string(need));
    if (reinterpret_cast<uintptr_t>(workspace) % 256) return fail(TDS_ERR_WORKSPACE, "workspace not 256-byte aligned");
    for (const void *p : {a, b, c, d, (const void *)x})
        if (overlaps(workspace, need, p, bytes)) return fail(TDS_ERR_INVALID_ARG, "workspace overlaps an array");
    if ((s = check_geometry(I)) != TDS_OK) return s;
    if ((s = check_device(plan)) != TDS_OK) return s;
    cudaStream_t st = static_cast<cudaStream_t>(cuda_stream);
    s = I.dtype == TDS_F32
            ? solve_interleaved_impl<float>(I, (const float *)a, (const float *)b, (const float *)c,
                                            (const float *)d, (float *)x, workspace, st)
            : solve_interleaved_impl<double>(I, (const double *)a, (const double *)b, (const double *)c,
                                             (const double *)d, (double *)x, workspace, st);
    if (s == TDS_OK) clear_error();
    return s;
}

}  // extern "C"
