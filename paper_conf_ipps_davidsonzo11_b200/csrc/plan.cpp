// plan.cpp -- the planner: the paper's DEFAULT and machine-query ("static")
// parameter selection (§IV-B/C) turned into an integer
// plan for the B200 kernels, plus the plan-handling half of the C ABI.
//
// The rules (the method's integers are pinned
// against oracle/plan.py, the rest are build choices):
//   DEFAULT  n_sub_target = 256, theta = 16 systems,
//            T = 32 (reading R10), split tile 1024 x 256 threads, on-chip CTA
//            <= 256 threads, no clusters.
//   STATIC   n_sub_target = n_onchip_max: the largest power of two whose four
//            arrays fit in the shared memory of ONE SM ("switch as soon as it
//            fits"; "shared memory per processor", Table II
//            P:L729-730): 8192 fp32 / 4096 fp64 on B200.  T = 2 x warp size
//            (P:L666-668), theta = #SMs, split tile =
//            n_onchip_max x 512 threads, on-chip CTA <= half the maximum
//            block size, no clusters (clusters are a TUNED dimension).
//   both     k = min{k : ceil(n/2^k) <= n_sub_target}; passes = ceil(k/kp_max)
//            with kp_max = 9 (fp32) / 8 (fp64) (lowered only
//            when a device's shared memory cannot hold the pass's halo), levels
//            as equal as possible, larger first; R = 2^c the smallest power of
//            two with ceil(n_sub/R) <= on-chip cap.
#include <algorithm>
#include <cstring>
#include <new>
#include <string>

#include "tds_internal.h"

namespace tds {

static thread_local std::string g_last_error;

tds_status fail(tds_status st, const std::string &msg) {
    g_last_error = msg;
    return st;
}
void clear_error() { g_last_error.clear(); }

static int ilog2(int64_t v) {
    int l = 0;
    while ((int64_t(1) << (l + 1)) <= v) ++l;
    return l;
}
static bool is_pow2(int64_t v) { return v > 0 && (v & (v - 1)) == 0; }
static int64_t pow2ceil(int64_t v) {
    int64_t p = 1;
    while (p < v) p <<= 1;
    return p;
}

int64_t slot_rows(int64_t n, int kk, int32_t dtype) {
    // ceil(n / 2^kk) rounded up to 16 bytes so every slot is 16-byte aligned
    return round_up(cdiv(n, int64_t(1) << kk), 16 / dsize(dtype));
}

int32_t split_tile_eff(const tds_params &p, int pass) {
    // rows one split CTA produces per tile: the register kernel (k_p <= 4) keeps
    // 16 rows x 256 threads minus one halo thread per side; the shared-memory
    // kernel produces split_tile_rows.
    return p.k_pass[pass] <= kRegSplitMaxKp ? kRegSplitRows * kRegSplitThreads - 2 * kRegSplitRows
                                            : p.split_tile_rows;
}

int64_t chunk_m(const tds_params &p, int64_t m) {
    return (p.chunk_systems <= 0 || p.chunk_systems >= m) ? m : p.chunk_systems;
}

int32_t split_segments(int64_t m_in, int64_t tiles, int32_t theta) {
    // Fig. 1: cooperative splitting (stage 1, several CTAs per
    // system) only while there are fewer than theta independent systems.
    if (m_in >= theta) return 1;
    return (int32_t)std::max<int64_t>(1, std::min<int64_t>(tiles, cdiv(theta, m_in)));
}

size_t split_smem_bytes(int32_t dtype, int32_t tile, int kp) {
    int64_t halo = (int64_t(1) << kp) - 1;
    int64_t e = tile + 2 * halo;
    int64_t ep = e + (e >> std::max(kp, 5)) + 1;  // bank-conflict padding: index + (index >> max(kp,5))
    return size_t(3 * ep * dsize(dtype));
}

size_t onchip_smem_bytes(int32_t dtype, int32_t threads, int32_t cluster, int32_t tl_levels) {
    // leader's reduced system [3][cluster * (threads >> c2)] + thread-level rows [4][threads]
    // + warp-edge exchange [2][3][threads/32] + ghosts (12 + 30) + 1, rounded up
    return size_t((3 * int64_t(cluster) * (threads >> tl_levels) + 4 * int64_t(threads) + 6 * (threads / 32) +
                   48) * dsize(dtype));
}

int32_t static_cluster(const tds_device_props &p) {
    // thread-block clusters (DSMEM) exist from compute capability 9.0; 8 is the portable maximum
    return p.cc_major >= 9 ? 8 : 1;
}

static int64_t n_onchip_max(const tds_device_props &p, int32_t dtype) {
    // "switch as soon as it fits" in the shared memory of one
    // processor (Table II): the largest power of two n with
    // 4 n sizeof(T) <= smem_optin - reserve
    const int64_t budget = int64_t(p.smem_optin_bytes) - kSmemReserve;
    int64_t n = 1;
    while (4 * (n * 2) * dsize(dtype) <= budget) n *= 2;
    return n;
}

static int kp_limit(const tds_device_props &props, int32_t dtype, int32_t tile) {
    int kp = 12;
    while (kp > 1 && ((int64_t(1) << kp) > tile ||
                      (int64_t)split_smem_bytes(dtype, tile, kp) >
                          int64_t(props.smem_optin_bytes) - kSmemReserve))
        --kp;
    return kp;
}

tds_status derive(tds_plan_info &info, const tds_device_props &props, const tds_params &p) {
    const int64_t n = info.n, m = info.m;
    const int32_t dtype = info.dtype;
    // --- validate the tunables against the kernels' limits
    if (p.k < 0 || p.k > 40) return fail(TDS_ERR_INVALID_ARG, "k out of range");
    if ((p.k == 0) != (p.passes == 0) || p.passes < 0 || p.passes > TDS_MAX_PASSES)
        return fail(TDS_ERR_INVALID_ARG, "passes must be 0 iff k == 0, <= 8");
    int ksum = 0;
    for (int i = 0; i < TDS_MAX_PASSES; ++i) {
        if (i < p.passes) {
            if (p.k_pass[i] < 1) return fail(TDS_ERR_INVALID_ARG, "k_pass[i] >= 1");
            ksum += p.k_pass[i];
        } else if (p.k_pass[i] != 0) {
            return fail(TDS_ERR_INVALID_ARG, "unused k_pass entries must be 0");
        }
    }
    if (ksum != p.k) return fail(TDS_ERR_INVALID_ARG, "sum(k_pass) != k");
    if (p.cr_levels < 0 || (1 << p.cr_levels) > r_max(dtype))
        return fail(TDS_ERR_UNSUPPORTED, "cr_levels exceeds the on-chip kernel's R_max");
    if (!is_pow2(p.thomas_chains)) return fail(TDS_ERR_INVALID_ARG, "thomas_chains must be a power of two");
    if (p.theta < 1) return fail(TDS_ERR_INVALID_ARG, "theta >= 1");
    if (!is_pow2(p.cluster) || p.cluster > 16) return fail(TDS_ERR_INVALID_ARG, "cluster must be 1, 2, 4, 8 or 16");
    const int R = 1 << p.cr_levels;
    if (p.cluster > 1 && (props.cc_major < 9 || R < 8))
        return fail(TDS_ERR_UNSUPPORTED, "clusters need compute capability >= 9.0 and 2^cr_levels >= 8");
    if (p.split_only != 0 && p.split_only != 1) return fail(TDS_ERR_INVALID_ARG, "split_only must be 0 or 1");
    if (p.split_only && p.k == 0) return fail(TDS_ERR_INVALID_ARG, "a split-only plan needs k >= 1");
    const int64_t n_sub = cdiv(n, int64_t(1) << std::min(p.k, 62));
    const int64_t nred = cdiv(n_sub, int64_t(R) * p.cluster);
    const bool coalesced = p.strided == 2;  // global fallback: no on-chip size limit
    const int64_t threads = p.split_only ? 32
                            : coalesced  ? coalesced_threads(dtype, n_sub, p.thomas_chains)
                                         : std::max<int64_t>(32, round_up(nred, 32));
    if (!p.split_only && !coalesced) {  // the on-chip stage must fit (a split-only plan never launches it)
        if (threads > onchip_max_threads(R, dsize(dtype)))
            return fail(TDS_ERR_UNSUPPORTED, "subsystem too large for the on-chip kernel (n_sub / (2^c cluster) > "
                                             "1024, or > 512 when 2^c * sizeof(T) >= 64)");
        if (p.tl_levels < 0 || p.tl_levels > 10 || threads % (int64_t(1) << p.tl_levels))
            return fail(TDS_ERR_INVALID_ARG, "tl_levels must be in [0, 10] and 2^tl_levels must divide the CTA size");
        if (p.thomas_chains > (threads >> p.tl_levels) * p.cluster)
            return fail(TDS_ERR_INVALID_ARG,
                        "thomas_chains > leader's reduced system (cluster x threads / 2^tl_levels)");
        if ((int64_t)onchip_smem_bytes(dtype, (int32_t)threads, p.cluster, p.tl_levels) >
            int64_t(props.smem_optin_bytes) - kSmemReserve)
            return fail(TDS_ERR_UNSUPPORTED, "on-chip shared memory exceeds the device limit");
    }
    if (p.passes > 0) {
        if (!is_pow2(p.split_tile_rows) || p.split_tile_rows < 32 || p.split_tile_rows > (1 << 15))
            return fail(TDS_ERR_INVALID_ARG, "split_tile_rows must be a power of two in [32, 32768]");
        if (p.split_threads < 32 || p.split_threads > kMaxSplitThreads || p.split_threads % 32)
            return fail(TDS_ERR_INVALID_ARG, "split_threads must be a multiple of 32 in [32, 512]");
        for (int i = 0; i < p.passes; ++i) {
            const int kp = p.k_pass[i];
            if (kp <= kRegSplitMaxKp) continue;  // register split kernel: no tile / smem limits
            if ((int64_t(1) << kp) > p.split_tile_rows)
                return fail(TDS_ERR_INVALID_ARG, "2^k_pass exceeds split_tile_rows");
            const int64_t e = p.split_tile_rows + 2 * ((int64_t(1) << kp) - 1);
            if (e > int64_t(p.split_threads) * kSplitQMax)
                return fail(TDS_ERR_UNSUPPORTED, "split tile + halo exceeds threads x 24 rows");
            if ((int64_t)split_smem_bytes(dtype, p.split_tile_rows, kp) >
                int64_t(props.smem_optin_bytes) - kSmemReserve)
                return fail(TDS_ERR_UNSUPPORTED, "split tile + halo exceeds shared memory");
        }
    }
    if (p.chunk_systems < 0) return fail(TDS_ERR_INVALID_ARG, "chunk_systems >= 0");
    if (p.strided == 1) {  // the paper's strided base-kernel variant (onchip_pipe.cu, strided kernel)
        if (p.split_only || p.passes != 1 || p.k_pass[0] > 4 || p.x_group != 0)
            return fail(TDS_ERR_UNSUPPORTED, "strided needs one split pass with k_pass <= 4 and x_group 0");
        if (p.cluster != 1 || p.tl_levels != 5 || R * dsize(dtype) != 64)
            return fail(TDS_ERR_UNSUPPORTED, "strided needs cluster 1, tl_levels 5, 64 bytes of rows per thread");
    } else if (coalesced) {  // the paper's coalesced variant with global fallback (onchip_coalesced.cu)
        const int G = 32 / dsize(dtype);
        if (p.split_only || p.passes != 1 || p.k_pass[0] > 4 || (1 << p.k) < G || p.x_group != 0)
            return fail(TDS_ERR_UNSUPPORTED, "strided 2 needs one split pass with log2(32 / sizeof(T)) <= k_pass "
                                             "<= 4 and x_group 0");
        if (p.cluster != 1 || p.cr_levels != 0 || p.tl_levels != 0)
            return fail(TDS_ERR_UNSUPPORTED, "strided 2 needs cluster 1, cr_levels 0, tl_levels 0");
        if (n_sub >= (int64_t(1) << 31))
            return fail(TDS_ERR_UNSUPPORTED, "strided 2 needs n / 2^k < 2^31");
        if ((info.batch_stride * dsize(dtype)) % 16)
            return fail(TDS_ERR_UNSUPPORTED, "strided 2 needs batch_stride x sizeof(T) a multiple of 16 (it reads "
                                             "the TMA split's in-place output)");
        if (int64_t(G) * p.thomas_chains > 1024)
            return fail(TDS_ERR_INVALID_ARG, "strided 2 needs (32 / sizeof(T)) x thomas_chains <= 1024");
    } else if (p.strided != 0) {
        return fail(TDS_ERR_INVALID_ARG, "strided must be 0, 1 or 2");
    }
    if (p.x_group != 0) {  // fused x placement (onchip_pipe.cu, gpipe kernel)
        const int G = p.x_group, ds = dsize(dtype);
        if (G != 2 && G != 4 && G != 8) return fail(TDS_ERR_INVALID_ARG, "x_group must be 0, 2, 4 or 8");
        if (p.split_only) return fail(TDS_ERR_INVALID_ARG, "x_group needs an on-chip stage");
        if (p.k == 0 || p.k > 30 || (int64_t(1) << p.k) < G || n % (int64_t(1) << p.k) != 0)
            return fail(TDS_ERR_UNSUPPORTED, "x_group needs k >= log2(x_group) and 2^k dividing n");
        const int64_t L = n >> p.k, seg = L / G;
        if (p.cluster != 1 || p.tl_levels != 5 || R * ds != 64 || L != threads * R || L % G ||
            (L * ds) % 128 || (seg > 256 && seg % 256))
            return fail(TDS_ERR_UNSUPPORTED, "x_group needs cluster 1, tl_levels 5, 64 bytes of rows per thread, "
                                             "n / 2^k = threads x 2^c in whole 128-byte lines");
        if (G * ds < 16 || ((int64_t(1) << p.k) * ds) % 16 || (info.batch_stride * ds) % 16)
            return fail(TDS_ERR_UNSUPPORTED, "x_group needs 16-byte runs, 2^k and batch_stride in 16-byte units");
    }
    // --- derived fields
    info.params = p;
    info.n_sub = n_sub;
    info.num_subsystems = m * std::min<int64_t>(int64_t(1) << std::min(p.k, 62), n);
    info.onchip_threads = (int32_t)threads;
    info.subsys_per_cta = 1;
    const int64_t mc = chunk_m(p, m);  // systems per chunk
    info.chunks = (int32_t)cdiv(m, mc);
    info.launches = info.chunks * (p.passes + 1 + (p.k > 0 && p.x_group == 0 && p.strided == 0 ? 1 : 0));
    if (p.passes > 0) {
        int kk = 0;
        int64_t elems = 0;
        for (int i = 0; i < p.passes; ++i) {
            kk += p.k_pass[i];
            elems = std::max<int64_t>(elems, mc * (int64_t(1) << kk) * slot_rows(n, kk, dtype));
        }
        const int64_t E = round_up(elems, 64);
        info.slot_rows = slot_rows(n, p.k, dtype);
        // two buffers for multi-pass plans and for the coalesced variant's global-fallback ping-pong
        info.workspace_bytes = size_t((p.passes == 1 && !coalesced ? 1 : 2) * 3 * E * dsize(dtype));
        info.split_tile_eff = split_tile_eff(p, 0);
        info.split_segments = split_segments(mc, cdiv(n, info.split_tile_eff), p.theta);
    } else {
        info.slot_rows = 0;
        info.workspace_bytes = 0;
        info.split_segments = 0;
        info.split_tile_eff = 0;
    }
    info.onchip_form = p.split_only ? -1 : onchip_form_of(info);
    return TDS_OK;
}

static tds_status seed(tds_plan_info &info, const tds_device_props &props, tds_params &p) {
    const int32_t dtype = info.dtype;
    const int64_t n = info.n;
    int64_t target;
    int32_t T, theta, tile, g1threads, kpmax, g2cap, cmax;
    info.n_onchip_max = (int32_t)n_onchip_max(props, dtype);
    const int kp_paper = dtype == TDS_F32 ? 9 : 8;
    if (info.mode == TDS_PARAMS_DEFAULT) {
        target = 256;
        theta = 16;
        T = 32;               // reading R10
        tile = 1024;
        g1threads = 256;
        g2cap = 256;
    } else {
        target = info.n_onchip_max;                       // P:L704-705, Table II
        T = 2 * props.warp_size;
        theta = props.sm_count;
        tile = (int32_t)std::min<int64_t>(info.n_onchip_max, int64_t(r_max(dtype)) * kMaxOnchipThreadsWide);
        g1threads = 512;
        g2cap = props.max_threads_per_block / 2;
    }
    kpmax = std::min(kp_paper, kp_limit(props, dtype, tile));
    cmax = 1;  // clusters: TUNED only (tds_tune), the paper's processor is one SM
    info.n_sub_target = (int32_t)target;
    info.split_kp_max = kpmax;
    std::memset(&p, 0, sizeof(p));
    int k = 0;
    while (cdiv(n, int64_t(1) << k) > target) ++k;
    p.k = k;
    const int P = k > 0 ? (int)cdiv(k, kpmax) : 0;
    if (P > TDS_MAX_PASSES) return fail(TDS_ERR_UNSUPPORTED, "system needs more than 8 split passes");
    p.passes = P;
    for (int i = 0; i < P; ++i) p.k_pass[i] = k / P + (i < k % P ? 1 : 0);
    const int64_t n_sub = cdiv(n, int64_t(1) << k);
    // smallest cluster whose CTAs hold the subsystem, then the fewest rows per thread
    int C = 1;
    while (C < cmax && n_sub > int64_t(C) * r_max(dtype) * g2cap) C *= 2;
    int R = 1;
    while (cdiv(n_sub, int64_t(R) * C) > g2cap && R < r_max(dtype)) R *= 2;
    if (C > 1 && R < 8) R = 8;  // the cluster kernel keeps >= 8 rows per thread
    p.cluster = C;
    p.cr_levels = ilog2(R);
    // CR across threads until the leader's system has one row per thread: c2 = log2(C)
    p.tl_levels = ilog2(C);
    p.thomas_chains = (int32_t)std::min<int64_t>(T, pow2ceil(cdiv(n_sub, R) >> p.tl_levels));
    p.split_tile_rows = tile;
    p.split_threads = g1threads;
    p.theta = theta;
    // L2-resident chunking (chunk_systems) is a tuner dimension only: measured on
    // B200 it loses to one launch per kernel over the whole batch (profiles/).
    p.chunk_systems = 0;
    return TDS_OK;
}

static tds_status make_plan(tds_plan_t *out, const tds_device_props &props, int device, tds_dtype dtype,
                            int64_t n, int64_t m, int64_t batch_stride, tds_param_mode mode) {
    if (!out) return fail(TDS_ERR_INVALID_ARG, "out is NULL");
    *out = nullptr;
    if (dtype != TDS_F32 && dtype != TDS_F64) return fail(TDS_ERR_INVALID_ARG, "dtype");
    if (mode != TDS_PARAMS_DEFAULT && mode != TDS_PARAMS_STATIC)
        return fail(TDS_ERR_INVALID_ARG, "mode must be DEFAULT or STATIC (TUNED comes from tds_tune)");
    if (n < 1 || m < 1) return fail(TDS_ERR_INVALID_ARG, "n and m must be >= 1");
    if (batch_stride == 0) batch_stride = n;
    if (batch_stride < n) return fail(TDS_ERR_INVALID_ARG, "batch_stride < n");
    if (props.sm_count < 1 || props.warp_size < 1 || props.max_threads_per_block < 32 ||
        props.smem_optin_bytes < 4096)
        return fail(TDS_ERR_INVALID_ARG, "implausible device properties");
    tds_plan_st *pl = new (std::nothrow) tds_plan_st();
    if (!pl) return fail(TDS_ERR_NO_MEMORY, "host allocation");
    std::memset(&pl->info, 0, sizeof(pl->info));
    pl->props = props;
    pl->info.dtype = dtype;
    pl->info.mode = mode;
    pl->info.device = device;
    pl->info.n = n;
    pl->info.m = m;
    pl->info.batch_stride = batch_stride;
    tds_params p;
    tds_status st = seed(pl->info, props, p);
    if (st == TDS_OK) st = derive(pl->info, props, p);
    if (st != TDS_OK) {
        delete pl;
        return st;
    }
    *out = pl;
    clear_error();
    return TDS_OK;
}

}  // namespace tds

using namespace tds;

extern "C" {

tds_status tds_plan_from_props(tds_plan_t *out, const tds_device_props *props, tds_dtype dtype, int64_t n,
                               int64_t m, int64_t batch_stride, tds_param_mode mode) {
    if (!props) return fail(TDS_ERR_INVALID_ARG, "props is NULL");
    return make_plan(out, *props, -1, dtype, n, m, batch_stride, mode);
}

tds_status tds_plan(tds_plan_t *out, int device, tds_dtype dtype, int64_t n, int64_t m, int64_t batch_stride,
                    tds_param_mode mode) {
    tds_device_props props;
    tds_status st = tds_device_props_query(device, &props);
    if (st != TDS_OK) return st;
    return make_plan(out, props, device, dtype, n, m, batch_stride, mode);
}

tds_status tds_plan_info_get(const tds_plan_t plan, tds_plan_info *out) {
    if (!plan || !out) return fail(TDS_ERR_INVALID_ARG, "NULL argument");
    *out = plan->info;
    return TDS_OK;
}

tds_status tds_plan_set_params(tds_plan_t plan, const tds_params *params) {
    if (!plan || !params) return fail(TDS_ERR_INVALID_ARG, "NULL argument");
    tds_plan_info info = plan->info;
    tds_status st = derive(info, plan->props, *params);
    if (st != TDS_OK) return st;
    info.mode = TDS_PARAMS_TUNED;
    plan->info = info;
    clear_error();
    return TDS_OK;
}

tds_status tds_plan_permutation(const tds_plan_t plan, int64_t *perm, int64_t len) {
    if (!plan || !perm) return fail(TDS_ERR_INVALID_ARG, "NULL argument");
    const int64_t n = plan->info.n;
    if (len != n) return fail(TDS_ERR_INVALID_ARG, "len must equal n");
    const int k = plan->info.params.k;
    const int64_t step = int64_t(1) << std::min(k, 62);
    int64_t o = 0;
    for (int64_t r = 0; r < std::min(step, n); ++r)
        for (int64_t i = r; i < n; i += step) perm[o++] = i;
    return TDS_OK;
}

tds_status tds_plan_destroy(tds_plan_t plan) {
    delete plan;
    return TDS_OK;
}

tds_status tds_plan_tune_trials(const tds_plan_t plan, int32_t *trials) {
    if (!plan || !trials) return fail(TDS_ERR_INVALID_ARG, "NULL argument");
    *trials = plan->tune_trials;
    return TDS_OK;
}

const char *tds_status_string(tds_status s) {
    switch (s) {
        case TDS_OK: return "TDS_OK";
        case TDS_ERR_INVALID_ARG: return "TDS_ERR_INVALID_ARG: invalid argument";
        case TDS_ERR_UNSUPPORTED: return "TDS_ERR_UNSUPPORTED: unsupported configuration";
        case TDS_ERR_NO_MEMORY: return "TDS_ERR_NO_MEMORY: allocation failed";
        case TDS_ERR_WORKSPACE: return "TDS_ERR_WORKSPACE: workspace missing, too small or misaligned";
        case TDS_ERR_CUDA: return "TDS_ERR_CUDA: CUDA error";
        case TDS_ERR_TUNE: return "TDS_ERR_TUNE: tuning failed";
        case TDS_ERR_DEVICE_MISMATCH: return "TDS_ERR_DEVICE_MISMATCH: current device differs from the plan's";
    }
    return "unknown tds_status";
}

const char *tds_last_error(void) { return g_last_error.c_str(); }

int tds_version(void) { return TDS_VERSION; }

}  // extern "C"
