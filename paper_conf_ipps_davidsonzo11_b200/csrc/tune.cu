// tune.cu -- the self-tuner (§IV-D).
//
// The paper's two pruning ideas, applied to the B200 plan parameters:
//  (1) decouple parameters that do not interact: the stage 3->4
//      switch (on-chip: CR levels c, Thomas chains T, cluster, form) depends
//      only on the subsystem size; the stage 2->3 switch (split levels k) is
//      compared "vs. two times the number of systems at half the size"
//      re-tuning the 3->4 switch for each; the stage 1->2
//      threshold theta and the split geometry (tile, CTA size, pass schedule)
//      are tuned last with the others fixed.  Trials therefore
//      add up instead of multiplying (the paper's 16 + 32 vs 16 x 32).
//  (2) start every search at the machine-query seed (the STATIC plan) and hill
//      climb to a local minimum ("a local minimum in a hyperbolic search
//      space").
// Results are saved to a cache file for future runs.
// Ties: candidates within 2% of the incumbent do not replace it; neighbours
// are visited in a fixed order (decrease before increase).
//
// The search is written against a cost function (median time of one solve
// with the candidate's parameters): tds_tune times real solves on the device;
// tds_tune_search (test-only) takes the cost from the caller, so the search
// itself is tested on the CPU (tests/test_tuner.py).
#include <algorithm>
#include <chrono>
#include <cmath>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <fstream>
#include <functional>
#include <sstream>
#include <string>
#include <vector>

#include "common.cuh"
#include "pipe.cuh"

namespace tds {

constexpr double kRejected = 1e30;  // cost of a candidate the planner or the kernels refuse
constexpr uint64_t kTuneSeed = 0x74756e65ull;  // "tune": trial systems, G4 generator, margin 1

using CostFn = std::function<double(const tds_params &)>;

struct Search {
    const tds_plan_st *plan;
    CostFn cost;        // median ms of one solve; >= kRejected: refused; NaN: fatal (abort)
    int trials = 0;
    bool fatal = false;
    std::chrono::steady_clock::time_point t_start;
    double budget_s = 50.0;
};

static bool out_of_time(const Search &S) {
    return S.fatal ||
           std::chrono::duration<double>(std::chrono::steady_clock::now() - S.t_start).count() > S.budget_s;
}

// One trial: the planner's validation first (a refused candidate costs no trial).
static double eval(Search &S, const tds_params &p) {
    if (S.fatal) return kRejected;
    tds_plan_info info = S.plan->info;
    if (derive(info, S.plan->props, p) != TDS_OK) return kRejected;
    ++S.trials;
    const double t = S.cost(p);
    if (std::isnan(t)) {
        S.fatal = true;
        return kRejected;
    }
    return t;
}

static bool better(double t_new, double t_best) { return t_new < 0.98 * t_best; }

static int ilog2i(int64_t v) {
    int l = 0;
    while ((int64_t(1) << (l + 1)) <= v) ++l;
    return l;
}

static int64_t cta_threads(const tds_plan_info &I, const tds_params &p) {
    const int64_t n_sub = cdiv(I.n, int64_t(1) << p.k);
    return std::max<int64_t>(32, round_up(cdiv(n_sub, (int64_t(1) << p.cr_levels) * p.cluster), 32));
}

// The warp form (TDS_FORM_WARP_CR) solves the per-warp top rows by shuffle
// PCR / CR: the Thomas switch T is not a parameter of that form, and is kept
// at its canonical value 1.
static bool warp_form(const tds_plan_st *plan, const tds_params &p) {
    tds_plan_info info = plan->info;
    return derive(info, plan->props, p) == TDS_OK && info.onchip_form == TDS_FORM_WARP_CR;
}

// Keep (c, C, c2, T) consistent: clusters need >= 8 rows per thread, 2^c2
// divides the CTA size, T <= the leader's system Z = C * threads / 2^c2.
static void clamp_onchip(const tds_plan_st *plan, tds_params &p) {
    const tds_plan_info &I = plan->info;
    if (p.cluster > 1 && p.cr_levels < 3) p.cr_levels = 3;
    const int64_t thr = cta_threads(I, p);
    while (p.tl_levels > 0 && (thr % (int64_t(1) << p.tl_levels))) --p.tl_levels;
    const int64_t Z = (thr >> p.tl_levels) * p.cluster;
    while (p.thomas_chains > Z && p.thomas_chains > 1) p.thomas_chains /= 2;
    if (warp_form(plan, p)) p.thomas_chains = 1;
}

static void fit_onchip(const tds_plan_st *plan, tds_params &p);

// Stage 3->4: hill climb over (form, c, T, c2, cluster, x placement, load variant) for the current k.
static void tune_onchip(Search &S, tds_params &best, double &t_best) {
    const tds_plan_info &I = S.plan->info;
    bool improved = true;
    while (improved && !out_of_time(S)) {
        improved = false;
        tds_params cand[20];
        int nc = 0;
        // the warp-level form (CR across all 32 lanes, shuffles only) is a
        // different kernel path, not a neighbour of tl_levels = 4: try it directly
        if (best.cluster == 1 && best.tl_levels != 5) { cand[nc] = best; cand[nc++].tl_levels = 5; }
        // ... and for k = 0 on one CTA or a cluster of <= 8, the persistent kernel's shape (64 bytes of rows per thread)
        if (best.k == 0 && best.cluster <= 8 && !(best.tl_levels == 5 && (1 << best.cr_levels) == r_max(I.dtype))) {
            cand[nc] = best;
            cand[nc].tl_levels = 5;
            cand[nc++].cr_levels = ilog2i(r_max(I.dtype));
        }
        const bool wf = warp_form(S.plan, best);
        if (!wf) {  // T is a dimension of the shared-memory PCR-Thomas form only
            if (best.thomas_chains > 1) { cand[nc] = best; cand[nc++].thomas_chains /= 2; }
            cand[nc] = best; cand[nc++].thomas_chains *= 2;
        }
        if (best.tl_levels > 0) {
            cand[nc] = best; cand[nc].tl_levels -= 1;
            if (wf) cand[nc].thomas_chains = 64;  // leaving the warp form: the static T
            ++nc;
        }
        if (best.tl_levels < 10) { cand[nc] = best; cand[nc++].tl_levels += 1; }
        if (best.cr_levels > 0) { cand[nc] = best; cand[nc++].cr_levels -= 1; }
        if ((1 << (best.cr_levels + 1)) <= r_max(I.dtype)) { cand[nc] = best; cand[nc++].cr_levels += 1; }
        if (best.cluster > 1) { cand[nc] = best; cand[nc].cluster /= 2; cand[nc++].tl_levels -= best.tl_levels > 0; }
        if (best.cluster < 16 && S.plan->props.cc_major >= 9) {
            cand[nc] = best; cand[nc].cluster *= 2; cand[nc++].tl_levels += 1;
        }
        // fused x placement (k > 0, warp form, 64 bytes of rows per thread): off, or
        // clusters of G CTAs on adjacent residue classes; G halves / doubles
        if (best.k > 0 && best.cluster == 1 && best.tl_levels == 5 &&
            (1 << best.cr_levels) * dsize(I.dtype) == 64) {
            const int gmin = 16 / dsize(I.dtype);
            if (best.x_group == 0) {
                cand[nc] = best; cand[nc++].x_group = 8;
                cand[nc] = best; cand[nc++].x_group = 4;
            } else {
                cand[nc] = best; cand[nc++].x_group = 0;
                if (best.x_group / 2 >= gmin) { cand[nc] = best; cand[nc++].x_group = best.x_group / 2; }
                if (best.x_group < 8) { cand[nc] = best; cand[nc++].x_group = best.x_group * 2; }
            }
        }
        // the paper's strided base-kernel variant (one pass of <= 4 levels): on / off
        if (best.k > 0 && best.passes == 1 && best.k_pass[0] <= 4 && best.cluster == 1 && best.tl_levels == 5 &&
            best.x_group == 0 && (1 << best.cr_levels) * dsize(I.dtype) == 64) {
            cand[nc] = best;
            cand[nc++].strided = best.strided ? 0 : 1;
        }
        // the paper's coalesced base-kernel variant with global fallback (strided = 2):
        // on from any form of a one-pass plan of log2(G) <= k <= 4 levels (the paper's
        // T = 64 to start), off back to the fitted default form
        if (best.k > 0 && best.passes == 1 && best.k_pass[0] <= 4 && (1 << best.k) >= 32 / dsize(I.dtype) &&
            best.x_group == 0) {
            cand[nc] = best;
            if (best.strided == 2) {
                fit_onchip(S.plan, cand[nc]);
            } else {
                cand[nc].strided = 2;
                cand[nc].cr_levels = 0;
                cand[nc].tl_levels = 0;
                cand[nc].cluster = 1;
                cand[nc].thomas_chains = std::min(64, 1024 / (32 / dsize(I.dtype)));
            }
            ++nc;
        }
        for (int i = 0; i < nc; ++i) {
            clamp_onchip(S.plan, cand[i]);
            if (std::memcmp(&cand[i], &best, sizeof(best)) == 0) continue;
            const double t = eval(S, cand[i]);
            if (better(t, t_best)) {
                best = cand[i];
                t_best = t;
                improved = true;
                break;
            }
        }
    }
}

static void schedule_passes(tds_params &p, int kpmax) {
    std::memset(p.k_pass, 0, sizeof(p.k_pass));
    p.passes = p.k > 0 ? int((p.k + kpmax - 1) / kpmax) : 0;
    for (int i = 0; i < p.passes; ++i) p.k_pass[i] = p.k / p.passes + (i < p.k % p.passes ? 1 : 0);
}

// Make (c, C, T) valid for a new k: the smallest cluster (clusters cost barrier
// latency) and the most rows per thread that fit the on-chip kernel.
static void fit_onchip(const tds_plan_st *plan, tds_params &p) {
    const tds_plan_info &I = plan->info;
    const tds_device_props &props = plan->props;
    const int64_t n_sub = cdiv(I.n, int64_t(1) << p.k);
    auto cap = [&](int c) { return onchip_max_threads(1 << c, dsize(I.dtype)); };
    auto thr = [&](const tds_params &q) {
        return round_up(cdiv(n_sub, (int64_t(1) << q.cr_levels) * q.cluster), 32);
    };
    p.cluster = 1;
    p.cr_levels = ilog2i(r_max(I.dtype));
    while (thr(p) > cap(p.cr_levels) && p.cluster < 16 && props.cc_major >= 9) p.cluster *= 2;
    p.tl_levels = ilog2i(p.cluster);
    if (p.thomas_chains < 1) p.thomas_chains = 64;
    p.x_group = 0;  // re-enabled by tune_onchip where the new subsystem size allows it
    p.strided = 0;
    clamp_onchip(plan, p);
}

// The whole decoupled search from `seed`; returns the best parameters and their cost.
static tds_params search(Search &S, const tds_params &seed, double &t_best) {
    const tds_plan_info &I = S.plan->info;
    tds_params best = seed;
    t_best = eval(S, best);
    if (t_best >= kRejected) return best;
    // (1) stage 3->4 switch at the seed's subsystem size
    tune_onchip(S, best, t_best);
    // (2) stage 2->3 switch: 2x the systems at half the size (k+1), or the
    // reverse.  For each k both pass schedules are tried -- register split
    // passes (k_p <= 4), the persistent TMA split kernel's limit (k_p <= 8)
    // and the seed's k_p limit -- with the smallest cluster that holds the
    // subsystem; the walk up tolerates two non-improving steps (splitting and
    // on-chip costs trade off unevenly), the walk down goes on while the
    // subsystems fit on chip (k = 0, no split pass at all, is a regime of its
    // own: a local minimum the climb must not miss -- config 4 from its static
    // seed k = 1).
    for (int dir : {+1, -1}) {
        tds_params walk = best;
        int misses = 0;
        while ((dir < 0 || misses < 3) && !out_of_time(S)) {
            tds_params base = walk;
            base.k += dir;
            if (base.k < 0 || base.k > 30 || (int64_t(1) << base.k) > 2 * I.n) break;
            double t_step = kRejected;
            tds_params step_best = base;
            const int spk = std::max(I.split_kp_max, 1);
            int kps[3] = {std::min(kRegSplitMaxKp, spk), std::min(kPipeSplitMaxKp, spk), spk};
            for (int ki = 0; ki < 3; ++ki) {
                const int kpmax = kps[ki];
                if (ki > 0 && kpmax == kps[ki - 1]) continue;
                tds_params cand = base;
                schedule_passes(cand, kpmax);
                fit_onchip(S.plan, cand);
                double t = eval(S, cand);
                if (t >= kRejected) continue;
                tune_onchip(S, cand, t);
                if (t < t_step) {
                    t_step = t;
                    step_best = cand;
                }
            }
            if (t_step >= kRejected) break;
            walk = step_best;
            if (better(t_step, t_best)) {
                best = step_best;
                t_best = t_step;
                misses = 0;
            } else {
                ++misses;
            }
        }
    }
    // (3) stage 1->2 threshold theta and split geometry, one dimension at a time
    if (best.passes > 0) {
        bool improved = true;
        while (improved && !out_of_time(S)) {
            improved = false;
            std::vector<tds_params> cands;
            tds_params q = best;
            if (best.theta > 1) { q = best; q.theta = std::max(1, best.theta / 2); cands.push_back(q); }
            q = best; q.theta = best.theta * 2; cands.push_back(q);
            q = best; q.split_tile_rows = best.split_tile_rows / 2; cands.push_back(q);
            q = best; q.split_tile_rows = best.split_tile_rows * 2; cands.push_back(q);
            q = best; q.split_threads = best.split_threads / 2; cands.push_back(q);
            q = best; q.split_threads = best.split_threads * 2; cands.push_back(q);
            {  // L2-resident chunks of systems: halve / double the chunk (0 = whole batch)
                const int64_t mc = chunk_m(best, I.m);
                if (mc > 1) { q = best; q.chunk_systems = (int32_t)cdiv(mc, 2); cands.push_back(q); }
                if (mc < I.m) { q = best; q.chunk_systems = (int32_t)std::min<int64_t>(2 * mc, I.m); cands.push_back(q); }
            }
            if (best.passes < TDS_MAX_PASSES && best.k > best.passes) {
                // one more (shallower) pass: less halo per pass, one more HBM round trip
                q = best;
                schedule_passes(q, std::max(1, (best.k + best.passes) / (best.passes + 1)));
                cands.push_back(q);
            }
            if (best.passes > 1) {
                // one fewer (deeper) pass, and the same levels in reverse order
                q = best;
                schedule_passes(q, (best.k + best.passes - 2) / (best.passes - 1));
                if (q.passes < best.passes) cands.push_back(q);
                q = best;
                std::reverse(q.k_pass, q.k_pass + q.passes);
                cands.push_back(q);
            }
            for (auto &cnd : cands) {
                const double t = eval(S, cnd);
                if (better(t, t_best)) {
                    best = cnd;
                    t_best = t;
                    improved = true;
                    break;
                }
            }
        }
    }
    return best;
}

static std::string cache_key(const tds_plan_st *plan) {
    cudaDeviceProp prop;
    std::string name = "unknown";
    if (plan->info.device >= 0 && cudaGetDeviceProperties(&prop, plan->info.device) == cudaSuccess) name = prop.name;
    for (auto &ch : name)
        if (ch == ' ' || ch == '\t') ch = '_';
    std::ostringstream o;
    o << name << "|sm" << plan->props.sm_count << "|smem" << plan->props.smem_optin_bytes << "|"
      << (plan->info.dtype == TDS_F64 ? "f64" : "f32") << "|n" << plan->info.n << "|m" << plan->info.m << "|s"
      << plan->info.batch_stride;
    return o.str();
}

static std::string params_str(const tds_params &p) {
    std::ostringstream o;
    o << p.k << " " << p.passes;
    for (int i = 0; i < TDS_MAX_PASSES; ++i) o << " " << p.k_pass[i];
    o << " " << p.cr_levels << " " << p.thomas_chains << " " << p.cluster << " " << p.tl_levels << " "
      << p.split_tile_rows << " " << p.split_threads << " " << p.theta << " " << p.chunk_systems << " "
      << p.x_group << " " << p.strided;
    return o.str();
}

static bool cache_lookup(const std::string &path, const std::string &key, tds_params &p) {
    std::ifstream f(path);
    if (!f) return false;
    std::string line;
    bool found = false;
    while (std::getline(f, line)) {  // last matching line wins
        std::istringstream is(line);
        std::string k;
        if (!(is >> k) || k != key) continue;
        tds_params q{};
        is >> q.k >> q.passes;
        for (int i = 0; i < TDS_MAX_PASSES; ++i) is >> q.k_pass[i];
        is >> q.cr_levels >> q.thomas_chains >> q.cluster >> q.tl_levels >> q.split_tile_rows >> q.split_threads >>
            q.theta >> q.chunk_systems;
        if (is) {
            if (!(is >> q.x_group)) q.x_group = 0;  // lines written before x_group existed
            if (!(is >> q.strided)) q.strided = 0;
            p = q;
            found = true;
        }
    }
    return found;
}

static std::string cache_path_of(const char *cache_path) {
    if (cache_path) return cache_path;
    const char *e = std::getenv("TDS_TUNE_CACHE");
    return e ? e : "";
}

// Apply a cache hit (true) or report a miss (false).
static bool apply_cached(tds_plan_st *plan, const std::string &path, const std::string &key) {
    tds_params p{};
    if (path.empty() || !cache_lookup(path, key, p)) return false;
    tds_plan_info info = plan->info;
    if (derive(info, plan->props, p) != TDS_OK) return false;
    info.mode = TDS_PARAMS_TUNED;
    info.tuned = 1;
    plan->info = info;
    plan->tune_trials = 0;
    return true;
}

// Install the search result (only a plan derive accepts; the cache line only then).
static tds_status commit(tds_plan_st *plan, const tds_params &best, int trials, const std::string &path,
                         const std::string &key) {
    tds_plan_info info = plan->info;
    if (derive(info, plan->props, best) != TDS_OK) return fail(TDS_ERR_TUNE, "the tuned parameters were refused");
    info.mode = TDS_PARAMS_TUNED;
    info.tuned = 1;
    plan->info = info;
    plan->tune_trials = trials;
    if (!path.empty()) {
        std::ofstream f(path, std::ios::app);
        if (f) f << key << " " << params_str(best) << "\n";
    }
    return TDS_OK;
}

// ---------------------------------------------------------------- device trials

struct TuneCtx {
    tds_plan_st *plan;
    cudaStream_t st;
    cudaStream_t cap = nullptr;  // private stream for graph-timed trials (created on first use)
    void *a = nullptr, *b = nullptr, *c = nullptr, *d = nullptr, *x = nullptr, *ws = nullptr;
    size_t ws_bytes = 0;
    int reps = 7;
};

static bool ensure_ws(TuneCtx &C, size_t need) {
    if (need <= C.ws_bytes) return true;
    if (C.ws) cudaFree(C.ws);
    C.ws = nullptr;
    C.ws_bytes = 0;
    if (cudaMalloc(&C.ws, need) != cudaSuccess) {
        cudaGetLastError();
        return false;
    }
    C.ws_bytes = need;
    return true;
}

// Launch-bound solves (a back-to-back eager solve under kGraphTrialMs) are
// timed as CUDA-graph replays of `inner` captured solves: eager launches of a
// few-microsecond solve measure the host's launch rate (~7 us per solve for
// every candidate of config 1), not the kernels, so the climb could not tell
// the plans apart (gpurun_out/r02aj: 3.0 vs 4.2 us per solve under graph
// replay for two plans that both time 7.0 us eagerly).  Returns the median ms
// per solve, kRejected if the capture is refused, NaN on a device fault.
constexpr float kGraphTrialMs = 0.03f;

static double graph_trial(TuneCtx &C, tds_plan_st &tmp, int inner) {
    if (!C.cap && cudaStreamCreateWithFlags(&C.cap, cudaStreamNonBlocking) != cudaSuccess) {
        cudaGetLastError();
        C.cap = nullptr;
        return kRejected;
    }
    if (cudaStreamSynchronize(C.st) != cudaSuccess) return NAN;  // trial data and workspace are ready
    cudaGraph_t g = nullptr;
    cudaGraphExec_t ge = nullptr;
    bool ok = cudaStreamBeginCapture(C.cap, cudaStreamCaptureModeThreadLocal) == cudaSuccess;
    for (int i = 0; i < inner && ok; ++i)
        ok = tds_solve_batched(&tmp, C.a, C.b, C.c, C.d, C.x, C.ws, C.ws_bytes, C.cap) == TDS_OK;
    const cudaError_t ec = cudaStreamEndCapture(C.cap, &g);
    ok = ok && ec == cudaSuccess && g && cudaGraphInstantiate(&ge, g, 0) == cudaSuccess;
    if (!ok) {
        if (ge) cudaGraphExecDestroy(ge);
        if (g) cudaGraphDestroy(g);
        cudaGetLastError();
        return kRejected;
    }
    cudaEvent_t e0, e1;
    if (cudaEventCreate(&e0) != cudaSuccess || cudaEventCreate(&e1) != cudaSuccess) return NAN;
    std::vector<float> ms;
    bool fault = false;
    for (int r = 0; r < C.reps + 1 && !fault; ++r) {
        cudaEventRecord(e0, C.cap);
        cudaGraphLaunch(ge, C.cap);
        cudaEventRecord(e1, C.cap);
        if (cudaEventSynchronize(e1) != cudaSuccess) fault = true;
        float t = 0;
        cudaEventElapsedTime(&t, e0, e1);
        if (r >= 1) ms.push_back(t / float(inner));
    }
    cudaEventDestroy(e0);
    cudaEventDestroy(e1);
    cudaGraphExecDestroy(ge);
    cudaGraphDestroy(g);
    if (fault || cudaStreamSynchronize(C.cap) != cudaSuccess) return NAN;
    std::sort(ms.begin(), ms.end());
    return ms[ms.size() / 2];
}

// Median time (ms) of the full solve with parameters p (already validated),
// measured as bench.py runs it: `inner` solves back to back between two
// events (inner chosen so one sample spans >= ~0.4 ms); launch-bound solves
// by graph replay (graph_trial); kRejected if the solve refuses to launch;
// NaN on a device fault (sticky: the search stops).
static double trial(TuneCtx &C, const tds_params &p) {
    tds_plan_st tmp = *C.plan;
    if (derive(tmp.info, tmp.props, p) != TDS_OK) return kRejected;
    if (!ensure_ws(C, tmp.info.workspace_bytes)) return kRejected;
    cudaEvent_t e0, e1;
    if (cudaEventCreate(&e0) != cudaSuccess || cudaEventCreate(&e1) != cudaSuccess) return NAN;
    std::vector<float> ms;
    bool launched = true, fault = false;
    int inner = 1;
    for (int r = 0; r < C.reps + 2 && launched && !fault; ++r) {
        cudaEventRecord(e0, C.st);
        for (int i = 0; i < inner && launched; ++i)
            launched = tds_solve_batched(&tmp, C.a, C.b, C.c, C.d, C.x, C.ws, C.ws_bytes, C.st) == TDS_OK;
        cudaEventRecord(e1, C.st);
        if (cudaEventSynchronize(e1) != cudaSuccess) fault = true;
        float t = 0;
        cudaEventElapsedTime(&t, e0, e1);
        if (r == 0 && inner == 1 && t > 0) inner = std::max(1, std::min(64, int(0.4f / t + 0.999f)));
        if (r >= 2) ms.push_back(t / float(inner));
    }
    cudaEventDestroy(e0);
    cudaEventDestroy(e1);
    if (fault || cudaStreamSynchronize(C.st) != cudaSuccess) return NAN;
    if (!launched) {
        cudaGetLastError();  // a refused launch configuration is not sticky
        return kRejected;
    }
    std::sort(ms.begin(), ms.end());
    const double eager = ms[ms.size() / 2];
    if (eager < kGraphTrialMs) {
        const double gt = graph_trial(C, tmp, std::max(inner, 16));
        if (std::isnan(gt)) return gt;
        if (gt < kRejected) return gt;
    }
    return eager;
}

// max |x - y| and max |y| over the rows of m systems (padding excluded);
// non-negative doubles compare as their bit patterns
template <typename T>
__global__ void compare_kernel(const T *x, const T *y, int64_t n, int64_t m, int64_t stride,
                               unsigned long long *out) {
    double dmax = 0, ymax = 0;
    for (int64_t e = blockIdx.x * int64_t(blockDim.x) + threadIdx.x; e < n * m; e += int64_t(gridDim.x) * blockDim.x) {
        const int64_t s = e / n, i = s * stride + (e - s * n);
        const double dx = double(x[i]), dy = double(y[i]);
        const double d = fabs(dx - dy);
        dmax = d != d ? INFINITY : fmax(dmax, d);
        ymax = fmax(ymax, fabs(dy));
    }
    atomicMax(out, (unsigned long long)__double_as_longlong(dmax));
    atomicMax(out + 1, (unsigned long long)__double_as_longlong(ymax));
}

// The chosen plan must give the seed plan's answer (both are solves of the
// same systems): relative difference <= 2e-4 (fp32) / 1e-9 (fp64).
static tds_status validate(TuneCtx &C, const tds_params &seed, const tds_params &best) {
    const tds_plan_info &I = C.plan->info;
    const int64_t elems = (I.m - 1) * I.batch_stride + I.n;
    const size_t es = size_t(dsize(I.dtype));
    void *xs = nullptr;
    unsigned long long *red = nullptr;
    tds_status st = TDS_OK;
    if (cudaMalloc(&xs, size_t(elems) * es) != cudaSuccess || cudaMalloc(&red, 16) != cudaSuccess) {
        cudaGetLastError();
        st = fail(TDS_ERR_NO_MEMORY, "tuner validation buffers");
    }
    for (int which = 0; which < 2 && st == TDS_OK; ++which) {
        tds_plan_st tmp = *C.plan;
        if (derive(tmp.info, tmp.props, which == 0 ? seed : best) != TDS_OK || !ensure_ws(C, tmp.info.workspace_bytes) ||
            tds_solve_batched(&tmp, C.a, C.b, C.c, C.d, which == 0 ? xs : C.x, C.ws, C.ws_bytes, C.st) != TDS_OK)
            st = fail(TDS_ERR_TUNE, "validation solve failed");
    }
    double h[2] = {0, 0};
    if (st == TDS_OK) {
        cudaMemsetAsync(red, 0, 16, C.st);
        const int blocks = (int)std::min<int64_t>(4 * sm_count_current(), cdiv(I.n * I.m, 256));
        if (I.dtype == TDS_F32)
            compare_kernel<float><<<blocks, 256, 0, C.st>>>((const float *)C.x, (const float *)xs, I.n, I.m,
                                                            I.batch_stride, red);
        else
            compare_kernel<double><<<blocks, 256, 0, C.st>>>((const double *)C.x, (const double *)xs, I.n, I.m,
                                                             I.batch_stride, red);
        unsigned long long hb[2];
        if (cudaMemcpyAsync(hb, red, 16, cudaMemcpyDeviceToHost, C.st) != cudaSuccess ||
            cudaStreamSynchronize(C.st) != cudaSuccess) {
            st = fail(TDS_ERR_TUNE, "device fault during validation");
        } else {
            std::memcpy(h, hb, 16);
        }
    }
    if (st == TDS_OK) {
        const double tol = I.dtype == TDS_F32 ? 2e-4 : 1e-9;
        if (!(h[0] <= tol * std::max(h[1], 1e-30)))
            st = fail(TDS_ERR_TUNE, "the tuned plan's x differs from the seed plan's (rel " +
                                        std::to_string(h[0] / std::max(h[1], 1e-30)) + ")");
    }
    if (xs) cudaFree(xs);
    if (red) cudaFree(red);
    return st;
}

}  // namespace tds

using namespace tds;

extern "C" tds_status tds_tune(tds_plan_t plan, void *cuda_stream, const char *cache_path) {
    if (!plan) return fail(TDS_ERR_INVALID_ARG, "plan is NULL");
    int dev = -1;
    if (cudaGetDevice(&dev) != cudaSuccess || plan->info.device < 0 || dev != plan->info.device)
        return fail(TDS_ERR_DEVICE_MISMATCH, "tds_tune must run on the plan's device");
    const std::string path = cache_path_of(cache_path);
    const std::string key = cache_key(plan);
    if (apply_cached(plan, path, key)) {
        clear_error();
        return TDS_OK;
    }
    TuneCtx C;
    C.plan = plan;
    C.st = static_cast<cudaStream_t>(cuda_stream);
    const tds_plan_info &I = plan->info;
    const size_t es = size_t(dsize(I.dtype));
    const size_t bytes = size_t((I.m - 1) * I.batch_stride + I.n) * es;
    void **bufs[5] = {&C.a, &C.b, &C.c, &C.d, &C.x};
    for (auto p : bufs) {
        if (cudaMalloc(p, bytes) != cudaSuccess) {
            cudaGetLastError();
            for (auto q : bufs)
                if (*q) cudaFree(*q);
            return fail(TDS_ERR_NO_MEMORY, "tuner trial buffers");
        }
    }
    // trial systems: the seeded diagonally dominant family (G4 generator, gen.cu)
    cudaError_t ge = I.dtype == TDS_F32
                         ? launch_generate<float>((float *)C.a, (float *)C.b, (float *)C.c, (float *)C.d, I.n, I.m,
                                                  I.batch_stride, kTuneSeed, 0, 1.0, C.st)
                         : launch_generate<double>((double *)C.a, (double *)C.b, (double *)C.c, (double *)C.d, I.n,
                                                   I.m, I.batch_stride, kTuneSeed, 0, 1.0, C.st);
    if (I.n * I.m < (1 << 20)) C.reps = 15;

    Search S;
    S.plan = plan;
    S.t_start = std::chrono::steady_clock::now();
    S.cost = [&](const tds_params &p) { return trial(C, p); };
    tds_status result = TDS_OK;
    const tds_params seed = I.params;
    double t_best = kRejected;
    tds_params best = seed;
    if (ge != cudaSuccess) {
        result = fail(TDS_ERR_CUDA, std::string("trial data: ") + cudaGetErrorString(ge));
    } else {
        best = search(S, seed, t_best);
        if (S.fatal)
            result = fail(TDS_ERR_TUNE, "device fault during a trial (sticky error): tuning aborted");
        else if (t_best >= kRejected)
            result = fail(TDS_ERR_TUNE, "the seed plan failed to run");
        else
            result = validate(C, seed, best);
    }
    const int trials = S.trials;
    if (result == TDS_OK) result = commit(plan, best, trials, path, key);
    cudaStreamSynchronize(C.st);
    if (C.cap) cudaStreamDestroy(C.cap);
    for (auto p : bufs) cudaFree(*p);
    if (C.ws) cudaFree(C.ws);
    if (result == TDS_OK) clear_error();
    return result;
}

// Test-only: the same search with the cost taken from the caller (no device
// work; a plan from tds_plan_from_props works).  cost(params, user) returns
// the "median ms" of one solve with those parameters (>= 1e30: refused, NaN:
// abort).  The cache is read and written exactly as tds_tune does.
extern "C" tds_status tds_tune_search(tds_plan_t plan, double (*cost)(const tds_params *, void *), void *user,
                                      const char *cache_path) {
    if (!plan || !cost) return fail(TDS_ERR_INVALID_ARG, "NULL argument");
    const std::string path = cache_path_of(cache_path);
    const std::string key = cache_key(plan);
    if (apply_cached(plan, path, key)) {
        clear_error();
        return TDS_OK;
    }
    Search S;
    S.plan = plan;
    S.t_start = std::chrono::steady_clock::now();
    S.budget_s = 1e9;  // deterministic: no wall-clock cut-off
    S.cost = [&](const tds_params &p) { return cost(&p, user); };
    double t_best = kRejected;
    const tds_params best = search(S, plan->info.params, t_best);
    if (S.fatal) return fail(TDS_ERR_TUNE, "the cost function aborted the search");
    if (t_best >= kRejected) return fail(TDS_ERR_TUNE, "the seed plan was refused");
    const tds_status st = commit(plan, best, S.trials, path, key);
    if (st == TDS_OK) clear_error();
    return st;
}
