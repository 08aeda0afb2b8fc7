// Internal (non-ABI) declarations shared by the libtds translation units.
#pragma once
#include <string>

#include "../../include/tds.h"

struct tds_plan_st {
    tds_plan_info info;
    tds_device_props props;
    int32_t tune_trials = 0;
};

namespace tds {

// Kernel limits the planner validates against.
constexpr int kSplitQMax = 24;        // rows per thread held in registers by the split pass
constexpr int kSmemReserve = 1024;    // per-CTA shared memory reserved by the runtime
constexpr int kMaxOnchipThreads = 1024;     // on-chip CTA size while R rows take <= 32 bytes per array
constexpr int kMaxOnchipThreadsWide = 512;  // ... and with 64 bytes (register budget)
constexpr int kMaxSplitThreads = 512;
constexpr int kRegSplitMaxKp = 4;       // split passes with k_p <= 4 use the register kernel
constexpr int kPipeSplitMaxKp = 8;      // ... up to 8 with 16-byte aligned rows (persistent TMA kernel)
constexpr int kRegSplitRows = 16;       // ... 16 rows per thread
constexpr int kRegSplitThreads = 256;   // ... 256 threads per CTA

inline int dsize(int32_t dtype) { return dtype == TDS_F64 ? 8 : 4; }
inline int r_max(int32_t dtype) { return dtype == TDS_F64 ? 8 : 16; }
inline int64_t cdiv(int64_t a, int64_t b) { return (a + b - 1) / b; }
inline int64_t round_up(int64_t a, int64_t b) { return cdiv(a, b) * b; }
inline int onchip_max_threads(int R, int ds) { return R * ds >= 64 ? kMaxOnchipThreadsWide : kMaxOnchipThreads; }

// Thread-local error detail (tds_last_error).
tds_status fail(tds_status st, const std::string &msg);
void clear_error();

// Planner helpers (plan.cpp).
int64_t slot_rows(int64_t n, int kk, int32_t dtype);
int32_t split_segments(int64_t m_in, int64_t tiles, int32_t theta);
size_t split_smem_bytes(int32_t dtype, int32_t tile, int kp);
size_t onchip_smem_bytes(int32_t dtype, int32_t threads, int32_t cluster, int32_t tl_levels);
int32_t split_tile_eff(const tds_params &p, int pass);
int64_t chunk_m(const tds_params &p, int64_t m);
int32_t static_cluster(const tds_device_props &p);
tds_status derive(tds_plan_info &info, const tds_device_props &props, const tds_params &p);
// The on-chip form the dispatch selects (api.cu solve_impl) for 16-byte aligned arrays.
int32_t onchip_form_of(const tds_plan_info &I);
// The coalesced base-kernel variant (strided = 2, onchip_coalesced.cu): rows per
// subsystem held in shared memory, and the CTA size.
int32_t coalesced_rows_in_smem(int32_t dtype, int64_t L, int64_t smem_budget);
int32_t coalesced_threads(int32_t dtype, int64_t L, int32_t thomas_chains);

}  // namespace tds
