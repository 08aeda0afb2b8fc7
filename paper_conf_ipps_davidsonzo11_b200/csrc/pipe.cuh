// pipe.cuh -- TMA bulk-copy / mbarrier helpers and conflict-free shared-memory
// row loads shared by the persistent (pipelined) kernels.
#pragma once
#include <cuda.h>

#include <map>
#include <mutex>
#include <tuple>
#include <utility>

#include "common.cuh"

namespace tds {

// Programmatic dependent launch: the persistent kernels are launched with
// cudaLaunchAttributeProgrammaticStreamSerialization, so their CTAs can be
// scheduled (and set up shared memory / mbarriers) while the previous kernel
// on the stream drains; every thread waits here for that kernel's completion
// and memory before its first global-memory access.  A no-op for a normal launch.
__device__ __forceinline__ void pdl_wait() { asm volatile("griddepcontrol.wait;" ::: "memory"); }
// Experiment switch (-DTDS_PDL_TRIGGER=1): a CTA that starts its LAST work item
// lets the next kernel on the stream launch (its CTAs take the SMs this grid's
// finished CTAs free; they still wait in pdl_wait for this grid's completion).
#ifndef TDS_PDL_TRIGGER
#define TDS_PDL_TRIGGER 0
#endif
__device__ __forceinline__ void pdl_trigger_if_last(bool last) {
    if (TDS_PDL_TRIGGER && last) asm volatile("griddepcontrol.launch_dependents;" ::: "memory");
}

// Host: per-launch setup that does not change between solves -- the dynamic
// shared-memory opt-in, the non-portable cluster opt-in and the occupancy
// query -- done once per (kernel, device, block, smem, cluster) and cached
// (they cost several microseconds of host time per launch otherwise).
// Returns the resident CTAs per SM (cluster == 1) or the resident clusters
// per device (cluster > 1) through *occ.
inline cudaError_t kernel_setup(const void *kern, int threads, size_t smem, int cluster, int *occ) {
    static std::mutex mu;
    static std::map<std::tuple<const void *, int, int, size_t, int>, int> cache;  // -> occupancy
    static std::map<std::pair<const void *, int>, size_t> smem_set;              // opt-in granted so far
    int dev = 0;
    cudaError_t e = cudaGetDevice(&dev);
    if (e != cudaSuccess) return e;
    const auto key = std::make_tuple(kern, dev, threads, smem, cluster);
    std::lock_guard<std::mutex> lock(mu);
    const auto it = cache.find(key);
    if (it != cache.end()) {
        *occ = it->second;
        return cudaSuccess;
    }
    // the opt-in only ever grows: a smaller request must not revoke a larger one
    size_t &granted = smem_set[std::make_pair(kern, dev)];
    if (smem > granted) {
        e = cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, int(smem));
        if (e != cudaSuccess) return e;
        granted = smem;
    }
    int v = 1;
    if (cluster > 1) {
        e = cudaFuncSetAttribute(kern, cudaFuncAttributeNonPortableClusterSizeAllowed, 1);
        if (e != cudaSuccess) return e;
        cudaLaunchConfig_t cfg{};
        cfg.blockDim = dim3(unsigned(threads));
        cfg.gridDim = dim3(unsigned(cluster));
        cfg.dynamicSmemBytes = smem;
        cudaLaunchAttribute attr[1];
        attr[0].id = cudaLaunchAttributeClusterDimension;
        attr[0].val.clusterDim.x = unsigned(cluster);
        attr[0].val.clusterDim.y = 1;
        attr[0].val.clusterDim.z = 1;
        cfg.attrs = attr;
        cfg.numAttrs = 1;
        e = cudaOccupancyMaxActiveClusters(&v, kern, &cfg);
    } else {
        e = cudaOccupancyMaxActiveBlocksPerMultiprocessor(&v, kern, threads, smem);
    }
    if (e != cudaSuccess) return e;
    cache.emplace(key, v);
    *occ = v;
    return cudaSuccess;
}

// Host: SM count of the current device (cached).
inline int sm_count_current() {
    static int sms[64] = {0};
    int dev = 0;
    if (cudaGetDevice(&dev) != cudaSuccess || dev < 0 || dev >= 64) return 148;
    if (sms[dev] == 0) {
        int v = 0;
        cudaDeviceGetAttribute(&v, cudaDevAttrMultiProcessorCount, dev);
        sms[dev] = v > 0 ? v : 148;
    }
    return sms[dev];
}

// Host: opt-in shared memory per CTA of the current device (cached).
inline int smem_optin_current() {
    static int v[64] = {0};
    int dev = 0;
    if (cudaGetDevice(&dev) != cudaSuccess || dev < 0 || dev >= 64) return 232448;
    if (v[dev] == 0) {
        int x = 0;
        cudaDeviceGetAttribute(&x, cudaDevAttrMaxSharedMemoryPerBlockOptin, dev);
        v[dev] = x > 0 ? x : 232448;
    }
    return v[dev];
}

// Host: launch with programmatic stream serialisation (plus an optional cluster).
template <typename... KArgs, typename... Args>
inline cudaError_t launch_pdl(void (*kern)(KArgs...), dim3 grid, dim3 block, size_t smem, cudaStream_t st,
                              int cluster, Args &&...args) {
    cudaLaunchConfig_t cfg{};
    cfg.gridDim = grid;
    cfg.blockDim = block;
    cfg.dynamicSmemBytes = smem;
    cfg.stream = st;
    cudaLaunchAttribute attr[2];
    int na = 0;
    attr[na].id = cudaLaunchAttributeProgrammaticStreamSerialization;
    attr[na].val.programmaticStreamSerializationAllowed = 1;
    ++na;
    if (cluster > 1) {
        attr[na].id = cudaLaunchAttributeClusterDimension;
        attr[na].val.clusterDim.x = unsigned(cluster);
        attr[na].val.clusterDim.y = 1;
        attr[na].val.clusterDim.z = 1;
        ++na;
    }
    cfg.attrs = attr;
    cfg.numAttrs = na;
    return cudaLaunchKernelEx(&cfg, kern, std::forward<Args>(args)...);
}

__device__ __forceinline__ uint32_t smem_u32(const void *p) {
    return static_cast<uint32_t>(__cvta_generic_to_shared(p));
}

__device__ __forceinline__ void mbar_init(uint64_t *bar, uint32_t count) {
    asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(bar)), "r"(count));
}

// Arrive once and announce `bytes` of TMA transactions for the current phase.
__device__ __forceinline__ void mbar_expect_tx(uint64_t *bar, uint32_t bytes) {
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)), "r"(bytes)
                 : "memory");
}

__device__ __forceinline__ void mbar_wait(uint64_t *bar, uint32_t parity) {
    uint32_t done = 0;
    while (!done) {
        asm volatile(
            "{\n .reg .pred p;\n mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2;\n selp.u32 %0, 1, 0, p;\n}\n"
            : "=r"(done)
            : "r"(smem_u32(bar)), "r"(parity)
            : "memory");
    }
}

// Global -> shared bulk copy by the Tensor Memory Accelerator (cp.async.bulk,
// SASS UBLKCP); completion is counted in bytes on the mbarrier.  dst, src and
// bytes must be multiples of 16.
__device__ __forceinline__ void bulk_g2s(void *dst, const void *src, uint32_t bytes, uint64_t *bar) {
    asm volatile(
        "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(
            smem_u32(dst)),
        "l"(src), "r"(bytes), "r"(smem_u32(bar))
        : "memory");
}

// ---- TMA tensor tiles with the 128-byte swizzle --------------------------
// A batch of row slots viewed as a 3-D tensor {ELINE rows per 128-byte line,
// lines per slot, slots}; a box of BL lines lands in shared memory with the
// 16-byte chunks of line L permuted by chunk ^ (L & 7) (the stage must be
// 1024-byte aligned).  A thread reading the 64 or 128 consecutive bytes of its
// rows then hits 8 distinct bank groups per quarter-warp with no register
// rotation.  Coordinates are signed: lines before 0 or past the tensor are
// zero-filled (their bytes still count on the mbarrier).
struct TmapSet {
    CUtensorMap m[4];
};
// the scatter views of a fused split + all-to-all: [array][destination], <= 8 destinations
struct TmapSet24 {
    CUtensorMap m[24];
};

__device__ __forceinline__ void tma_load_lines(void *dst, const CUtensorMap *map, int line, int slot, uint64_t *bar) {
    asm volatile(
        "cp.async.bulk.tensor.3d.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1, {%2, %3, %4}], [%5];" ::
            "r"(smem_u32(dst)),
        "l"(map), "r"(0), "r"(line), "r"(slot), "r"(smem_u32(bar))
        : "memory");
}

// L2 eviction-priority policies for TMA (createpolicy): streamed-once inputs
// evict first, data a later kernel re-reads evicts last.
// TDS_L2HINT bits (default 7): 1 on-chip workspace loads evict-first, 2 on-chip
// x-slot stores evict-last, 4 placement loads evict-first, 8 split input loads
// evict-first, 16 split output stores evict-last (8 and 16 measured neutral /
// slower, profiles/r01g_l2.md).
#ifndef TDS_L2HINT
#define TDS_L2HINT 7
#endif
// Drop a dead 128-byte line from L2 without writing it back (scratch data
// whose last reader has it in shared memory).  p must be 128-byte aligned.
__device__ __forceinline__ void l2_discard_line(const void *p) {
    asm volatile("discard.global.L2 [%0], 128;" ::"l"(p) : "memory");
}
__device__ __forceinline__ uint64_t l2_evict_first() {
    uint64_t p;
    asm volatile("createpolicy.fractional.L2::evict_first.b64 %0, 1.0;" : "=l"(p));
    return p;
}
__device__ __forceinline__ uint64_t l2_evict_last() {
    uint64_t p;
    asm volatile("createpolicy.fractional.L2::evict_last.b64 %0, 1.0;" : "=l"(p));
    return p;
}
__device__ __forceinline__ void tma_load_lines_hint(void *dst, const CUtensorMap *map, int line, int slot, uint64_t *bar,
                                                    uint64_t pol) {
    asm volatile(
        "cp.async.bulk.tensor.3d.shared::cluster.global.mbarrier::complete_tx::bytes.L2::cache_hint [%0], [%1, {%2, %3, "
        "%4}], [%5], %6;" ::"r"(smem_u32(dst)),
        "l"(map), "r"(0), "r"(line), "r"(slot), "r"(smem_u32(bar)), "l"(pol)
        : "memory");
}
__device__ __forceinline__ void tma_load_box3_hint(void *dst, const CUtensorMap *map, int c0, int c1, int c2,
                                                   uint64_t *bar, uint64_t pol) {
    asm volatile(
        "cp.async.bulk.tensor.3d.shared::cluster.global.mbarrier::complete_tx::bytes.L2::cache_hint [%0], [%1, {%2, %3, "
        "%4}], [%5], %6;" ::"r"(smem_u32(dst)),
        "l"(map), "r"(c0), "r"(c1), "r"(c2), "r"(smem_u32(bar)), "l"(pol)
        : "memory");
}

// Element offset of stage row s in a swizzled stage.
template <typename T>
__device__ __forceinline__ int sw_off(int s) {
    constexpr int CH = 16 / int(sizeof(T)), ELINE = 128 / int(sizeof(T));
    const int line = s / ELINE, within = s % ELINE;
    return line * ELINE + (((within / CH) ^ (line & 7)) * CH) + within % CH;
}

// R consecutive rows starting at stage row s0 (a multiple of R) of a swizzled stage.
template <typename T, int R>
__device__ __forceinline__ void lds_rows_sw(const T *stage, int s0, T *v) {
    constexpr int CH = 16 / int(sizeof(T));     // rows per 16-byte chunk
    constexpr int ELINE = 128 / int(sizeof(T));  // rows per line
    const unsigned char *base = reinterpret_cast<const unsigned char *>(stage);
#pragma unroll
    for (int q = 0; q < R / CH; ++q) {
        const int row = s0 + q * CH;
        const int line = row / ELINE, chunk = (row % ELINE) / CH;
        const unsigned char *p = base + line * 128 + ((chunk ^ (line & 7)) << 4);
        if constexpr (sizeof(T) == 4) {
            const float4 f = *reinterpret_cast<const float4 *>(p);
            v[4 * q] = f.x;
            v[4 * q + 1] = f.y;
            v[4 * q + 2] = f.z;
            v[4 * q + 3] = f.w;
        } else {
            const double2 f = *reinterpret_cast<const double2 *>(p);
            v[2 * q] = f.x;
            v[2 * q + 1] = f.y;
        }
    }
}

// TMA tensor store (shared -> global, bulk-group completion) of a 4-D box.
__device__ __forceinline__ void tma_store_4d(const CUtensorMap *map, const void *src, int c0, int c1, int c2, int c3) {
    asm volatile("cp.async.bulk.tensor.4d.global.shared::cta.bulk_group [%0, {%2, %3, %4, %5}], [%1];" ::"l"(map),
                 "r"(smem_u32(src)), "r"(c0), "r"(c1), "r"(c2), "r"(c3)
                 : "memory");
}
__device__ __forceinline__ void tma_store_5d(const CUtensorMap *map, const void *src, int c0, int c1, int c2, int c3,
                                             int c4) {
    asm volatile("cp.async.bulk.tensor.5d.global.shared::cta.bulk_group [%0, {%2, %3, %4, %5, %6}], [%1];" ::"l"(map),
                 "r"(smem_u32(src)), "r"(c0), "r"(c1), "r"(c2), "r"(c3), "r"(c4)
                 : "memory");
}
__device__ __forceinline__ void bulk_commit() { asm volatile("cp.async.bulk.commit_group;" ::: "memory"); }
// the committed bulk stores have finished READING shared memory
__device__ __forceinline__ void bulk_wait_read0() { asm volatile("cp.async.bulk.wait_group.read 0;" ::: "memory"); }
template <int N>
__device__ __forceinline__ void bulk_wait_read() { asm volatile("cp.async.bulk.wait_group.read %0;" ::"n"(N) : "memory"); }
__device__ __forceinline__ void bulk_wait_all() { asm volatile("cp.async.bulk.wait_group 0;" ::: "memory"); }
__device__ __forceinline__ void fence_proxy_async_smem() {
    asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
}

// Host: encode the output view of a split pass -- slot (sys << (kprev + kp)) +
// (rho << kprev) + r as the 4-D tensor {position < slot, r < nr, rho < nrho,
// sys < msys} -- with a box of {box_pos, 1, nrho, 1}.
bool encode_out_tmap(CUtensorMap *out, const void *base, int dsize, int64_t slot, int64_t nr, int64_t nrho,
                     int64_t msys, int box_pos);
// the same output view with the residue split as rho = rho_lo + 16 mu (dims {position,
// r, rho_lo < 16, mu < nrho / 16, system}), box {box_pos, 1, 1, nrho / 16, 1}: one warp's
// residues rho_lo + 16 mu of a tile in one store
bool encode_out5_tmap(CUtensorMap *out, const void *base, int dsize, int64_t slot, int64_t nr, int64_t nrho,
                      int64_t msys, int box_pos);

// R consecutive rows to stage row s0 of a swizzled stage (the inverse of lds_rows_sw).
template <typename T, int R>
__device__ __forceinline__ void sts_rows_sw(T *stage, int s0, const T *v) {
    constexpr int CH = 16 / int(sizeof(T));
    constexpr int ELINE = 128 / int(sizeof(T));
    unsigned char *base = reinterpret_cast<unsigned char *>(stage);
#pragma unroll
    for (int q = 0; q < R / CH; ++q) {
        const int row = s0 + q * CH;
        const int line = row / ELINE, chunk = (row % ELINE) / CH;
        unsigned char *p = base + line * 128 + ((chunk ^ (line & 7)) << 4);
        if constexpr (sizeof(T) == 4)
            *reinterpret_cast<float4 *>(p) = make_float4(v[4 * q], v[4 * q + 1], v[4 * q + 2], v[4 * q + 3]);
        else
            *reinterpret_cast<double2 *>(p) = make_double2(v[2 * q], v[2 * q + 1]);
    }
}

// TMA tensor store of a 3-D row box (the inverse of tma_load_lines).
__device__ __forceinline__ void tma_store_lines(const CUtensorMap *map, const void *src, int line, int slot) {
    asm volatile("cp.async.bulk.tensor.3d.global.shared::cta.bulk_group [%0, {%2, %3, %4}], [%1];" ::"l"(map),
                 "r"(smem_u32(src)), "r"(0), "r"(line), "r"(slot)
                 : "memory");
}

__device__ __forceinline__ void tma_store_lines_hint(const CUtensorMap *map, const void *src, int line, int slot,
                                                     uint64_t pol) {
    asm volatile("cp.async.bulk.tensor.3d.global.shared::cta.bulk_group.L2::cache_hint [%0, {%2, %3, %4}], [%1], %5;" ::"l"(map),
                 "r"(smem_u32(src)), "r"(0), "r"(line), "r"(slot), "l"(pol)
                 : "memory");
}

__device__ __forceinline__ void tma_store_4d_hint(const CUtensorMap *map, const void *src, int c0, int c1, int c2,
                                                  int c3, uint64_t pol) {
    asm volatile("cp.async.bulk.tensor.4d.global.shared::cta.bulk_group.L2::cache_hint [%0, {%2, %3, %4, %5}], [%1], %6;" ::"l"(map),
                 "r"(smem_u32(src)), "r"(c0), "r"(c1), "r"(c2), "r"(c3), "l"(pol)
                 : "memory");
}

// 3-D box load / store with explicit coordinates (generic views).
__device__ __forceinline__ void tma_load_box3(void *dst, const CUtensorMap *map, int c0, int c1, int c2, uint64_t *bar) {
    asm volatile(
        "cp.async.bulk.tensor.3d.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1, {%2, %3, %4}], [%5];" ::
            "r"(smem_u32(dst)),
        "l"(map), "r"(c0), "r"(c1), "r"(c2), "r"(smem_u32(bar))
        : "memory");
}
__device__ __forceinline__ void tma_store_box3(const CUtensorMap *map, const void *src, int c0, int c1, int c2) {
    asm volatile("cp.async.bulk.tensor.3d.global.shared::cta.bulk_group [%0, {%2, %3, %4}], [%1];" ::"l"(map),
                 "r"(smem_u32(src)), "r"(c0), "r"(c1), "r"(c2)
                 : "memory");
}

// Host: a 3-D view with the 128-byte swizzle (box inner dimension = 128 bytes).
bool encode_box3_tmap(CUtensorMap *out, const void *base, int dsize, const uint64_t dims[3], const uint64_t strides[2],
                      const uint32_t box[3]);

// ---- cluster point-to-point transfers (DSMEM): st.async stores into a peer
// CTA's shared memory that count down the peer's mbarrier transaction bytes,
// so a consumer waits on its own mbarrier instead of a cluster barrier.
__device__ __forceinline__ uint32_t cluster_addr(const void *p, int rank) {
    uint32_t r;
    asm volatile("mapa.shared::cluster.u32 %0, %1, %2;" : "=r"(r) : "r"(smem_u32(p)), "r"(rank));
    return r;
}
__device__ __forceinline__ void st_async(uint32_t raddr, float v, uint32_t rbar) {
    asm volatile("st.async.shared::cluster.mbarrier::complete_tx::bytes.b32 [%0], %1, [%2];" ::"r"(raddr),
                 "r"(__float_as_uint(v)), "r"(rbar)
                 : "memory");
}
__device__ __forceinline__ void st_async(uint32_t raddr, double v, uint32_t rbar) {
    asm volatile("st.async.shared::cluster.mbarrier::complete_tx::bytes.b64 [%0], %1, [%2];" ::"r"(raddr),
                 "l"(__double_as_longlong(v)), "r"(rbar)
                 : "memory");
}

// 16 bytes (4 fp32 / 2 fp64) into a peer CTA's shared memory, counted on its mbarrier.
__device__ __forceinline__ void st_async16(uint32_t raddr, const float *v, uint32_t rbar) {
    asm volatile("st.async.shared::cluster.mbarrier::complete_tx::bytes.v4.b32 [%0], {%1, %2, %3, %4}, [%5];" ::"r"(
                     raddr),
                 "r"(__float_as_uint(v[0])), "r"(__float_as_uint(v[1])), "r"(__float_as_uint(v[2])),
                 "r"(__float_as_uint(v[3])), "r"(rbar)
                 : "memory");
}
__device__ __forceinline__ void st_async16(uint32_t raddr, const double *v, uint32_t rbar) {
    asm volatile("st.async.shared::cluster.mbarrier::complete_tx::bytes.v2.b64 [%0], {%1, %2}, [%3];" ::"r"(raddr),
                 "l"(__double_as_longlong(v[0])), "l"(__double_as_longlong(v[1])), "r"(rbar)
                 : "memory");
}
// Arrive (count 1) on an mbarrier of a cluster peer (address from cluster_addr).
// Relaxed: used only as a "this buffer may be overwritten" signal after a CTA
// barrier that completed every read of the buffer (no data is published).
__device__ __forceinline__ void mbar_arrive_remote(uint32_t rbar) {
    asm volatile("mbarrier.arrive.relaxed.cluster.shared::cluster.b64 _, [%0];" ::"r"(rbar) : "memory");
}
// Wait for a phase completed by cluster peers (acquire at cluster scope).
__device__ __forceinline__ void mbar_wait_cluster(uint64_t *bar, uint32_t parity) {
    uint32_t done = 0;
    while (!done) {
        asm volatile(
            "{\n .reg .pred p;\n mbarrier.try_wait.parity.acquire.cluster.shared::cta.b64 p, [%1], %2;\n selp.u32 %0, "
            "1, 0, p;\n}\n"
            : "=r"(done)
            : "r"(smem_u32(bar)), "r"(parity)
            : "memory");
    }
}

// Host: a 3-D view without swizzle (box inner dimension: any multiple of 16 bytes).
bool encode_box3_tmap_plain(CUtensorMap *out, const void *base, int dsize, const uint64_t dims[3],
                            const uint64_t strides[2], const uint32_t box[3]);

// Host: encode the tensor map of `slots` row slots of `lines` full 128-byte
// lines each, slot stride `stride` elements, box of `box_lines` lines.
bool encode_rows_tmap(CUtensorMap *out, const void *base, int dsize, int64_t lines, int64_t slots, int64_t stride,
                      int box_lines);

// Load R consecutive rows (R * sizeof(T) = 16 * NCH bytes, NCH in {2, 4, 8})
// per thread from shared memory into registers without bank conflicts.
// Lanes l whose segments start 16*NCH bytes apart would collide on the same
// 16-byte bank group; lane l reads chunk (q + rot) mod NCH in step q, rot
// chosen so the 8 lanes of a quarter-warp hit 8 distinct groups, and a
// log2(NCH)-stage barrel of predicated selects (FSEL, no branches) undoes it.
template <typename T, int R>
__device__ __forceinline__ void lds_rows(const T *seg, T *v, int lane) {
    constexpr int E = 16 / sizeof(T);      // elements per 16-byte chunk
    constexpr int NCH = R / E;             // chunks per thread
    static_assert(NCH == 2 || NCH == 4 || NCH == 8, "lds_rows: 32, 64 or 128 bytes per thread");
    const int rot = NCH == 8 ? (lane & 7) : NCH == 4 ? ((lane >> 1) & 3) : ((lane >> 2) & 1);
    T arr[NCH][E];
#pragma unroll
    for (int q = 0; q < NCH; ++q) {
        const int c = (q + rot) & (NCH - 1);
        if constexpr (sizeof(T) == 4) {
            const float4 f = reinterpret_cast<const float4 *>(seg)[c];
            arr[q][0] = f.x;
            arr[q][1] = f.y;
            arr[q][2] = f.z;
            arr[q][3] = f.w;
        } else {
            const double2 f = reinterpret_cast<const double2 *>(seg)[c];
            arr[q][0] = f.x;
            arr[q][1] = f.y;
        }
    }
    // arr[q] holds chunk q + rot: rotate right by rot, one bit of rot per stage
#pragma unroll
    for (int b = 1; b < NCH; b <<= 1) {
        const bool on = rot & b;
        T nx[NCH][E];
#pragma unroll
        for (int q = 0; q < NCH; ++q)
#pragma unroll
            for (int e = 0; e < E; ++e) nx[q][e] = on ? arr[(q - b + NCH) & (NCH - 1)][e] : arr[q][e];
#pragma unroll
        for (int q = 0; q < NCH; ++q)
#pragma unroll
            for (int e = 0; e < E; ++e) arr[q][e] = nx[q][e];
    }
#pragma unroll
    for (int q = 0; q < NCH; ++q)
#pragma unroll
        for (int e = 0; e < E; ++e) v[q * E + e] = arr[q][e];
}

}  // namespace tds
