// split_reg.cuh -- register-level building blocks of the split pass (G1):
// one PCR level over 16 register rows per thread, and the de-interleaved
// vector store of one residue's run.  Shared by split_reg.cu and split_pipe.cu.
#pragma once
#include "common.cuh"

namespace tds {

template <typename T, int G>
__device__ __forceinline__ void store_run(T *p, const T *v) {
    if constexpr (G * sizeof(T) >= 16) {
        constexpr int W = 16 / sizeof(T);
#pragma unroll
        for (int q = 0; q < G / W; ++q) {
            if constexpr (sizeof(T) == 4)
                reinterpret_cast<float4 *>(p)[q] = make_float4(v[4 * q], v[4 * q + 1], v[4 * q + 2], v[4 * q + 3]);
            else
                reinterpret_cast<double2 *>(p)[q] = make_double2(v[2 * q], v[2 * q + 1]);
        }
    } else if constexpr (G * sizeof(T) == 8 && sizeof(T) == 4) {
        reinterpret_cast<float2 *>(p)[0] = make_float2(v[0], v[1]);
    } else {
#pragma unroll
        for (int u = 0; u < G; ++u) p[u] = v[u];
    }
}

// One PCR level with compile-time stride S on 16 register rows per thread.
// A level couples only rows of one class rho (mod S): each class is updated in
// place, ascending, carrying the previous OLD row, so only a few registers
// beyond the 48 row values stay live.  eL/eR: [2][3][NW][SM] edge buffers.
template <typename T, int R, int S, int NW, int SM>
__device__ __forceinline__ void reg_level(T (&ra)[R], T (&rc)[R], T (&rd)[R], T *eL, T *eR, int bsel, int lane,
                                          int warp) {
    auto E = [&](T *e, int arr, int w, int u) -> T & { return e[((bsel * 3 + arr) * NW + w) * SM + u]; };
    if (lane == 0) {
#pragma unroll
        for (int u = 0; u < S; ++u) {
            E(eL, 0, warp, u) = ra[u];
            E(eL, 1, warp, u) = rc[u];
            E(eL, 2, warp, u) = rd[u];
        }
    }
    if (lane == 31) {
#pragma unroll
        for (int u = 0; u < S; ++u) {
            E(eR, 0, warp, u) = ra[R - S + u];
            E(eR, 1, warp, u) = rc[R - S + u];
            E(eR, 2, warp, u) = rd[R - S + u];
        }
    }
    __syncthreads();
#pragma unroll
    for (int rho = 0; rho < S; ++rho) {
        // left neighbour of row rho: row R-S+rho of thread t-1 (old; same class)
        T pa = __shfl_up_sync(0xffffffffu, ra[R - S + rho], 1);
        T pc = __shfl_up_sync(0xffffffffu, rc[R - S + rho], 1);
        T pd = __shfl_up_sync(0xffffffffu, rd[R - S + rho], 1);
        // right neighbour of row R-S+rho: row rho of thread t+1 (old)
        T xa = __shfl_down_sync(0xffffffffu, ra[rho], 1);
        T xc = __shfl_down_sync(0xffffffffu, rc[rho], 1);
        T xd = __shfl_down_sync(0xffffffffu, rd[rho], 1);
        if (lane == 0) {
            const bool h = warp > 0;
            const int w = h ? warp - 1 : 0;
            pa = h ? E(eR, 0, w, rho) : T(0);
            pc = h ? E(eR, 1, w, rho) : T(0);
            pd = h ? E(eR, 2, w, rho) : T(0);
        }
        if (lane == 31) {
            const bool h = warp < NW - 1;
            const int w = h ? warp + 1 : 0;
            xa = h ? E(eL, 0, w, rho) : T(0);
            xc = h ? E(eL, 1, w, rho) : T(0);
            xd = h ? E(eL, 2, w, rho) : T(0);
        }
#pragma unroll
        for (int v = rho; v < R; v += S) {
            const T oa = ra[v], oc = rc[v], od = rd[v];
            const bool last = v + S >= R;
            row_update(ra[v], rc[v], rd[v], pa, pc, pd, last ? xa : ra[(v + S) % R], last ? xc : rc[(v + S) % R],
                       last ? xd : rd[(v + S) % R]);
            pa = oa;
            pc = oc;
            pd = od;
        }
    }
}

// One PCR level with stride S (in the thread's own row index) over chains of
// W lanes (__shfl width W): the lanes of a segment hold consecutive R-row
// blocks of one chain.  The first / last lane of a segment get their own rows
// back as "neighbours" -- garbage that spreads 2^l - 1 rows per level from the
// segment ends, i.e. stays inside the halo the caller discards (after l
// levels, rows closer than 2^l - 1 to a segment end are invalid).  No shared
// memory, no barrier, no select.
template <typename T, int R, int S, int W>
__device__ __forceinline__ void reg_level_w(T (&ra)[R], T (&rc)[R], T (&rd)[R]) {
    if constexpr (sizeof(T) == 4 && S % 2 == 0) {
        // fp32, even stride: classes rho and rho + 1 move together as row pairs
        // (v, v+1), whose neighbours (v -+ S, v+1 -+ S) are again aligned pairs
        auto P = [](const T *r, int v) { return make_float2(r[v], r[v + 1]); };
#pragma unroll
        for (int rho = 0; rho < S; rho += 2) {
            float2 pa, pc, pd, xa, xc, xd;
            pa.x = __shfl_up_sync(0xffffffffu, ra[R - S + rho], 1, W);
            pa.y = __shfl_up_sync(0xffffffffu, ra[R - S + rho + 1], 1, W);
            pc.x = __shfl_up_sync(0xffffffffu, rc[R - S + rho], 1, W);
            pc.y = __shfl_up_sync(0xffffffffu, rc[R - S + rho + 1], 1, W);
            pd.x = __shfl_up_sync(0xffffffffu, rd[R - S + rho], 1, W);
            pd.y = __shfl_up_sync(0xffffffffu, rd[R - S + rho + 1], 1, W);
            xa.x = __shfl_down_sync(0xffffffffu, ra[rho], 1, W);
            xa.y = __shfl_down_sync(0xffffffffu, ra[rho + 1], 1, W);
            xc.x = __shfl_down_sync(0xffffffffu, rc[rho], 1, W);
            xc.y = __shfl_down_sync(0xffffffffu, rc[rho + 1], 1, W);
            xd.x = __shfl_down_sync(0xffffffffu, rd[rho], 1, W);
            xd.y = __shfl_down_sync(0xffffffffu, rd[rho + 1], 1, W);
#pragma unroll
            for (int v = rho; v < R; v += S) {
                float2 a = P(ra, v), c = P(rc, v), d = P(rd, v);
                const float2 oa = a, oc = c, od = d;
                const bool last = v + S >= R;
                row_update2(a, c, d, pa, pc, pd, last ? xa : P(ra, (v + S) % R), last ? xc : P(rc, (v + S) % R),
                            last ? xd : P(rd, (v + S) % R));
                ra[v] = a.x;
                ra[v + 1] = a.y;
                rc[v] = c.x;
                rc[v + 1] = c.y;
                rd[v] = d.x;
                rd[v + 1] = d.y;
                pa = oa;
                pc = oc;
                pd = od;
            }
        }
    } else {
#pragma unroll
    for (int rho = 0; rho < S; ++rho) {
        T pa = __shfl_up_sync(0xffffffffu, ra[R - S + rho], 1, W);
        T pc = __shfl_up_sync(0xffffffffu, rc[R - S + rho], 1, W);
        T pd = __shfl_up_sync(0xffffffffu, rd[R - S + rho], 1, W);
        T xa = __shfl_down_sync(0xffffffffu, ra[rho], 1, W);
        T xc = __shfl_down_sync(0xffffffffu, rc[rho], 1, W);
        T xd = __shfl_down_sync(0xffffffffu, rd[rho], 1, W);
#pragma unroll
        for (int v = rho; v < R; v += S) {
            const T oa = ra[v], oc = rc[v], od = rd[v];
            const bool last = v + S >= R;
            row_update(ra[v], rc[v], rd[v], pa, pc, pd, last ? xa : ra[(v + S) % R], last ? xc : rc[(v + S) % R],
                       last ? xd : rd[(v + S) % R]);
            pa = oa;
            pc = oc;
            pd = od;
        }
    }
    }
}

// Shared-memory transpose buffer of the deep split kernel: element (m, rho) =
// row 16m + rho of the tile at 16m + (rho ^ g(m)), g(m) = ((m >> 4) + (m >> 1)) & 15.
// Layout-A writes (fixed rho, consecutive m across lanes) and layout-B reads
// (fixed m offset, m 16 apart across lanes, two rho per warp) both hit at most
// two lanes per bank.
__device__ __forceinline__ int tr_addr(int m, int rho) { return 16 * m + (rho ^ (((m >> 4) + (m >> 1)) & 15)); }

// layout A -> buffer: the R rows of block m
template <typename T, int R>
__device__ __forceinline__ void tr_write(const T (&x)[R], T *buf, int m) {
#pragma unroll
    for (int v = 0; v < R; ++v) buf[tr_addr(m, v)] = x[v];
}

// buffer -> layout B: the addresses of members mb .. mb+R-1 of class rho
// (mb even, mb mod 16 = MBLOW known at compile time, so g(mb + u) =
// (g0 + K(u)) & 15 with a compile-time K); members outside [0, AV) -- the
// halo lanes b = 0 / 15 -- are clamped to a valid address (halo garbage).
template <int R, int AV, int MBLOW>
__device__ __forceinline__ void tr_read_addrs(int mb, int rho, int (&ad)[R]) {
    const int g0 = (mb >> 4) + (mb >> 1);
#pragma unroll
    for (int u = 0; u < R; ++u) {
        const int k = ((MBLOW + u) >> 4) + (u >> 1);
        const int a = 16 * (mb + u) + (rho ^ ((g0 + k) & 15));
        ad[u] = int(min(unsigned(a), unsigned(16 * AV - 1)));
    }
}

// fp32 class-major transpose buffer [rho][m] (row stride AV): member m of
// class rho at rho*AV + 4*((m >> 2) ^ ((m >> 5) & 3)) + (m & 3).  Layout-A
// writes are 16 scalar stores at immediate offsets (consecutive m across the
// warp, <= 2-way conflicts); layout-B reads are 4 LDS.128 of 4 consecutive
// members each, conflict-free across the 16 lanes of a class.
__device__ __forceinline__ int trc_phys(int m) { return (((m >> 2) ^ ((m >> 5) & 3)) << 2) | (m & 3); }

template <typename T, int R, int AV>
__device__ __forceinline__ void trc_write(const T (&x)[R], T *p) {  // p = buf + trc_phys(m)
#pragma unroll
    for (int v = 0; v < R; ++v) p[v * AV] = x[v];
}

// chunk offsets of members mb + 4q (mb a multiple of 4).  Chunks outside
// [0, AV) (halo lanes, garbage anyway) are moved by whole lanes (4 chunks) onto
// the chunk a neighbouring lane of the same quarter-warp reads in the same
// instruction: a broadcast, so the halo lanes add no extra wavefront.
template <int R, int AV>
__device__ __forceinline__ void trc_read_chunks(int mb, int (&ch)[R / 4]) {
#pragma unroll
    for (int q = 0; q < R / 4; ++q) {
        int c = mb / 4 + q;
        c = c < 0 ? c + 4 : c;
        c = c > AV / 4 - 1 ? c - 4 : c;
        c = c > AV / 4 - 1 ? c - 4 : c;
        ch[q] = (c ^ ((c >> 3) & 3)) << 2;
    }
}

template <int R>
__device__ __forceinline__ void trc_read(float (&x)[R], const float *row, const int (&ch)[R / 4]) {
#pragma unroll
    for (int q = 0; q < R / 4; ++q) {
        const float4 f = *reinterpret_cast<const float4 *>(row + ch[q]);
        x[4 * q] = f.x;
        x[4 * q + 1] = f.y;
        x[4 * q + 2] = f.z;
        x[4 * q + 3] = f.w;
    }
}

// fp32 512-thread and fp64 256-thread tiles (TDS_SPLIT_TR34): the class
// transpose without bank conflicts in either direction.  Class row rho holds
// its members as 16 sub-rows (m mod 16) of W elements, member m at
// (m & 15) * W + (m >> 4).
// fp32, W = 34 words: layout-A stores (30 consecutive m across a warp, one
// class per store) land on banks (2 (m & 15) + (m >> 4)) mod 32: distinct,
// because members one sub-row column apart differ in parity and members two
// columns apart would need (m & 15) to step by one across a whole window.
// Layout-B loads (one class per warp, lanes b 16 members apart, member u of
// every lane in one load) read 32 consecutive words.
// fp64, W = 17 doubles: an 8-byte store is served per half-warp (15
// consecutive members, lanes 1..15 / 16..30), whose 8-byte bank pairs
// ((m & 15) + (m >> 4)) mod 16 are distinct (a window spans two sub-row
// columns, and m, m' one column apart collide only if (m & 15) - (m' & 15) = 1,
// i.e. never inside one window); layout-B loads (one class per half-warp)
// read 16 consecutive doubles.  Each direction is one wavefront per access:
// 16 scalar loads per array instead of 4 LDS.128 (fp32) / 8 (fp64), the same
// wavefronts; the [rho][m] swizzles keep ~1.6 (fp32) / ~1.7 (fp64) wavefronts
// per store.
template <typename T>
struct Tr34 {
    static constexpr int W = sizeof(T) == 4 ? 34 : 17;
    // class-row stride: the last stored member is 15 W + AV / 16 - 1 (AV = 480 / 240);
    // the halo lanes' reads run to sub-row column 15 of the last sub-row (fp64: inside
    // the class; fp32: 2 words into the next class or the 32 spare words after the
    // buffer).  Any stride keeps the banks: one class per access (per half-warp).
    static constexpr int C = sizeof(T) == 4 ? 540 : 271;
    static constexpr int SLACK = sizeof(T) == 4 ? 32 : 0;
};
template <typename T>
__device__ __forceinline__ int tr34_phys(int m) { return (m & 15) * Tr34<T>::W + (m >> 4); }

// members mb + u, u = 0..R-1, of the class whose row starts at row; mb = LEFT - 16 + 16 b
// and p = row + b - 1, so member mb + u is p[((LEFT + u) & 15) * W + ((LEFT + u) >> 4)]:
// a compile-time offset from one per-thread base (halo lanes read padding / neighbours)
template <int R, int LEFT, typename T>
__device__ __forceinline__ void tr34_read(T (&x)[R], const T *p) {
#pragma unroll
    for (int u = 0; u < R; ++u) x[u] = p[((LEFT + u) & 15) * Tr34<T>::W + ((LEFT + u) >> 4)];
}

// fp64 class-major buffer [rho][m] (row stride AV doubles): member m at
// 2 * (c ^ ((c >> 3) & 7)) + (m & 1), c = m >> 1 (16-byte chunks of two
// members XOR-swizzled by the 128-byte block).  Layout-A writes are 16 scalar
// stores of consecutive m across the warp; layout-B reads are 8 LDS.128 of two
// consecutive members each, lanes 16 members apart: the 8 lanes of a
// quarter-warp hit 8 different bank groups.
__device__ __forceinline__ int trc_phys64(int m) {
    const int c = m >> 1;
    return ((c ^ ((c >> 3) & 7)) << 1) | (m & 1);
}

template <int R, int AV>
__device__ __forceinline__ void trc_read_chunks64(int mb, int (&ch)[R / 2]) {
#pragma unroll
    for (int q = 0; q < R / 2; ++q) {
        int c = mb / 2 + q;  // chunks outside [0, AV/2): a neighbouring lane's chunk (broadcast)
        c = c < 0 ? c + 8 : c;
        c = c > AV / 2 - 1 ? c - 8 : c;
        c = c > AV / 2 - 1 ? c - 8 : c;
        ch[q] = (c ^ ((c >> 3) & 7)) << 1;
    }
}

template <int R>
__device__ __forceinline__ void trc_read64(double (&x)[R], const double *row, const int (&ch)[R / 2]) {
#pragma unroll
    for (int q = 0; q < R / 2; ++q) {
        const double2 f = *reinterpret_cast<const double2 *>(row + ch[q]);
        x[2 * q] = f.x;
        x[2 * q + 1] = f.y;
    }
}

template <typename T, int R>
__device__ __forceinline__ void tr_read(T (&x)[R], const T *buf, const int (&ad)[R]) {
#pragma unroll
    for (int u = 0; u < R; ++u) x[u] = buf[ad[u]];
}

}  // namespace tds
