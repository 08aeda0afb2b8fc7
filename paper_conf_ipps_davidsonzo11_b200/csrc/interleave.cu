// interleave.cu -- batch-interleaved layout (ADI / gtsvInterleavedBatch style,
// SURVEY.md §8(f) item 3): element i of system s at ptr[i * m + s].
//
// The solver's kernels stream one system's rows contiguously (TMA boxes of
// whole 128-byte lines), so an interleaved batch is transposed into the
// system-major layout of the ABI, solved by the plan's kernels, and x is
// transposed back.  The transpose moves 32 x 32 tiles through shared memory
// (reads coalesced along systems, writes along rows), up to four arrays per
// tile so one launch carries a, b, c, d; grid-stride over the tiles.
#include "common.cuh"
#include "pipe.cuh"

namespace tds {

template <typename T, int NA>
struct TransposeArgs {
    const T *in[NA];
    T *out[NA];
};

// in: rows x cols row-major  ->  out: cols x rows row-major, NA arrays at once.
template <typename T, int NA>
__global__ void __launch_bounds__(256) transpose_kernel(const TransposeArgs<T, NA> A, int64_t rows, int64_t cols) {
    __shared__ T tile[NA][32][33];
    const int tx = threadIdx.x & 31, ty = threadIdx.x >> 5;  // 32 x 8 threads
    const int64_t tc = (cols + 31) / 32, ntiles = ((rows + 31) / 32) * tc;
    pdl_wait();  // the previous kernel on the stream is complete before any global access
    for (int64_t w = blockIdx.x; w < ntiles; w += gridDim.x) {
        const int64_t r0 = (w / tc) * 32, c0 = (w % tc) * 32;
#pragma unroll
        for (int q = 0; q < NA; ++q)
#pragma unroll
            for (int j = ty; j < 32; j += 8) {
                const int64_t r = r0 + j, c = c0 + tx;
                tile[q][j][tx] = (r < rows && c < cols) ? __ldcs(A.in[q] + r * cols + c) : T(0);
            }
        __syncthreads();
#pragma unroll
        for (int q = 0; q < NA; ++q)
#pragma unroll
            for (int j = ty; j < 32; j += 8) {
                const int64_t c = c0 + j, r = r0 + tx;
                if (c < cols && r < rows) A.out[q][c * rows + r] = tile[q][tx][j];
            }
        __syncthreads();
    }
}

// The same transpose by the Tensor Memory Accelerator (rows and columns of
// whole 16-byte units, 16-byte aligned arrays): per tile and array one
// E x E box (E = 128 bytes of elements, 128-byte swizzle) in by TMA, a
// conflict-free swizzled shared-memory transpose, one box out by a TMA tensor
// store; persistent, the next tile's boxes load while this one is transposed.
template <typename T, int NA>
__global__ void __launch_bounds__(256) transpose_tma_kernel(const __grid_constant__ TmapSet tin,
                                                             const __grid_constant__ TmapSet tout, int64_t rows,
                                                             int64_t cols) {
    constexpr int E = 128 / int(sizeof(T)), CH = 16 / int(sizeof(T)), BOX = E * E;
    extern __shared__ __align__(1024) unsigned char smem_raw[];
    T *base = reinterpret_cast<T *>(smem_raw + ((1024u - (smem_u32(smem_raw) & 1023u)) & 1023u));
    T *sin = base;                 // [2][NA][E rows][E cols]
    T *sout = base + 2 * NA * BOX;  // [NA][E cols][E rows]
    __shared__ __align__(8) uint64_t full[2];
    const int t = threadIdx.x;
    const int64_t tc = (cols + E - 1) / E, ntiles = ((rows + E - 1) / E) * tc;
    auto issue = [&](int64_t w, int s) {  // thread 0
        if (w >= ntiles) return;
        const int r0 = int((w / tc) * E), c0 = int((w % tc) * E);
        mbar_expect_tx(&full[s], NA * BOX * sizeof(T));  // out-of-range elements arrive as zeros
#pragma unroll
        for (int q = 0; q < NA; ++q) tma_load_box3(sin + (s * NA + q) * BOX, &tin.m[q], c0, r0, 0, &full[s]);
    };
    pdl_wait();
    if (t == 0) {
        mbar_init(&full[0], 1);
        mbar_init(&full[1], 1);
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
        issue(blockIdx.x, 0);
        issue(int64_t(blockIdx.x) + gridDim.x, 1);
    }
    __syncthreads();
    for (int64_t it = 0;; ++it) {
        const int64_t w = int64_t(blockIdx.x) + it * gridDim.x;
        if (w >= ntiles) break;
        const int s = int(it & 1);
        mbar_wait(&full[s], uint32_t((it >> 1) & 1));
        if (t == 0) bulk_wait_read0();  // the previous tile's stores have read sout
        __syncthreads();
        for (int task = t; task < NA * E * (E / CH); task += 256) {  // (array, input row r, chunk jq)
            const int q = task / (E * (E / CH)), rem = task % (E * (E / CH)), r = rem % E, jq = rem / E;
            const T *in = sin + (s * NA + q) * BOX + r * E + ((jq ^ (r & 7)) * CH);
            T v[CH];
            if constexpr (sizeof(T) == 4) {
                const float4 f = *reinterpret_cast<const float4 *>(in);
                v[0] = f.x;
                v[1] = f.y;
                v[2] = f.z;
                v[3] = f.w;
            } else {
                const double2 f = *reinterpret_cast<const double2 *>(in);
                v[0] = f.x;
                v[1] = f.y;
            }
            T *out = sout + q * BOX;
#pragma unroll
            for (int e = 0; e < CH; ++e) {
                const int j = jq * CH + e;  // input column = output row
                out[j * E + (((r / CH) ^ (j & 7)) * CH) + r % CH] = v[e];
            }
        }
        fence_proxy_async_smem();
        __syncthreads();
        if (t == 0) {
            const int r0 = int((w / tc) * E), c0 = int((w % tc) * E);
#pragma unroll
            for (int q = 0; q < NA; ++q) tma_store_box3(&tout.m[q], sout + q * BOX, r0, c0, 0);  // clipped at the edges
            bulk_commit();
            issue(w + 2 * int64_t(gridDim.x), s);  // stage s is free: every thread passed the barrier
        }
    }
    if (t == 0) bulk_wait_all();
}

template <typename T, int NA>
static bool launch_transpose_tma(const T *const *in, T *const *out, int64_t rows, int64_t cols, cudaStream_t st,
                                 cudaError_t *err) {
    constexpr int E = 128 / int(sizeof(T));
    if ((cols * int64_t(sizeof(T))) % 16 || (rows * int64_t(sizeof(T))) % 16 || rows >= (int64_t(1) << 31) ||
        cols >= (int64_t(1) << 31))
        return false;
    for (int q = 0; q < NA; ++q)
        if (uintptr_t(in[q]) % 16 || uintptr_t(out[q]) % 16) return false;
    TmapSet tin{}, tout{};
    for (int q = 0; q < NA; ++q) {
        const uint64_t di[3] = {uint64_t(cols), uint64_t(rows), 1}, si[2] = {uint64_t(cols) * sizeof(T),
                                                                             uint64_t(cols) * sizeof(T) * rows};
        const uint64_t dq[3] = {uint64_t(rows), uint64_t(cols), 1}, sq[2] = {uint64_t(rows) * sizeof(T),
                                                                             uint64_t(rows) * sizeof(T) * cols};
        const uint32_t box[3] = {uint32_t(E), uint32_t(E), 1};
        if (!encode_box3_tmap(&tin.m[q], in[q], int(sizeof(T)), di, si, box) ||
            !encode_box3_tmap(&tout.m[q], out[q], int(sizeof(T)), dq, sq, box))
            return false;
    }
    auto kern = transpose_tma_kernel<T, NA>;
    const size_t smem = 1024 + size_t(3 * NA * E * E) * sizeof(T);
    int occ = 1;
    *err = kernel_setup((const void *)kern, 256, smem, 1, &occ);
    if (*err != cudaSuccess) return true;
    const int64_t ntiles = ((rows + E - 1) / E) * ((cols + E - 1) / E);
    const int64_t grid = std::max<int64_t>(1, std::min<int64_t>(ntiles, int64_t(std::max(occ, 1)) * sm_count_current()));
    *err = launch_pdl(kern, dim3(unsigned(grid)), dim3(256), smem, st, 1, tin, tout, rows, cols);
    return true;
}

template <typename T>
cudaError_t launch_transpose(const T *const *in, T *const *out, int narrays, int64_t rows, int64_t cols,
                             cudaStream_t st) {
    const int64_t ntiles = ((rows + 31) / 32) * ((cols + 31) / 32);
    if (ntiles == 0) return cudaSuccess;
    cudaError_t err = cudaSuccess;
    if (narrays == 4 ? launch_transpose_tma<T, 4>(in, out, rows, cols, st, &err)
                     : narrays == 1 && launch_transpose_tma<T, 1>(in, out, rows, cols, st, &err))
        return err;
    const int64_t grid = std::min<int64_t>(ntiles, int64_t(sm_count_current()) * 16);
    if (narrays == 4) {
        TransposeArgs<T, 4> A{};
        for (int q = 0; q < 4; ++q) {
            A.in[q] = in[q];
            A.out[q] = out[q];
        }
        return launch_pdl(transpose_kernel<T, 4>, dim3(unsigned(grid)), dim3(256), 0, st, 1, A, rows, cols);
    }
    if (narrays != 1) return cudaErrorInvalidValue;
    TransposeArgs<T, 1> A{};
    A.in[0] = in[0];
    A.out[0] = out[0];
    return launch_pdl(transpose_kernel<T, 1>, dim3(unsigned(grid)), dim3(256), 0, st, 1, A, rows, cols);
}

template cudaError_t launch_transpose<float>(const float *const *, float *const *, int, int64_t, int64_t,
                                             cudaStream_t);
template cudaError_t launch_transpose<double>(const double *const *, double *const *, int, int64_t, int64_t,
                                              cudaStream_t);

}  // namespace tds
