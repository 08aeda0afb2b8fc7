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

template <typename T>
cudaError_t launch_transpose(const T *const *in, T *const *out, int narrays, int64_t rows, int64_t cols,
                             cudaStream_t st) {
    const int64_t ntiles = ((rows + 31) / 32) * ((cols + 31) / 32);
    if (ntiles == 0) return cudaSuccess;
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
