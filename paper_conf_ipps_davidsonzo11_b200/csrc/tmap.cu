// tmap.cu -- host-side encoding of the TMA tensor maps used by the persistent
// kernels (pipe.cuh).  The driver entry point is resolved through the runtime
// (cudaGetDriverEntryPoint), so libtds.so needs no link against libcuda.
#include <cudaTypedefs.h>

#include "pipe.cuh"

namespace tds {

static PFN_cuTensorMapEncodeTiled_v12000 encode_fn() {
    static const PFN_cuTensorMapEncodeTiled_v12000 fn = [] {
        void *p = nullptr;
        cudaDriverEntryPointQueryResult q{};
        if (cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &p, cudaEnableDefault, &q) != cudaSuccess ||
            q != cudaDriverEntryPointSuccess)
            return static_cast<PFN_cuTensorMapEncodeTiled_v12000>(nullptr);
        return reinterpret_cast<PFN_cuTensorMapEncodeTiled_v12000>(p);
    }();
    return fn;
}

bool encode_rows_tmap(CUtensorMap *out, const void *base, int dsize, int64_t lines, int64_t slots, int64_t stride,
                      int box_lines) {
    const PFN_cuTensorMapEncodeTiled_v12000 fn = encode_fn();
    if (!fn || lines < 1 || slots < 1 || box_lines < 1 || box_lines > 256) return false;
    const cuuint64_t dims[3] = {cuuint64_t(128 / dsize), cuuint64_t(lines), cuuint64_t(slots)};
    const cuuint64_t strides[2] = {128, cuuint64_t(stride) * cuuint64_t(dsize)};
    const cuuint32_t box[3] = {cuuint32_t(128 / dsize), cuuint32_t(box_lines), 1};
    const cuuint32_t estr[3] = {1, 1, 1};
    const CUresult r = fn(out, dsize == 4 ? CU_TENSOR_MAP_DATA_TYPE_FLOAT32 : CU_TENSOR_MAP_DATA_TYPE_FLOAT64, 3,
                          const_cast<void *>(base), dims, strides, box, estr, CU_TENSOR_MAP_INTERLEAVE_NONE,
                          CU_TENSOR_MAP_SWIZZLE_128B, CU_TENSOR_MAP_L2_PROMOTION_L2_256B,
                          CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    return r == CUDA_SUCCESS;
}

bool encode_out_tmap(CUtensorMap *out, const void *base, int dsize, int64_t slot, int64_t nr, int64_t nrho,
                     int64_t msys, int box_pos) {
    const PFN_cuTensorMapEncodeTiled_v12000 fn = encode_fn();
    if (!fn || slot < 1 || nr < 1 || nrho < 1 || nrho > 256 || msys < 1 || box_pos < 1 || box_pos > 256) return false;
    const cuuint64_t ds = cuuint64_t(dsize);
    const cuuint64_t dims[4] = {cuuint64_t(slot), cuuint64_t(nr), cuuint64_t(nrho), cuuint64_t(msys)};
    const cuuint64_t strides[3] = {cuuint64_t(slot) * ds, cuuint64_t(slot * nr) * ds, cuuint64_t(slot * nr * nrho) * ds};
    const cuuint32_t box[4] = {cuuint32_t(box_pos), 1, cuuint32_t(nrho), 1};
    const cuuint32_t estr[4] = {1, 1, 1, 1};
    const CUresult r = fn(out, dsize == 4 ? CU_TENSOR_MAP_DATA_TYPE_FLOAT32 : CU_TENSOR_MAP_DATA_TYPE_FLOAT64, 4,
                          const_cast<void *>(base), dims, strides, box, estr, CU_TENSOR_MAP_INTERLEAVE_NONE,
                          CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_NONE,
                          CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    return r == CUDA_SUCCESS;
}

bool encode_out5_tmap(CUtensorMap *out, const void *base, int dsize, int64_t slot, int64_t nr, int64_t nrho,
                      int64_t msys, int box_pos) {
    const PFN_cuTensorMapEncodeTiled_v12000 fn = encode_fn();
    if (!fn || slot < 1 || nr < 1 || nrho < 16 || nrho % 16 != 0 || nrho > 4096 || msys < 1 || box_pos < 1 ||
        box_pos > 256)
        return false;
    const cuuint64_t ds = cuuint64_t(dsize);
    const cuuint64_t dims[5] = {cuuint64_t(slot), cuuint64_t(nr), 16, cuuint64_t(nrho / 16), cuuint64_t(msys)};
    const cuuint64_t strides[4] = {cuuint64_t(slot) * ds, cuuint64_t(slot * nr) * ds, cuuint64_t(slot * nr * 16) * ds,
                                   cuuint64_t(slot * nr * nrho) * ds};
    const cuuint32_t box[5] = {cuuint32_t(box_pos), 1, 1, cuuint32_t(nrho / 16), 1};
    const cuuint32_t estr[5] = {1, 1, 1, 1, 1};
    const CUresult r = fn(out, dsize == 4 ? CU_TENSOR_MAP_DATA_TYPE_FLOAT32 : CU_TENSOR_MAP_DATA_TYPE_FLOAT64, 5,
                          const_cast<void *>(base), dims, strides, box, estr, CU_TENSOR_MAP_INTERLEAVE_NONE,
                          CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_NONE,
                          CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    return r == CUDA_SUCCESS;
}

bool encode_box3_tmap(CUtensorMap *out, const void *base, int dsize, const uint64_t dims[3], const uint64_t strides[2],
                      const uint32_t box[3]) {
    const PFN_cuTensorMapEncodeTiled_v12000 fn = encode_fn();
    if (!fn) return false;
    for (int i = 0; i < 3; ++i)
        if (dims[i] < 1 || box[i] < 1 || box[i] > 256) return false;
    const cuuint64_t d[3] = {dims[0], dims[1], dims[2]};
    const cuuint64_t st[2] = {strides[0], strides[1]};
    const cuuint32_t b[3] = {box[0], box[1], box[2]};
    const cuuint32_t estr[3] = {1, 1, 1};
    const CUresult r = fn(out, dsize == 4 ? CU_TENSOR_MAP_DATA_TYPE_FLOAT32 : CU_TENSOR_MAP_DATA_TYPE_FLOAT64, 3,
                          const_cast<void *>(base), d, st, b, estr, CU_TENSOR_MAP_INTERLEAVE_NONE,
                          CU_TENSOR_MAP_SWIZZLE_128B, CU_TENSOR_MAP_L2_PROMOTION_L2_256B,
                          CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    return r == CUDA_SUCCESS;
}

bool encode_box3_tmap_plain(CUtensorMap *out, const void *base, int dsize, const uint64_t dims[3],
                            const uint64_t strides[2], const uint32_t box[3]) {
    const PFN_cuTensorMapEncodeTiled_v12000 fn = encode_fn();
    if (!fn) return false;
    for (int i = 0; i < 3; ++i)
        if (dims[i] < 1 || box[i] < 1 || box[i] > 256) return false;
    const cuuint64_t d[3] = {dims[0], dims[1], dims[2]};
    const cuuint64_t st[2] = {strides[0], strides[1]};
    const cuuint32_t b[3] = {box[0], box[1], box[2]};
    const cuuint32_t estr[3] = {1, 1, 1};
    const CUresult r = fn(out, dsize == 4 ? CU_TENSOR_MAP_DATA_TYPE_FLOAT32 : CU_TENSOR_MAP_DATA_TYPE_FLOAT64, 3,
                          const_cast<void *>(base), d, st, b, estr, CU_TENSOR_MAP_INTERLEAVE_NONE,
                          CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_NONE,
                          CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    return r == CUDA_SUCCESS;
}

}  // namespace tds
