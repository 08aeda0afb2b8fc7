// Which TMA tensor stores fault on sm_100a?  ./tma_store_probe CASE
//   0: coords (0,0,0)   1: coords (-4,0,0)   2: coords (480,0,0)   3: box inner 64 elems at (0,0,0)
//   4: coords (-4,0,0) with box inner 64
#include <cuda.h>
#include <cudaTypedefs.h>
#include <cuda_runtime.h>
#include <cstdio>
#include <cstdlib>

__global__ void store_kernel(const CUtensorMap *map, int c0, int nelem) {
    extern __shared__ __align__(1024) float buf[];
    for (int i = threadIdx.x; i < nelem; i += blockDim.x) buf[i] = float(i);
    asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
    __syncthreads();
    if (threadIdx.x == 0) {
        unsigned s = (unsigned)__cvta_generic_to_shared(buf);
        asm volatile("cp.async.bulk.tensor.3d.global.shared::cta.bulk_group [%0, {%2, %3, %4}], [%1];" ::"l"(map),
                     "r"(s), "r"(c0), "r"(0), "r"(0) : "memory");
        asm volatile("cp.async.bulk.commit_group;" ::: "memory");
        asm volatile("cp.async.bulk.wait_group 0;" ::: "memory");
    }
}

int main(int argc, char **argv) {
    const int cs = argc > 1 ? atoi(argv[1]) : 0;
    void *p = nullptr;
    cudaDriverEntryPointQueryResult q{};
    cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &p, cudaEnableDefault, &q);
    auto enc = reinterpret_cast<PFN_cuTensorMapEncodeTiled_v12000>(p);
    float *dst;
    const int stride = 504, qn = 4;
    cudaMalloc(&dst, stride * qn * sizeof(float));
    const unsigned inner = (cs >= 3) ? 64 : 240;
    cuuint64_t dims[3] = {500, cuuint64_t(qn), 1};
    cuuint64_t strides[2] = {stride * 4, stride * 4 * qn};
    cuuint32_t box[3] = {inner, cuuint32_t(qn), 1};
    cuuint32_t estr[3] = {1, 1, 1};
    CUtensorMap hmap;
    CUresult r = enc(&hmap, CU_TENSOR_MAP_DATA_TYPE_FLOAT32, 3, dst, dims, strides, box, estr,
                     CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_NONE,
                     CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    CUtensorMap *dmap;
    cudaMalloc(&dmap, sizeof(hmap));
    cudaMemcpy(dmap, &hmap, sizeof(hmap), cudaMemcpyHostToDevice);
    const int c0 = (cs == 1 || cs == 4) ? -4 : (cs == 2 ? 480 : 0);
    store_kernel<<<1, 128, inner * qn * 4>>>(dmap, c0, inner * qn);
    cudaError_t e = cudaDeviceSynchronize();
    printf("case %d: encode=%d c0=%d inner=%u -> %s\n", cs, int(r), c0, inner, cudaGetErrorString(e));
    return 0;
}
