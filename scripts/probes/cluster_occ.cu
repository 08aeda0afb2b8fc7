// Max active clusters per device for cluster sizes 1..16 at one CTA per SM
// (large dynamic shared memory) and at two CTAs per SM (diagnostic).
#include <cstdio>
#include <cuda_runtime.h>
__global__ void dummy() { extern __shared__ char s[]; if (threadIdx.x == 0) s[0] = 0; }
int main() {
    cudaFuncSetAttribute(dummy, cudaFuncAttributeNonPortableClusterSizeAllowed, 1);
    for (size_t smem : {size_t(200 * 1024), size_t(100 * 1024)}) {
        cudaFuncSetAttribute(dummy, cudaFuncAttributeMaxDynamicSharedMemorySize, int(smem));
        for (int c = 1; c <= 16; ++c) {
            cudaLaunchConfig_t cfg{};
            cfg.blockDim = dim3(256);
            cfg.gridDim = dim3(c);
            cfg.dynamicSmemBytes = smem;
            cudaLaunchAttribute a[1];
            a[0].id = cudaLaunchAttributeClusterDimension;
            a[0].val.clusterDim.x = c; a[0].val.clusterDim.y = 1; a[0].val.clusterDim.z = 1;
            cfg.attrs = a; cfg.numAttrs = 1;
            int n = -1;
            cudaError_t e = cudaOccupancyMaxActiveClusters(&n, dummy, &cfg);
            printf("smem %zu KB cluster %2d: max active clusters %d (%d CTAs) %s\n", smem / 1024, c, n, n * c,
                   e == cudaSuccess ? "" : cudaGetErrorString(e));
        }
    }
    return 0;
}
