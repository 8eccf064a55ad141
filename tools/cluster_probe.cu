// cluster_probe.cu -- how many thread-block clusters of a given size can be
// co-resident on this GPU at 1 CTA/SM (cudaOccupancyMaxActiveClusters)?
// nvcc -gencode arch=compute_100a,code=sm_100a -o cluster_probe cluster_probe.cu
#include <cstdio>
#include <cuda_runtime.h>

__global__ void k(float* p) {
  extern __shared__ float s[];
  s[threadIdx.x] = threadIdx.x;
  __syncthreads();
  if (p) p[blockIdx.x] = s[(threadIdx.x + 1) % blockDim.x];
}

int main() {
  cudaFuncSetAttribute(k, cudaFuncAttributeNonPortableClusterSizeAllowed, 1);
  const int smems[] = {64 << 10, 136 << 10, 200 << 10};
  const int threads[] = {256, 512};
  for (int sm : smems) {
    cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, sm);
    for (int th : threads) {
      for (int cs = 1; cs <= 16; cs *= 2) {
        cudaLaunchConfig_t cfg = {};
        cfg.gridDim = dim3(cs * 16);
        cfg.blockDim = dim3(th);
        cfg.dynamicSmemBytes = sm;
        cudaLaunchAttribute at[1];
        at[0].id = cudaLaunchAttributeClusterDimension;
        at[0].val.clusterDim.x = cs; at[0].val.clusterDim.y = 1; at[0].val.clusterDim.z = 1;
        cfg.attrs = at; cfg.numAttrs = 1;
        int n = -1;
        cudaError_t e = cudaOccupancyMaxActiveClusters(&n, k, &cfg);
        printf("{\"smem_kb\": %d, \"threads\": %d, \"cluster\": %d, \"max_active_clusters\": %d, \"ctas\": %d, \"err\": \"%s\"}\n",
               sm >> 10, th, cs, n, n * cs, cudaGetErrorString(e));
      }
    }
  }
  return 0;
}
