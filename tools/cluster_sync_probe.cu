// cluster_sync_probe.cu -- cycles per cluster.sync() (barrier.cluster arrive +
// wait) for clusters of 2..16 CTAs of 512 threads, one CTA per SM, and the
// cost of a DSMEM store burst before it.
// nvcc -gencode arch=compute_100a,code=sm_100a -o cluster_sync_probe cluster_sync_probe.cu
#include <cooperative_groups.h>
#include <cstdio>
#include <cuda_runtime.h>
namespace cg = cooperative_groups;

__global__ void __launch_bounds__(512, 1) k(long long* out, int iters, int remote) {
  extern __shared__ float s[];
  cg::cluster_group cl = cg::this_cluster();
  const int r = (int)cl.block_rank(), n = (int)cl.num_blocks();
  float* peer = cl.map_shared_rank(s, (r + 1) % n);
  cl.sync();
  long long t0 = clock64();
  for (int i = 0; i < iters; ++i) {
    if (remote) peer[threadIdx.x + 512 * (i & 7)] = (float)i;
    cl.sync();
  }
  long long t1 = clock64();
  if (threadIdx.x == 0) out[blockIdx.x] = (t1 - t0) / iters;
}

int main() {
  long long* d;
  cudaMalloc(&d, 4096 * sizeof(long long));
  cudaFuncSetAttribute(k, cudaFuncAttributeNonPortableClusterSizeAllowed, 1);
  cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, 150 << 10);
  for (int remote = 0; remote < 2; ++remote)
    for (int cs = 2; cs <= 16; cs *= 2) {
      cudaLaunchConfig_t cfg = {};
      cudaLaunchAttribute at[1];
      at[0].id = cudaLaunchAttributeClusterDimension;
      at[0].val.clusterDim.x = cs; at[0].val.clusterDim.y = 1; at[0].val.clusterDim.z = 1;
      cfg.attrs = at; cfg.numAttrs = 1;
      cfg.blockDim = dim3(512);
      cfg.dynamicSmemBytes = 150 << 10;
      int nc = 0;
      cfg.gridDim = dim3(cs);
      cudaOccupancyMaxActiveClusters(&nc, k, &cfg);
      cfg.gridDim = dim3(cs * nc);
      cudaLaunchKernelEx(&cfg, k, d, 1000, remote);
      cudaDeviceSynchronize();
      long long h[4096];
      cudaMemcpy(h, d, cs * nc * sizeof(long long), cudaMemcpyDeviceToHost);
      double avg = 0;
      for (int i = 0; i < cs * nc; ++i) avg += h[i];
      printf("{\"cluster\": %d, \"clusters\": %d, \"remote_store_per_thread\": %d, \"cycles_per_sync\": %.0f, \"err\": \"%s\"}\n",
             cs, nc, remote, avg / (cs * nc), cudaGetErrorString(cudaGetLastError()));
    }
  return 0;
}
