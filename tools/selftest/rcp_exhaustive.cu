// Exhaustive check of the batched fp32 reciprocal (tridiag_device.cuh
// rcp_batch) against CUDA's rcp.rn (__frcp_rn) over every float bit pattern:
// counts bitwise mismatches (NaN results compare as equal when both are NaN).
#include <cstdio>
#include <cstdint>
#include "../../paper_conf_ppopp_zhangco10_b200/csrc/tridiag_device.cuh"

__global__ void check(unsigned long long* mism, unsigned long long* nfast) {
  const uint64_t tid = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x;
  const uint64_t nthr = (uint64_t)gridDim.x * blockDim.x;
  unsigned long long bad = 0, fast = 0;
  const uint64_t groups = 1ull << 30;  // 4 bit patterns per group
  const uint64_t iters = (groups + nthr - 1) / nthr;  // warp-uniform trip count (rcp_batch votes)
  for (uint64_t it = 0; it < iters; ++it) {
    const uint64_t g = it * nthr + tid;
    const bool valid = g < groups;
    const uint64_t base = g * 4;
    float v[4], r[4];
    for (int i = 0; i < 4; ++i) v[i] = valid ? __uint_as_float((uint32_t)(base + i)) : 1.0f;
    tdg::rcp_batch<4>(v, r);
    for (int i = 0; i < 4 && valid; ++i) {
      const float ref = __frcp_rn(v[i]);
      const bool both_nan = (r[i] != r[i]) && (ref != ref);
      if (!both_nan && __float_as_uint(r[i]) != __float_as_uint(ref)) ++bad;
    }
  }
  atomicAdd(mism, bad);
  atomicAdd(nfast, fast);
}

int main() {
  unsigned long long *d, h[2];
  cudaMalloc(&d, 16);
  cudaMemset(d, 0, 16);
  check<<<148 * 8, 256>>>(d, d + 1);
  cudaMemcpy(h, d, 16, cudaMemcpyDeviceToHost);
  printf("{\"test\": \"rcp_batch vs __frcp_rn, all 2^32 fp32 bit patterns\", \"mismatches\": %llu, \"cuda\": \"%s\"}\n",
         h[0], cudaGetErrorString(cudaGetLastError()));
  return h[0] != 0;
}
