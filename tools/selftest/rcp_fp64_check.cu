// Check of the batched fp64 reciprocal (tridiag_device.cuh rcp_batch<double>)
// against CUDA's rcp.rn.f64 (__drcp_rn): 2^32 pseudo-random 64-bit patterns
// (every exponent and sign), plus, for every one of the 2^12 sign/exponent
// values, 2^20 mantissas (edge mantissas 0, 1, max and hashed ones), so the
// fast-path threshold, subnormals, zero, inf and NaN are all covered.  Counts
// bitwise mismatches (NaN results equal when both are NaN).
#include <cstdio>
#include <cstdint>
#include "../../paper_conf_ppopp_zhangco10_b200/csrc/tridiag_device.cuh"

__device__ __forceinline__ uint64_t mix(uint64_t x) {  // splitmix64
  x += 0x9e3779b97f4a7c15ull;
  x = (x ^ (x >> 30)) * 0xbf58476d1ce4e5b9ull;
  x = (x ^ (x >> 27)) * 0x94d049bb133111ebull;
  return x ^ (x >> 31);
}

__global__ void check(unsigned long long* mism, int mode) {
  const uint64_t tid = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x;
  const uint64_t nthr = (uint64_t)gridDim.x * blockDim.x;
  unsigned long long bad = 0;
  const uint64_t groups = 1ull << 30;  // 4 patterns per group
  const uint64_t iters = (groups + nthr - 1) / nthr;
  for (uint64_t it = 0; it < iters; ++it) {
    const uint64_t g = it * nthr + tid;
    const bool valid = g < groups;
    double v[4], r[4];
    for (int i = 0; i < 4; ++i) {
      const uint64_t k = g * 4 + i;
      uint64_t bits;
      if (mode == 0) {
        bits = mix(k);
      } else {  // exponent sweep: sign+exponent from k's top 12 bits of 32, mantissa edge/hashed
        const uint64_t se = (k >> 20) & 0xfff;
        const uint64_t j = k & 0xfffff;
        const uint64_t man = j == 0 ? 0 : j == 1 ? 1 : j == 2 ? 0xfffffffffffffull : (mix(k) & 0xfffffffffffffull);
        bits = (se << 52) | man;
      }
      v[i] = valid ? __longlong_as_double((long long)bits) : 1.0;
    }
    tdg::rcp_batch<4>(v, r);
    for (int i = 0; i < 4 && valid; ++i) {
      const double ref = __drcp_rn(v[i]);
      const bool both_nan = (r[i] != r[i]) && (ref != ref);
      if (!both_nan && __double_as_longlong(r[i]) != __double_as_longlong(ref)) ++bad;
    }
  }
  atomicAdd(mism, bad);
}

int main() {
  unsigned long long *d, h[2];
  cudaMalloc(&d, 16);
  cudaMemset(d, 0, 16);
  check<<<148 * 8, 256>>>(d, 0);
  check<<<148 * 8, 256>>>(d + 1, 1);
  cudaMemcpy(h, d, 16, cudaMemcpyDeviceToHost);
  printf("{\"test\": \"rcp_batch<double> vs __drcp_rn\", \"random_2^32_mismatches\": %llu, "
         "\"exponent_sweep_2^32_mismatches\": %llu, \"cuda\": \"%s\"}\n",
         h[0], h[1], cudaGetErrorString(cudaGetLastError()));
  return (h[0] | h[1]) != 0;
}
