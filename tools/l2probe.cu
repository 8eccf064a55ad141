// l2probe.cu -- how much of a just-read buffer does a second pass find in L2?
// Standalone probe (not part of the library): read a buffer of X MB with
// 16-byte loads (grid = SMs x 8 CTAs), then read it again; between the two,
// optionally read / write another buffer (pollution of Y MB).
// nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o l2probe l2probe.cu
#include <cstdio>
#include <cuda_runtime.h>

__global__ void rd(const float4* __restrict__ p, size_t n4, float* out) {
  float acc = 0.f;
  for (size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x; i < n4; i += (size_t)gridDim.x * blockDim.x) {
    float4 v = p[i];
    acc += v.x + v.y + v.z + v.w;
  }
  if (acc == 123.456f) out[0] = acc;
}
__global__ void wr(float4* __restrict__ p, size_t n4) {
  for (size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x; i < n4; i += (size_t)gridDim.x * blockDim.x)
    p[i] = make_float4(1.f, 2.f, 3.f, 4.f);
}

int main() {
  int sms = 0;
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  int l2 = 0;
  cudaDeviceGetAttribute(&l2, cudaDevAttrL2CacheSize, 0);
  printf("{\"sms\": %d, \"l2_bytes\": %d}\n", sms, l2);
  const size_t MB = 1 << 20;
  char *a, *b, *flush;
  float* out;
  cudaMalloc(&a, 256 * MB);
  cudaMalloc(&b, 256 * MB);
  cudaMalloc(&flush, 1024 * MB);
  cudaMalloc(&out, 16);
  cudaMemset(a, 0, 256 * MB);
  cudaMemset(b, 0, 256 * MB);
  cudaEvent_t e[4];
  for (auto& x : e) cudaEventCreate(&x);
  const int grid = sms * 8, blk = 256;
  int sizes[] = {8, 16, 24, 32, 48, 64, 80, 96, 112, 128, 192};
  int polls[] = {0, 8, 16, 32};  // MB written between the two reads
  for (int pol : polls) {
    for (int s : sizes) {
      float best1 = 1e9, best2 = 1e9;
      for (int rep = 0; rep < 5; ++rep) {
        cudaMemset(flush, rep, 1024 * MB);
        cudaEventRecord(e[0]);
        rd<<<grid, blk>>>((const float4*)a, s * MB / 16, out);
        cudaEventRecord(e[1]);
        if (pol) wr<<<grid, blk>>>((float4*)b, pol * MB / 16);
        cudaEventRecord(e[2]);
        rd<<<grid, blk>>>((const float4*)a, s * MB / 16, out);
        cudaEventRecord(e[3]);
        cudaEventSynchronize(e[3]);
        float t1, t2;
        cudaEventElapsedTime(&t1, e[0], e[1]);
        cudaEventElapsedTime(&t2, e[2], e[3]);
        if (t1 < best1) best1 = t1;
        if (t2 < best2) best2 = t2;
      }
      printf("{\"pollute_MB\": %d, \"MB\": %d, \"first_us\": %.2f, \"second_us\": %.2f, \"first_GBs\": %.0f, \"second_GBs\": %.0f}\n",
             pol, s, best1 * 1e3, best2 * 1e3, s * MB / (best1 * 1e6), s * MB / (best2 * 1e6));
    }
  }
  return 0;
}
