// Launcher of the paper-schedule CR kernel (tridiag_paper.cuh): the GT200
// design of P:L640-696 -- one CTA per system, n/2 threads, in-place shared
// memory, a barrier per step -- kept only as the Fig 9 baseline (E5).
#include "host_common.h"
#include "tridiag_paper.cuh"

namespace tdg_host {

template <typename T>
cudaError_t paper_cr(const T* a, const T* b, const T* c, const T* d, T* x, int64_t n, int64_t S,
                     int mode, cudaStream_t st) {
  const size_t smem = (size_t)5 * (size_t)n * sizeof(T);
  auto kern = mode == 0 ? tdg::tdg_paper_cr_kernel<T, 0> : tdg::tdg_paper_cr_kernel<T, 1>;
  if (smem > 48 * 1024) cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  long long* stamps = stamp_buffer(std::min<int64_t>(S, tdg::kPaperStampBlocks) * tdg::kPaperStampSlots);
  const cudaError_t e = launch_k(kern, dim3((unsigned)S), dim3((unsigned)(n / 2)), smem, st, a, b, c,
                                 d, x, (int)n, stamps);
  if (e != cudaSuccess) return e;
  g_last_launches = 1;
  return cudaGetLastError();
}

template cudaError_t paper_cr<float>(const float*, const float*, const float*, const float*, float*,
                                     int64_t, int64_t, int, cudaStream_t);
template cudaError_t paper_cr<double>(const double*, const double*, const double*, const double*,
                                      double*, int64_t, int64_t, int, cudaStream_t);

}  // namespace tdg_host
