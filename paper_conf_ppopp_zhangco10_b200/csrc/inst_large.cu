// Launchers of the large-n passes (tridiag_large.cuh) for T = float / double;
// the level plan and workspace layout live in tridiag_api.cu (solve_large).
#include "host_common.h"
#include "tridiag_large.cuh"

namespace tdg_host {

namespace {
template <typename T>
constexpr int large_R() { return sizeof(T) == 4 ? 16 : 8; }
constexpr int kLargeW = 8;

template <typename T>
int persistent_grid(const void* kern, int threads, int64_t units) {
  int dev = 0;
  cudaGetDevice(&dev);
  int occ = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, kern, threads, 0) != cudaSuccess || occ < 1)
    occ = 1;
  return (int)std::max<int64_t>(1, std::min<int64_t>(units, (int64_t)device_sms(dev) * occ));
}
}  // namespace

template <typename T>
int64_t large_chunk() { return 32LL * kLargeW * large_R<T>(); }

template <typename T>
cudaError_t large_pass(int which, const T* a, const T* b, const T* c, const T* d, T* o0, T* o1,
                       T* o2, T* o3, const T* x2, int64_t n, int64_t n_real, int64_t ss,
                       int64_t S, int kin, bool vec, T c_pad, cudaStream_t st) {
  constexpr int R = large_R<T>();
  constexpr int W = kLargeW;
  constexpr int LR = tdg::ilog2c(R);
  const int64_t CH = large_chunk<T>();
  const int64_t C = n / CH;
  if (kin < 1 || kin > LR || n % CH != 0) return cudaErrorInvalidValue;
  // KIN is a template parameter (survivor slots are compile-time indices)
  auto pick = [&](auto kin_c) -> cudaError_t {
    constexpr int K = decltype(kin_c)::value;
    if (which == 1) {
      auto kern = tdg::tdg_large_reduce_kernel<T, R, W, K>;
      const int grid = persistent_grid<T>((const void*)kern, 32 * W, S * C);
      long long* stamps = stamp_buffer((int64_t)grid * tdg::kStampSystems * tdg::kStampSlots);
      const cudaError_t lerr = launch_k(kern, dim3(grid), dim3(32 * W), 0, st, a, b, c, d, o0, o1, o2, o3, n, n_real, ss, S,
          vec ? 1 : 0, c_pad, stamps);
      if (lerr != cudaSuccess) return lerr;
    } else {
      auto kern = tdg::tdg_large_expand_kernel<T, R, W, K>;
      const int grid = persistent_grid<T>((const void*)kern, 32 * W, S * C);
      long long* stamps = stamp_buffer((int64_t)grid * tdg::kStampSystems * tdg::kStampSlots);
      const cudaError_t lerr = launch_k(kern, dim3(grid), dim3(32 * W), 0, st, a, b, c, d, o0, x2, n, n_real, ss, S, vec ? 1
          : 0, c_pad, stamps);
      if (lerr != cudaSuccess) return lerr;
    }
    return cudaGetLastError();
  };
  switch (kin) {
    case 1: return pick(std::integral_constant<int, 1>{});
    case 2: return pick(std::integral_constant<int, 2>{});
    case 3: return pick(std::integral_constant<int, 3>{});
    default:
      if constexpr (LR >= 4) return pick(std::integral_constant<int, (LR >= 4 ? 4 : 3)>{});
      return cudaErrorInvalidValue;
  }
}

template int64_t large_chunk<float>();
template int64_t large_chunk<double>();
template cudaError_t large_pass<float>(int, const float*, const float*, const float*, const float*,
                                       float*, float*, float*, float*, const float*, int64_t,
                                       int64_t, int64_t, int64_t, int, bool, float, cudaStream_t);
template cudaError_t large_pass<double>(int, const double*, const double*, const double*,
                                        const double*, double*, double*, double*, double*,
                                        const double*, int64_t, int64_t, int64_t, int64_t,
                                        int, bool, double, cudaStream_t);

}  // namespace tdg_host
