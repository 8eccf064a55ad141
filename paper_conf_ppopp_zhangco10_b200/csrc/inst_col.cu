// Launchers of the interleaved-layout (ADI column sweep) CR passes
// (tridiag_colpass.cuh) for T = float / double; the level plan and the
// workspace layout live in tridiag_api.cu (solve_col_t).
#include <cstdlib>

#include "host_common.h"
#include "tridiag_colpass.cuh"

namespace tdg_host {

namespace {
template <typename T>
constexpr int col_R() { return sizeof(T) == 4 ? 16 : 8; }
// Warps per CTA of the TMA reduction / expansion passes (a unit is 32
// systems x W R rows); the chunk every level must divide is the larger one.
#ifndef TDG_COL_RED_W
#define TDG_COL_RED_W 8
#endif
#ifndef TDG_COL_EXP_W
#define TDG_COL_EXP_W 8
#endif
constexpr int kColRedW = TDG_COL_RED_W;
constexpr int kColExpW = TDG_COL_EXP_W;
constexpr int kColW = kColRedW > kColExpW ? kColRedW : kColExpW;
}  // namespace

template <typename T>
int64_t col_chunk() { return (int64_t)kColW * col_R<T>(); }

namespace {
// One array of an interleaved level as a 2-D tensor {S systems, rows}, row
// pitch es elements; boxes of {32 systems, CH rows}, no swizzle.  False when
// the layout cannot be described (TMA needs 16-byte aligned base and pitch).
template <typename T>
bool make_col_map(CUtensorMap* m, const void* base, int64_t S, int64_t rows, int64_t es, int box_rows) {
  auto fn = encode_fn();
  if (!fn) return false;
  if ((reinterpret_cast<uintptr_t>(base) & 15) != 0 || ((uint64_t)es * sizeof(T)) % 16 != 0) return false;
  if (S >= (int64_t(1) << 31) || rows >= (int64_t(1) << 31) || (uint64_t)es * sizeof(T) >= (uint64_t(1) << 40))
    return false;
  const cuuint64_t dims[2] = {(cuuint64_t)S, (cuuint64_t)rows};
  const cuuint64_t strides[1] = {(cuuint64_t)es * sizeof(T)};
  const cuuint32_t box[2] = {32u, (cuuint32_t)box_rows};
  const cuuint32_t estr[2] = {1, 1};
  const CUresult r = fn(m, sizeof(T) == 4 ? CU_TENSOR_MAP_DATA_TYPE_FLOAT32 : CU_TENSOR_MAP_DATA_TYPE_FLOAT64,
                        2, const_cast<void*>(base), dims, strides, box, estr,
                        CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE,
                        // 128 B: a 256-B promotion would fetch the neighbouring
                        // group's half line, which another CTA reads much later
                        // (1.5x DRAM reads measured in the reduction pass)
                        sizeof(T) == 4 ? CU_TENSOR_MAP_L2_PROMOTION_L2_128B
                                       : CU_TENSOR_MAP_L2_PROMOTION_L2_256B,
                        CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  return r == CUDA_SUCCESS;
}

}  // namespace

template <typename T>
cudaError_t col_pass(int which, const T* a, const T* b, const T* c, const T* d, T* o0, T* o1,
                     T* o2, T* o3, const T* x2, int64_t n, int64_t n_real, int64_t es, int64_t S,
                     int64_t es2, int64_t ss2, int kin, T c_pad, cudaStream_t st) {
  constexpr int R = col_R<T>();
  constexpr int W = kColW;
  constexpr int LR = tdg::ilog2c(R);
  const int64_t CH = col_chunk<T>();
  if (kin < 1 || kin > LR || n % CH != 0) return cudaErrorInvalidValue;
  int dev = 0;
  cudaGetDevice(&dev);
  // TMA passes: units of 32 systems x WP R rows (WP = this pass's warps)
  const int WP = which == 1 ? kColRedW : kColExpW;
  const int64_t CHP = (int64_t)WP * R;
  const int64_t units_p = ((S + 31) / 32) * (n / CHP);
  CUtensorMap mA, mB, mC, mD;
  const bool tma = col_tma_mode() != 0 && make_col_map<T>(&mA, a, S, n_real, es, (int)CHP) &&
                   make_col_map<T>(&mB, b, S, n_real, es, (int)CHP) &&
                   make_col_map<T>(&mC, c, S, n_real, es, (int)CHP) &&
                   make_col_map<T>(&mD, d, S, n_real, es, (int)CHP);
  const int64_t units = ((S + 31) / 32) * (n / CH);
  auto pick = [&](auto kin_c) -> cudaError_t {
    constexpr int K = decltype(kin_c)::value;
    if (tma && which == 1) {
      constexpr int WR = kColRedW;
      auto kern = tdg::tdg_col_reduce_tma_kernel<T, R, WR, K>;
      const size_t smem = tdg::col_reduce_tma_smem<T, R, WR>();
      const int occ = occupancy(dev, kern, 32 * WR, smem);
      if (occ <= 0) return cudaErrorInvalidConfiguration;
      int64_t grid = std::max<int64_t>(1, std::min<int64_t>(units_p, (int64_t)device_sms(dev) * occ));
      // row-aligned pieces when every group gets at least one CTA
      const int64_t groups = (S + 31) / 32, C = n / CHP;
      int pieces = 0;
      if (col_order_mode() && groups <= grid) {
        pieces = (int)std::min<int64_t>(C, grid / groups);
        grid = groups * pieces;
      }
      long long* stamps = stamp_buffer(grid * tdg::kStampSystems * tdg::kStampSlots);
      const cudaError_t lerr = launch_k(kern, dim3((unsigned)grid), dim3(32 * WR), smem, st, mA, mB, mC, mD, a, b, c, d, o0, o1,
          o2, o3, n, n_real, es, S, es2, ss2, c_pad, tma_pf_mode(), stamps, pieces);
      if (lerr != cudaSuccess) return lerr;
    } else if (tma) {
      constexpr int WE = kColExpW;
      auto kern = tdg::tdg_col_expand_tma_kernel<T, R, WE, K>;
      const size_t smem = tdg::col_stage_bytes<T, R, WE>() + 16;
      const int occ = occupancy(dev, kern, 32 * WE, smem);
      if (occ <= 0) return cudaErrorInvalidConfiguration;
      const int64_t grid = std::max<int64_t>(1, std::min<int64_t>(units_p, (int64_t)device_sms(dev) * occ));
      long long* stamps = stamp_buffer(grid * tdg::kStampSystems * tdg::kStampSlots);
      const cudaError_t lerr = launch_k(kern, dim3((unsigned)grid), dim3(32 * WE), smem, st, mA, mB, mC, mD, o0, x2, n, n_real, es,
          S, es2, ss2, c_pad, tma_pf_mode() | (col_order_mode() ? 4 : 0), stamps);
      if (lerr != cudaSuccess) return lerr;
    } else if (which == 1) {
      auto kern = tdg::tdg_col_reduce_kernel<T, R, W, K>;
      const size_t smem = tdg::col_reduce_smem<T, R, W>();
      const int occ = occupancy(dev, kern, 32 * W, smem);
      if (occ <= 0) return cudaErrorInvalidConfiguration;
      const int64_t grid = std::max<int64_t>(1, std::min<int64_t>(units, (int64_t)device_sms(dev) * occ));
      const cudaError_t lerr = launch_k(kern, dim3((unsigned)grid), dim3(32 * W), smem, st, a, b, c, d, o0, o1, o2, o3, n, n_real,
          es, S, es2, ss2, c_pad);
      if (lerr != cudaSuccess) return lerr;
    } else {
      auto kern = tdg::tdg_col_expand_kernel<T, R, W, K>;
      const int occ = occupancy(dev, kern, 32 * W, 0);
      if (occ <= 0) return cudaErrorInvalidConfiguration;
      const int64_t grid = std::max<int64_t>(1, std::min<int64_t>(units, (int64_t)device_sms(dev) * occ));
      const cudaError_t lerr = launch_k(kern, dim3((unsigned)grid), dim3(32 * W), 0, st, a, b, c, d, o0, x2, n, n_real, es, S,
          es2, ss2, c_pad);
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

template int64_t col_chunk<float>();
template int64_t col_chunk<double>();
template cudaError_t col_pass<float>(int, const float*, const float*, const float*, const float*,
                                     float*, float*, float*, float*, const float*, int64_t, int64_t,
                                     int64_t, int64_t, int64_t, int64_t, int, float, cudaStream_t);
template cudaError_t col_pass<double>(int, const double*, const double*, const double*,
                                      const double*, double*, double*, double*, double*,
                                      const double*, int64_t, int64_t, int64_t, int64_t, int64_t,
                                      int64_t, int, double, cudaStream_t);

}  // namespace tdg_host
