// Launcher of the single-pass interleaved-layout (ADI column sweep) kernel
// (tridiag_colfused.cuh) for T = float / double.  The choice between it and
// the column passes (inst_col.cu) is made in tridiag_api.cu (solve_col_t).
#include <cstdlib>

#include "host_common.h"
#include "tridiag_colfused.cuh"

namespace tdg_host {

namespace {
template <typename T>
constexpr int cf_R() { return sizeof(T) == 4 ? 16 : 8; }
constexpr int kCfW = 8;

int env_or(const char* name, int dflt) {
  const char* e = getenv(name);
  return (e && *e) ? atoi(e) : dflt;
}

size_t al256(size_t v) { return (v + 255) & ~size_t(255); }

template <typename T>
bool make_cf_map(CUtensorMap* m, const void* base, int64_t S, int64_t rows, int64_t es, int box_rows) {
  auto fn = encode_fn();
  if (!fn) return false;
  if ((reinterpret_cast<uintptr_t>(base) & 15) != 0 || ((uint64_t)es * sizeof(T)) % 16 != 0) return false;
  if (S >= (int64_t(1) << 31) || rows >= (int64_t(1) << 31) || (uint64_t)es * sizeof(T) >= (uint64_t(1) << 40))
    return false;
  const cuuint64_t dims[2] = {(cuuint64_t)S, (cuuint64_t)rows};
  const cuuint64_t strides[1] = {(cuuint64_t)es * sizeof(T)};
  const cuuint32_t box[2] = {32u, (cuuint32_t)box_rows};
  const cuuint32_t estr[2] = {1, 1};
  return fn(m, sizeof(T) == 4 ? CU_TENSOR_MAP_DATA_TYPE_FLOAT32 : CU_TENSOR_MAP_DATA_TYPE_FLOAT64, 2,
            const_cast<void*>(base), dims, strides, box, estr, CU_TENSOR_MAP_INTERLEAVE_NONE,
            CU_TENSOR_MAP_SWIZZLE_NONE,
            sizeof(T) == 4 ? CU_TENSOR_MAP_L2_PROMOTION_L2_128B : CU_TENSOR_MAP_L2_PROMOTION_L2_256B,
            CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE) == CUDA_SUCCESS;
}
}  // namespace

// Shape-only eligibility (no pointers): n padded, inner kPCR / kRD, m the
// intermediate size.  The reduced system of n_red = n / R equations is solved
// by one warp (R2 = n_red / 32 per lane, 2..16) with the register path.
template <typename T>
bool col_fused_eligible(int64_t n, int inner, int64_t m) {
  if (env_or("TRIDIAG_COL_FUSED", 0) == 0) return false;
  constexpr int R = cf_R<T>();
  const int64_t CH = (int64_t)kCfW * R;
  if (n % CH != 0 || n <= 32 * R) return false;
  const int64_t n_red = n / R;
  if (n_red < 64 || n_red > 512) return false;
  if (m < 2 || m > n_red || (m & (m - 1)) != 0) return false;
  const int k2 = tdg::ilog2c((int)(n_red / m));
  const int lr2 = tdg::ilog2c((int)(n_red / 32));
  (void)inner;
  return k2 >= lr2;
}

template <typename T>
size_t col_fused_ws_bytes(int64_t n, int64_t S) {
  const int64_t G = (S + 31) / 32;
  return 5 * al256((size_t)G * 32 * (size_t)(n / cf_R<T>()) * sizeof(T)) + al256((size_t)G * 8 + 4);
}

// Enqueue the fused solve; false if it cannot run for these pointers / this
// device (the caller then takes the column passes).
template <typename T>
bool col_fused(const T* a, const T* b, const T* c, const T* d, T* x, int64_t n, int64_t n_real,
               int64_t es, int64_t S, int inner, int64_t m, T c_pad, void* ws, cudaStream_t st,
               cudaError_t* err) {
  constexpr int R = cf_R<T>();
  constexpr int W = kCfW;
  constexpr int BR = tdg::cf_box_rows<T, R, W>();
  if (!col_fused_eligible<T>(n, inner, m)) return false;
  const int64_t n_red = n / R;
  const int r2 = (int)(n_red / 32);
  const int k2 = tdg::ilog2c((int)(n_red / m));
  const int64_t C = n / (W * R);
  const int64_t G = (S + 31) / 32;
  CUtensorMap mf[4], me[4];
  const void* src[4] = {a, b, c, d};
  for (int q = 0; q < 4; ++q)
    if (!make_cf_map<T>(&mf[q], src[q], S, n_real, es, BR) || !make_cf_map<T>(&me[q], src[q], S, n_real, es, W * R))
      return false;
  int dev = 0;
  cudaGetDevice(&dev);
  T* wsT = static_cast<T*>(ws);
  // (G * 32 * n_red * sizeof(T) is a multiple of 256: n_red >= 64)
  const size_t arr = al256((size_t)G * 32 * (size_t)n_red * sizeof(T));
  unsigned* cnt = reinterpret_cast<unsigned*>(static_cast<char*>(ws) + 5 * arr);
  auto launch = [&](auto kern) -> bool {
    const size_t smem = tdg::cf_smem_bytes<T, R, W>();
    const int occ = occupancy(dev, kern, 32 * W, smem);
    if (occ < 2) return false;  // one forward + one expand CTA per SM
    const int64_t U = G * C;
    int64_t half = (int64_t)device_sms(dev) * occ / 2;
    const int fr = env_or("TRIDIAG_COL_FUSED_FWD_PCT", 50);
    int64_t nf = std::max<int64_t>(1, (int64_t)device_sms(dev) * occ * fr / 100);
    int64_t ne = (int64_t)device_sms(dev) * occ - nf;
    (void)half;
    nf = std::min(nf, U);
    ne = std::max<int64_t>(1, std::min(ne, U));
    *err = cudaMemsetAsync(cnt, 0, (size_t)G * 8 + 4, st);
    if (*err != cudaSuccess) return true;
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = dim3((unsigned)(nf + ne));
    cfg.blockDim = dim3(32 * W);
    cfg.dynamicSmemBytes = smem;
    cfg.stream = st;
    cudaLaunchAttribute attr[1];
    attr[0].id = cudaLaunchAttributeCooperative;
    attr[0].val.cooperative = 1;
    cfg.attrs = attr;
    cfg.numAttrs = 1;
    *err = cudaLaunchKernelEx(&cfg, kern, mf[0], mf[1], mf[2], mf[3], me[0], me[1], me[2], me[3], x, wsT,
                              cnt, (long long)n, (long long)n_real, (long long)es, (long long)S, k2,
                              c_pad, (int)nf);
    return true;
  };
  auto go = [&](auto inner_c) -> bool {
    constexpr int IN = decltype(inner_c)::value;
    switch (r2) {
      case 2: return launch(tdg::tdg_col_fused_kernel<T, R, W, 2, IN>);
      case 4: return launch(tdg::tdg_col_fused_kernel<T, R, W, 4, IN>);
      case 8: return launch(tdg::tdg_col_fused_kernel<T, R, W, 8, IN>);
      case 16: return launch(tdg::tdg_col_fused_kernel<T, R, W, 16, IN>);
      default: return false;
    }
  };
  return inner == tdg::kRD ? go(std::integral_constant<int, tdg::kRD>{})
                           : go(std::integral_constant<int, tdg::kPCR>{});
}

template bool col_fused_eligible<float>(int64_t, int, int64_t);
template bool col_fused_eligible<double>(int64_t, int, int64_t);
template size_t col_fused_ws_bytes<float>(int64_t, int64_t);
template size_t col_fused_ws_bytes<double>(int64_t, int64_t);
template bool col_fused<float>(const float*, const float*, const float*, const float*, float*,
                               int64_t, int64_t, int64_t, int64_t, int, int64_t, float, void*,
                               cudaStream_t, cudaError_t*);
template bool col_fused<double>(const double*, const double*, const double*, const double*,
                                double*, int64_t, int64_t, int64_t, int64_t, int, int64_t, double,
                                void*, cudaStream_t, cudaError_t*);

}  // namespace tdg_host
