// launch.cuh -- kernel launchers and dispatch of libtridiag.so (included by
// the instantiation units inst_*.cu; see host_common.h).
#pragma once

#include "host_common.h"
#include "tridiag_ileave.cuh"
#include "tridiag_tma.cuh"

namespace tdg_host {

using tdg::ilog2c;

template <typename T, int R, int INNER, int KB>
cudaError_t launch_ileave_k(const T* a, const T* b, const T* c, const T* d, T* x, int64_t n,
                            int64_t S, int k, cudaStream_t st, int64_t n_real, Layout L) {
  const int P = (int)(n / R);
  const int lp = ilog2c(P);
  int dev = 0;
  cudaGetDevice(&dev);
  // narrow tiles (16-byte row segments: 2^LNS threads at P = 32) when the
  // default tiles would leave SMs idle (the paper's literal n x n sweeps)
  constexpr int LNS = 5 + ilog2c(16 / (int)sizeof(T));
  const bool narrow = lp == 5 && ((S + (512 / 32) - 1) / (512 / 32)) < (int64_t)device_sms(dev) &&
                      small_cta_mode();
  const int threads = narrow ? (1 << LNS) : 1 << tdg::ilv_log_threads(lp);
  const int G = threads / P;  // a tile is threads * R elements per array
  const size_t smem = (size_t)5 * tdg::ilv_tile_elems((int)n, G) * sizeof(T);
  if (smem > 227 * 1024) return cudaErrorInvalidValue;
  // compile-time geometry for the lane counts the plans use (P = 4 .. 32)
  auto kern = narrow  ? tdg::tdg_ileave_kernel<T, R, INNER, KB, 5, LNS>
            : lp == 5 ? tdg::tdg_ileave_kernel<T, R, INNER, KB, 5>
            : lp == 4 ? tdg::tdg_ileave_kernel<T, R, INNER, KB, 4>
            : lp == 3 ? tdg::tdg_ileave_kernel<T, R, INNER, KB, 3>
            : lp == 2 ? tdg::tdg_ileave_kernel<T, R, INNER, KB, 2>
                      : tdg::tdg_ileave_kernel<T, R, INNER, KB, -1>;
  const int occ = occupancy(dev, kern, threads, smem);
  if (occ <= 0) return cudaErrorInvalidConfiguration;
  const int64_t tiles = (S + G - 1) / G;
  const int64_t grid = std::max<int64_t>(1, std::min<int64_t>(tiles, (int64_t)device_sms(dev) * occ));
  const T c_pad = INNER == tdg::kRD ? T(1) : T(0);
  const cudaError_t lerr = launch_k(kern, dim3((unsigned)grid), dim3(threads), smem, st, a, b, c, d, x, (int)n, (long long)S, k,
      lp, (int)n_real, c_pad, (long long)L.es);
  if (lerr != cudaSuccess) return lerr;
  g_last_launches = 1;
  return cudaGetLastError();
}

template <typename T, int R, int INNER, int KB>
cudaError_t launch_warp_k(const T* a, const T* b, const T* c, const T* d, T* x, int64_t n,
                          int64_t S, int k, bool vec, cudaStream_t st, int64_t n_real, Layout L) {
  if (L.ss == 1 && L.es != 1) return launch_ileave_k<T, R, INNER, KB>(a, b, c, d, x, n, S, k, st, n_real, L);
  const int P = (int)(n / R);
  const int log2P = ilog2c(P);
  const int G = 32 / P;
  int dev = 0;
  cudaGetDevice(&dev);
  // 8 warps per CTA; a batch too small to give every SM 8 warps is spread
  // over all SMs in smaller CTAs instead (fewer warps per scheduler: the
  // latency-bound regime of the paper-sized batches, e.g. 512 x 512)
  const bool small = vec && blocked_minb() != 1 && P >= 4 && tdg::pcr_small_cta<T, R, INNER, KB, false>();
  // compile-time P: the small-CTA PCR kernels and the LU-form RD kernel
  const bool lp_fixed = small || (vec && blocked_minb() != 1 && P >= 4 && INNER == tdg::kSTONE);
  int wpb = small ? 4 : 8;
  {
    const int64_t warps_needed = (S + G - 1) / G;
    const int64_t sms = device_sms(dev);
    while (wpb > 1 && warps_needed < sms * wpb && small_cta_mode()) wpb >>= 1;
  }
  const int threads = wpb * 32;
  // vec: the contiguous power-of-two vector path; otherwise the general
  // (scalar / strided / padded) instantiation
  // The tuned register path (KB < 0, vector) lets ptxas choose (~127
  // registers); every other instantiation asks for two CTAs per SM
  // (TRIDIAG_BLOCKED_MINB=1 at run time selects the unconstrained build for
  // the blocked inner instead, for A/B measurements).
  // ragged contiguous rows with 16-byte aligned systems: per-lane vector
  // accesses, no staging (register path)
  const bool rag = KB < 0 && !vec && L.es == 1 && (L.ss >= n_real || S <= 1) &&
                   (R * sizeof(T)) % 16 == 0 && ((uint64_t)L.ss * sizeof(T)) % 16 == 0 &&
                   ((reinterpret_cast<uintptr_t>(a) | reinterpret_cast<uintptr_t>(b) |
                     reinterpret_cast<uintptr_t>(c) | reinterpret_cast<uintptr_t>(d) |
                     reinterpret_cast<uintptr_t>(x)) & 15) == 0 &&
                   rag_tma_mode();
  // the small-CTA PCR kernels and the LU-form RD kernel with P fixed at compile time
  auto small_kern = [&] {
    if constexpr (tdg::pcr_small_cta<T, R, INNER, KB, false>())
      return log2P == 5   ? tdg::tdg_warp_blocked_kernel<T, R, INNER, KB, false, true, 5>
             : log2P == 4 ? tdg::tdg_warp_blocked_kernel<T, R, INNER, KB, false, true, 4>
             : log2P == 3 ? tdg::tdg_warp_blocked_kernel<T, R, INNER, KB, false, true, 3>
                          : tdg::tdg_warp_blocked_kernel<T, R, INNER, KB, false, true, 2>;
    else if constexpr (INNER == tdg::kSTONE)  // LU-form RD: P fixed at compile time too
      return log2P == 5   ? tdg::tdg_warp_blocked_kernel<T, R, INNER, KB, false, false, 5>
             : log2P == 4 ? tdg::tdg_warp_blocked_kernel<T, R, INNER, KB, false, false, 4>
             : log2P == 3 ? tdg::tdg_warp_blocked_kernel<T, R, INNER, KB, false, false, 3>
                          : tdg::tdg_warp_blocked_kernel<T, R, INNER, KB, false, false, 2>;
    else
      return tdg::tdg_warp_blocked_kernel<T, R, INNER, KB, false>;
  }();
  auto kern = rag ? tdg::tdg_warp_kernel<T, R, INNER, KB, false, true>
            : (KB < 0 && vec) ? tdg::tdg_warp_kernel<T, R, INNER, KB, false>
            : (KB < 0)        ? tdg::tdg_warp_blocked_kernel<T, R, INNER, KB, true>
            : vec ? (blocked_minb() == 1 ? tdg::tdg_warp_kernel<T, R, INNER, KB, false>
                     : lp_fixed          ? small_kern
                                         : tdg::tdg_warp_blocked_kernel<T, R, INNER, KB, false>)
                  : tdg::tdg_warp_blocked_kernel<T, R, INNER, KB, true>;
  const size_t tiles = (vec || rag) ? 0 : (((size_t)wpb * 4 * tdg::warp_tile_elems<T, R>() * sizeof(T) + 15) & ~size_t(15));
  const size_t smem = tiles + (size_t)wpb * tdg::pcr_scratch_bytes<T, R, INNER, KB>();
  const int occ = occupancy(dev, kern, threads, smem);
  if (occ <= 0) return cudaErrorInvalidConfiguration;
  const int64_t groups = (S + (int64_t)wpb * G - 1) / ((int64_t)wpb * G);
  const int64_t grid = std::max<int64_t>(1, std::min<int64_t>(groups, (int64_t)device_sms(dev) * occ));
  const int pm = prefetch_mode();
  const int pf = (vec && (pm == 1 || (pm == 2 && P == 32)) ? 1 : 0) | (prewait_pf_mode() ? 2 : 0);
  const T c_pad = INNER == tdg::kRD ? T(1) : T(0);
  long long* stamps = stamp_buffer((int64_t)grid * tdg::kStampSystems * tdg::kStampSlots);
  const cudaError_t lerr = launch_k(kern, dim3((unsigned)grid), dim3(threads), smem, st, a, b, c, d, x, (int)n, (long long)S, k,
      log2P, vec ? 1 : 0, pf, (int)n_real, c_pad, (long long)L.es, (long long)L.ss, stamps);
  if (lerr != cudaSuccess) return lerr;
  g_last_launches = 1;
  return cudaGetLastError();
}

// k >= log2 R: one register-path kernel for every such k; k < log2 R: the
// blocked-inner kernel compiled for that k.
template <typename T, int R, int INNER>
cudaError_t launch_warp(const T* a, const T* b, const T* c, const T* d, T* x, int64_t n,
                        int64_t S, int k, bool vec, cudaStream_t st, int64_t nr, Layout L) {
  constexpr int LR = ilog2c(R);
  if constexpr (INNER == tdg::kSTONE)  // k = 0 always: the whole system in registers
    return launch_warp_k<T, R, INNER, (LR > 0 ? 0 : -1)>(a, b, c, d, x, n, S, 0, vec, st, nr, L);
  if (k >= LR) return launch_warp_k<T, R, INNER, -1>(a, b, c, d, x, n, S, k, vec, st, nr, L);
  switch (k) {
    case 0: return launch_warp_k<T, R, INNER, 0>(a, b, c, d, x, n, S, k, vec, st, nr, L);
    case 1: if constexpr (LR > 1) return launch_warp_k<T, R, INNER, 1>(a, b, c, d, x, n, S, k, vec, st, nr, L); break;
    case 2: if constexpr (LR > 2) return launch_warp_k<T, R, INNER, 2>(a, b, c, d, x, n, S, k, vec, st, nr, L); break;
    case 3: if constexpr (LR > 3) return launch_warp_k<T, R, INNER, 3>(a, b, c, d, x, n, S, k, vec, st, nr, L); break;
  }
  return cudaErrorInvalidValue;
}

// View one input array as [S*n/R rows][R columns] (64-byte rows), boxes of
// min(P, 256) rows, 64-byte swizzle.
template <typename T>
bool make_row_map(CUtensorMap* m, const void* base, int64_t rows, int R, int box_rows) {
  auto fn = encode_fn();
  if (!fn) return false;
  const cuuint64_t dims[2] = {(cuuint64_t)R, (cuuint64_t)rows};
  const cuuint64_t strides[1] = {(cuuint64_t)R * sizeof(T)};
  const cuuint32_t box[2] = {(cuuint32_t)R, (cuuint32_t)box_rows};
  const cuuint32_t estr[2] = {1, 1};
  const CUresult r = fn(m, sizeof(T) == 4 ? CU_TENSOR_MAP_DATA_TYPE_FLOAT32 : CU_TENSOR_MAP_DATA_TYPE_FLOAT64,
                        2, const_cast<void*>(base), dims, strides, box, estr,
                        CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_64B,
                        CU_TENSOR_MAP_L2_PROMOTION_L2_256B, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  return r == CUDA_SUCCESS;
}

// Ragged and / or pitched rows (system stride ss >= n_real, ss T a multiple of
// 16 B): 3-D map {R, ceil(n_real/R), S} with strides {R T, ss T}
// (tdg_cta_tma_kernel<..., RAG = true>).
template <typename T>
bool make_rag_map(CUtensorMap* m, const void* base, int64_t n_real, int64_t ss, int64_t S, int R, int box_rows) {
  auto fn = encode_fn();
  if (!fn) return false;
  if ((reinterpret_cast<uintptr_t>(base) & 15) != 0 || ((uint64_t)ss * sizeof(T)) % 16 != 0) return false;
  const int64_t rows = (n_real + R - 1) / R;
  if (S >= (int64_t(1) << 31) || rows >= (int64_t(1) << 31)) return false;
  const cuuint64_t dims[3] = {(cuuint64_t)R, (cuuint64_t)rows, (cuuint64_t)S};
  const cuuint64_t strides[2] = {(cuuint64_t)R * sizeof(T), (cuuint64_t)ss * sizeof(T)};
  const cuuint32_t box[3] = {(cuuint32_t)R, (cuuint32_t)box_rows, 1};
  const cuuint32_t estr[3] = {1, 1, 1};
  const CUresult r = fn(m, sizeof(T) == 4 ? CU_TENSOR_MAP_DATA_TYPE_FLOAT32 : CU_TENSOR_MAP_DATA_TYPE_FLOAT64,
                        3, const_cast<void*>(base), dims, strides, box, estr,
                        CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_64B,
                        CU_TENSOR_MAP_L2_PROMOTION_L2_256B, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  return r == CUDA_SUCCESS;
}

template <typename T, int R, int W, int INNER>
cudaError_t launch_cta_tma(const T* a, const T* b, const T* c, const T* d, T* x, int64_t n,
                           int64_t S, int k, cudaStream_t st, bool* used, int64_t nr = -1,
                           int64_t ss = -1) {
  *used = false;
  const int P = 32 * W;
  if (nr < 0) nr = n;
  if (ss < 0) ss = n;
  const bool rag = nr != n || ss != n;
  const int64_t rows = S * P;
  if (rows >= (int64_t(1) << 31)) return cudaSuccess;
  CUtensorMap mA, mB, mC, mD;
  const int box = P > 256 ? 256 : P;
  if (rag) {
    if ((reinterpret_cast<uintptr_t>(x) & 15) != 0 || !make_rag_map<T>(&mA, a, nr, ss, S, R, box) ||
        !make_rag_map<T>(&mB, b, nr, ss, S, R, box) || !make_rag_map<T>(&mC, c, nr, ss, S, R, box) ||
        !make_rag_map<T>(&mD, d, nr, ss, S, R, box))
      return cudaSuccess;
  } else if (!make_row_map<T>(&mA, a, rows, R, box) || !make_row_map<T>(&mB, b, rows, R, box) ||
             !make_row_map<T>(&mC, c, rows, R, box) || !make_row_map<T>(&mD, d, rows, R, box)) {
    return cudaSuccess;
  }
  const size_t smem = tdg::cta_tma_smem_bytes<T>(R, W, INNER, k);
  int dev = 0;
  cudaGetDevice(&dev);
  constexpr int LR = ilog2c(R);
  auto kern = tdg::tdg_cta_tma_kernel<T, R, W, INNER, -1>;
  if (rag) {
    // register path only (k >= log2 R; RD: k > log2 R)
    if (k < LR || (INNER == tdg::kRD && k == LR)) return cudaSuccess;
    kern = tdg::tdg_cta_tma_kernel<T, R, W, INNER, -1, true>;
  }
  // RD with k <= log2 R (one survivor per lane at k = log2 R): blocked CTA scan
  if (!rag && (k < LR || (INNER == tdg::kRD && k == LR))) {
    if constexpr (INNER != tdg::kRD) {
      return cudaSuccess;
    } else {
      switch (k) {
        case 0: kern = tdg::tdg_cta_tma_kernel<T, R, W, INNER, 0>; break;
        case 1: kern = tdg::tdg_cta_tma_kernel<T, R, W, INNER, (LR > 1 ? 1 : 0)>; break;
        case 2: kern = tdg::tdg_cta_tma_kernel<T, R, W, INNER, (LR > 2 ? 2 : 0)>; break;
        case 3: kern = tdg::tdg_cta_tma_kernel<T, R, W, INNER, (LR > 3 ? 3 : 0)>; break;
        default: kern = tdg::tdg_cta_tma_kernel<T, R, W, INNER, LR>; break;
      }
    }
  }
  int occ = occupancy(dev, kern, W * 32, smem);
  if (occ <= 0) return cudaSuccess;
  // double-buffered heads / survivor regions (no end-of-system barrier) when
  // that does not cost occupancy (TRIDIAG_CTA_DBUF=0 disables)
  size_t smem_use = smem;
  int dbuf = 0;
  if (cta_dbuf_mode()) {
    const size_t smem2 = tdg::cta_tma_smem_bytes<T>(R, W, INNER, k, 2);
    if (smem2 <= 227 * 1024 && occupancy(dev, kern, W * 32, smem2) >= occ) {
      smem_use = smem2;
      dbuf = (int)(tdg::cta_tma_region_bytes<T>(R, W, INNER, k) / sizeof(T));
    }
  }
  const int64_t grid = std::max<int64_t>(1, std::min<int64_t>(S, (int64_t)device_sms(dev) * occ));
  long long* stamps = stamp_buffer(grid * tdg::kStampSystems * tdg::kStampSlots);
  const cudaError_t lerr = launch_k(kern, dim3((unsigned)grid), dim3(W * 32), smem_use, st, mA, mB, mC, mD, x, (int)n, (long long)S, k, dbuf, (tma_pf_mode() ? 1 : 0) | (prewait_pf_mode() ? 2 : 0), (int)nr,
                                    (long long)ss, stamps);
  if (lerr != cudaSuccess) return lerr;
  g_last_launches = 1;
  *used = true;
  return cudaGetLastError();
}

template <typename T, int R, int W, int INNER>
cudaError_t launch_cta(const T* a, const T* b, const T* c, const T* d, T* x, int64_t n,
                       int64_t S, int k, bool vec, cudaStream_t st, int64_t nr, Layout L) {
  if (vec && nr == n && L.es == 1 && L.ss == n && (k >= ilog2c(R) || INNER == tdg::kRD) &&
      tma_mode()) {
    bool used = false;
    const cudaError_t e = launch_cta_tma<T, R, W, INNER>(a, b, c, d, x, n, S, k, st, &used);
    if (used || e != cudaSuccess) return e;
  }
  // ragged contiguous rows with 16-byte aligned systems: the TMA kernel with
  // 3-D maps (rows past the system zero-filled, padding in registers)
  if ((nr != n || L.ss != n) && L.es == 1 && (L.ss >= nr || S <= 1) && tma_mode() && rag_tma_mode()) {
    bool used = false;
    const int64_t ss = S <= 1 ? std::max<int64_t>(nr, (L.ss * (int64_t)sizeof(T) % 16) ? ((nr + 3) & ~3LL) : L.ss) : L.ss;
    const cudaError_t e = launch_cta_tma<T, R, W, INNER>(a, b, c, d, x, n, S, k, st, &used, nr, ss);
    if (used || e != cudaSuccess) return e;
  }
  const bool staged = (nr != n || !vec) && L.es == 1;
  const size_t smem = tdg::cta_smem_bytes<T>(R, W, INNER, k, staged);
  int dev = 0;
  cudaGetDevice(&dev);
  constexpr int LR = ilog2c(R);
  // RD with k < log2 R: register-blocked CTA scan compiled for that k
  auto kern = tdg::tdg_cta_kernel<T, R, W, INNER, -1>;
  if (k < LR || (INNER == tdg::kRD && k == LR)) {
    if constexpr (INNER != tdg::kRD) {
      kern = tdg::tdg_cta_kernel<T, R, W, INNER, -2>;
    } else {
      switch (k) {
        case 0: kern = tdg::tdg_cta_kernel<T, R, W, INNER, 0>; break;
        case 1: kern = tdg::tdg_cta_kernel<T, R, W, INNER, (LR > 1 ? 1 : 0)>; break;
        case 2: kern = tdg::tdg_cta_kernel<T, R, W, INNER, (LR > 2 ? 2 : 0)>; break;
        case 3: kern = tdg::tdg_cta_kernel<T, R, W, INNER, (LR > 3 ? 3 : 0)>; break;
        default: kern = tdg::tdg_cta_kernel<T, R, W, INNER, LR>; break;
      }
    }
  }
  const int occ = occupancy(dev, kern, W * 32, smem);
  if (occ <= 0) return cudaErrorInvalidConfiguration;
  const int64_t grid = std::max<int64_t>(1, std::min<int64_t>(S, (int64_t)device_sms(dev) * occ));
  const int pm = prefetch_mode();
  const int pf = vec && (pm == 1 || pm == 2) ? 1 : 0;
  const T c_pad = INNER == tdg::kRD ? T(1) : T(0);
  const cudaError_t lerr = launch_k(kern, dim3((unsigned)grid), dim3(W * 32), smem, st, a, b, c, d, x, (int)n, (long long)S, k,
      vec ? 1 : 0, pf, (int)nr, c_pad, (long long)L.es, (long long)L.ss);
  if (lerr != cudaSuccess) return lerr;
  g_last_launches = 1;
  return cudaGetLastError();
}

template <typename T, int INNER>
cudaError_t dispatch_t(const void* a_, const void* b_, const void* c_, const void* d_, void* x_,
                       int64_t n, int64_t S, int k, cudaStream_t st, int dtype, int64_t nr,
                       Layout L) {
  const T* a = static_cast<const T*>(a_);
  const T* b = static_cast<const T*>(b_);
  const T* c = static_cast<const T*>(c_);
  const T* d = static_cast<const T*>(d_);
  T* x = static_cast<T*>(x_);
  // The RD-family inners use a work-efficient block scan whose association
  // depends on R, so they always take the HBM-scale plan: results stay
  // bitwise independent of the batch size (R22).
  const Plan p = plan_for(dtype, n, INNER == tdg::kPCR ? S : -1);
  const size_t tile = std::min<size_t>(32, (size_t)p.R * sizeof(T));
  auto al = [tile](const void* q) { return (reinterpret_cast<uintptr_t>(q) % tile) == 0; };
  const bool vec = nr == n && L.es == 1 && ((uint64_t)L.ss * sizeof(T)) % tile == 0 && al(a) &&
                   al(b) && al(c) && al(d) && al(x);
  if (!p.cta) {
    switch (p.R) {
      case 1: return launch_warp<T, 1, INNER>(a, b, c, d, x, n, S, k, vec, st, nr, L);
      case 2: return launch_warp<T, 2, INNER>(a, b, c, d, x, n, S, k, vec, st, nr, L);
      case 4: return launch_warp<T, 4, INNER>(a, b, c, d, x, n, S, k, vec, st, nr, L);
      case 8: return launch_warp<T, 8, INNER>(a, b, c, d, x, n, S, k, vec, st, nr, L);
      case 16:
        if constexpr (sizeof(T) == 4) return launch_warp<T, 16, INNER>(a, b, c, d, x, n, S, k, vec, st, nr, L);
        break;
    }
    return cudaErrorInvalidValue;
  }
  if constexpr (INNER == tdg::kSTONE) {
    return cudaErrorInvalidValue;  // n <= 32 R only (tridiag_max_n)
  } else if constexpr (sizeof(T) == 4) {
    switch (p.W) {
      case 2: return launch_cta<T, 16, 2, INNER>(a, b, c, d, x, n, S, k, vec, st, nr, L);
      case 4: return launch_cta<T, 16, 4, INNER>(a, b, c, d, x, n, S, k, vec, st, nr, L);
      case 8: return launch_cta<T, 16, 8, INNER>(a, b, c, d, x, n, S, k, vec, st, nr, L);
      case 16: return launch_cta<T, 16, 16, INNER>(a, b, c, d, x, n, S, k, vec, st, nr, L);
    }
  } else {
    switch (p.W) {
      case 2: return launch_cta<T, 8, 2, INNER>(a, b, c, d, x, n, S, k, vec, st, nr, L);
      case 4: return launch_cta<T, 8, 4, INNER>(a, b, c, d, x, n, S, k, vec, st, nr, L);
      case 8: return launch_cta<T, 8, 8, INNER>(a, b, c, d, x, n, S, k, vec, st, nr, L);
      case 16: return launch_cta<T, 8, 16, INNER>(a, b, c, d, x, n, S, k, vec, st, nr, L);
    }
  }
  return cudaErrorInvalidValue;
}


}  // namespace tdg_host
