// host_common.h -- host-side declarations shared by the translation units of
// libtridiag.so (tridiag_api.cu and the per-(dtype, inner) kernel
// instantiation units inst_*.cu, compiled in parallel).
#pragma once

#include <cuda.h>
#include <cuda_runtime.h>
#include <cudaTypedefs.h>

#include <algorithm>
#include <cstdint>
#include <map>
#include <mutex>
#include <tuple>
#include <utility>

#include "tridiag.h"

namespace tdg_host {

extern thread_local int g_last_launches;  // launches of the last call on this thread
// Kernels launched by the last call on this thread, in launch order (the
// first kMaxKernelLog; diagnostic: tridiag_last_kernel_name).
constexpr int kMaxKernelLog = 16;
extern thread_local const void* g_kernel_log[kMaxKernelLog];
extern thread_local int g_kernel_log_len;
inline void begin_call() {
  g_last_launches = 0;
  g_kernel_log_len = 0;
}

struct Layout {
  int64_t es, ss;  // element stride, system stride (elements)
};

// Launch plan: kernel family and per-lane equation count R per (dtype, n, S).
struct Plan {
  bool cta;  // CTA kernels (W warps / system) or warp kernels
  int R;
  int W;     // cta only
};
Plan plan_for(int dtype, int64_t n, int64_t S = -1);

int device_sms(int dev);
int prefetch_mode();
int tma_mode();
int blocked_minb();
// Phase-stamp buffer for the next launch (nullptr unless TRIDIAG_PHASE_STAMPS=1;
// diagnostic only: the one device allocation the library ever makes).
long long* stamp_buffer(int64_t elems);
PFN_cuTensorMapEncodeTiled_v12000 encode_fn();

// Programmatic dependent launch (TRIDIAG_PDL, default 1): see pdl_entry().
int pdl_mode();
// Smaller warp-kernel CTAs for batches below 8 warps per SM (TRIDIAG_SMALL_CTA).
int small_cta_mode();
// L2 prefetch of the unit after the one a TMA kernel is copying (TRIDIAG_TMA_PF).
int tma_pf_mode();
// L2 prefetch of a CTA's first system before the dependent-launch wait
// (TRIDIAG_PREWAIT_PF, default 1).
int prewait_pf_mode();
// Column expansion pass unit order: 1 = chunk-major (TRIDIAG_COL_ORDER).
int col_order_mode();
// Vector paths for ragged contiguous rows: the TMA CTA kernel with 3-D maps
// and the warp kernel's per-lane 16-byte accesses (TRIDIAG_RAG_TMA, default 1).
int rag_tma_mode();
// Double-buffered CTA-kernel regions (TRIDIAG_CTA_DBUF, default 1).
int cta_dbuf_mode();
// TMA-fed column passes (TRIDIAG_COL_TMA, default 1).
int col_tma_mode();

// Launch with the programmatic-stream-serialization attribute (when enabled):
// the kernel's CTAs may be scheduled while the previous grid on the stream
// drains; every kernel of the library starts with pdl_entry(), which waits
// for that grid before touching global memory.
template <typename... KArgs, typename... Args>
cudaError_t launch_k(void (*kern)(KArgs...), dim3 grid, dim3 block, size_t smem, cudaStream_t st,
                     Args&&... args) {
  cudaLaunchConfig_t cfg = {};
  cfg.gridDim = grid;
  cfg.blockDim = block;
  cfg.dynamicSmemBytes = smem;
  cfg.stream = st;
  cudaLaunchAttribute at[1];
  at[0].id = cudaLaunchAttributeProgrammaticStreamSerialization;
  at[0].val.programmaticStreamSerializationAllowed = 1;
  cfg.attrs = at;
  cfg.numAttrs = pdl_mode() ? 1 : 0;
  if (g_kernel_log_len < kMaxKernelLog) g_kernel_log[g_kernel_log_len++] = reinterpret_cast<const void*>(kern);
  return cudaLaunchKernelEx(&cfg, kern, std::forward<Args>(args)...);
}

std::mutex& occ_mutex();
std::map<std::tuple<int, const void*, int, size_t>, int>& occ_cache();

// Resident CTAs per SM of `kernel` (cached per device / kernel / size).
template <typename K>
int occupancy(int dev, K kernel, int threads, size_t smem) {
  const void* key = reinterpret_cast<const void*>(kernel);
  std::lock_guard<std::mutex> lk(occ_mutex());
  auto& cache = occ_cache();
  auto it = cache.find({dev, key, threads, smem});
  if (it != cache.end()) return it->second;
  if (smem > 48 * 1024) cudaFuncSetAttribute(kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, 227 * 1024);
  int nb = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&nb, kernel, threads, smem) != cudaSuccess) nb = 0;
  cache[{dev, key, threads, smem}] = nb;
  return nb;
}

// Enqueue one solve of S systems (n = padded size, nr = real size, k CR
// levels) with the kernels of element type T and inner solver INNER.
// Explicitly instantiated in inst_<f32|f64>_<pcr|rd>.cu.
template <typename T, int INNER>
cudaError_t dispatch_t(const void* a, const void* b, const void* c, const void* d, void* x,
                       int64_t n, int64_t S, int k, cudaStream_t st, int dtype, int64_t nr,
                       Layout L);

// Large-n passes (tridiag_large.cuh, inst_large.cu).  which: 1 = reduction
// (a, b, c, d) -> (o0..o3), 2 = expansion writing x to o0 from the
// survivors' solution x2.  n = padded
// size of this level, n_real / ss = stored equations / system stride.
template <typename T>
int64_t large_chunk();
template <typename T>
cudaError_t large_pass(int which, const T* a, const T* b, const T* c, const T* d, T* o0, T* o1,
                       T* o2, T* o3, const T* x2, int64_t n, int64_t n_real, int64_t ss,
                       int64_t S, int kin, bool vec, T c_pad, cudaStream_t st);

// Interleaved-layout (ADI column sweep) passes (tridiag_colpass.cuh,
// inst_col.cu).  which: 1 = reduction (a, b, c, d) -> (o0..o3), 2 = expansion
// writing x to o0 from x2.  es = element stride of the input (system stride
// 1); row r of system s of the reduced arrays (and of x2) at r es2 + s ss2.
template <typename T>
int64_t col_chunk();
template <typename T>
cudaError_t col_pass(int which, const T* a, const T* b, const T* c, const T* d, T* o0, T* o1,
                     T* o2, T* o3, const T* x2, int64_t n, int64_t n_real, int64_t es, int64_t S,
                     int64_t es2, int64_t ss2, int kin, T c_pad, cudaStream_t st);

// The paper's own CR schedule (tridiag_paper.cuh, inst_paper.cu): Fig 9
// baseline only.  mode 0 = in place (bank conflicts), 1 = stride-one control.
template <typename T>
cudaError_t paper_cr(const T* a, const T* b, const T* c, const T* d, T* x, int64_t n, int64_t S,
                     int mode, cudaStream_t st);

}  // namespace tdg_host
