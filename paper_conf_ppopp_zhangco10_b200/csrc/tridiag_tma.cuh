// tridiag_tma.cuh -- TMA-pipelined CTA kernel for large systems (sm_100a).
//
// One CTA owns one system at a time (W warps, R equations per lane, as in
// tdg_cta_kernel).  Its four input arrays arrive through the Tensor Memory
// Accelerator: each array is viewed as a 2-D tensor of 64-byte rows (one row =
// one lane's R consecutive equations), copied with cp.async.bulk.tensor into a
// shared-memory stage with the 64-byte swizzle, which makes the lane-blocked
// 128-bit reads bank-conflict free (16-byte chunk q of row r sits at chunk
// q ^ ((r >> 1) & 3)).  The copy of the NEXT system is issued as soon as every
// thread has pulled the current one into registers, so HBM streams while the
// CTA runs its CR levels (the paper's block-level overlap, made
// explicit).  Completion is tracked by an mbarrier with expect-tx bytes.
#pragma once

#include <cuda.h>

#include "tridiag_kernels.cuh"

namespace tdg {

__device__ __forceinline__ uint32_t smem_u32(const void* p) {
  return static_cast<uint32_t>(__cvta_generic_to_shared(p));
}
__device__ __forceinline__ void mbar_init(uint64_t* bar, uint32_t count) {
  asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(bar)), "r"(count) : "memory");
  asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
}
__device__ __forceinline__ void mbar_arrive_expect_tx(uint64_t* bar, uint32_t bytes) {
  asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)),
               "r"(bytes)
               : "memory");
}
__device__ __forceinline__ void mbar_wait(uint64_t* bar, uint32_t parity) {
  uint32_t done = 0;
  do {
    asm volatile(
        "{\n .reg .pred p;\n mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2;\n"
        " selp.u32 %0, 1, 0, p;\n}\n"
        : "=r"(done)
        : "r"(smem_u32(bar)), "r"(parity)
        : "memory");
  } while (!done);
}
__device__ __forceinline__ void tma_load_2d(void* dst, const CUtensorMap* map, int c0, int c1,
                                            uint64_t* bar) {
  asm volatile(
      "cp.async.bulk.tensor.2d.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1, {%2, %3}], [%4];" ::"r"(
          smem_u32(dst)),
      "l"(reinterpret_cast<uint64_t>(map)), "r"(c0), "r"(c1), "r"(smem_u32(bar))
      : "memory");
}

__device__ __forceinline__ void tma_load_3d(void* dst, const CUtensorMap* map, int c0, int c1, int c2,
                                            uint64_t* bar) {
  asm volatile(
      "cp.async.bulk.tensor.3d.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1, {%2, %3, %4}], [%5];" ::"r"(
          smem_u32(dst)),
      "l"(reinterpret_cast<uint64_t>(map)), "r"(c0), "r"(c1), "r"(c2), "r"(smem_u32(bar))
      : "memory");
}

// L2 prefetch of a TMA box (no shared memory, no completion): issued for the
// unit after the one being copied, it keeps two units per CTA in flight to
// HBM while the stage holds only one.
__device__ __forceinline__ void tma_prefetch_2d(const CUtensorMap* map, int c0, int c1) {
  asm volatile("cp.async.bulk.prefetch.tensor.2d.L2.global.tile [%0, {%1, %2}];" ::"l"(
                   reinterpret_cast<uint64_t>(map)),
               "r"(c0), "r"(c1)
               : "memory");
}

// One lane's 64-byte row out of the 64B-swizzled stage: 16-byte chunk ch is
// stored at chunk ch ^ sw, sw = (row >> 1) & 3 (CU_TENSOR_MAP_SWIZZLE_64B).
template <typename T, int R>
__device__ __forceinline__ void read_row(const unsigned char* row, int sw, T (&v)[R]) {
  constexpr int E = 16 / (int)sizeof(T);
#pragma unroll
  for (int ch = 0; ch < 4; ++ch) {
    const unsigned char* src = row + ((ch ^ sw) << 4);
    if constexpr (sizeof(T) == 4) {
      const float4 t = *reinterpret_cast<const float4*>(src);
      v[ch * E + 0] = t.x; v[ch * E + 1] = t.y; v[ch * E + 2] = t.z; v[ch * E + 3] = t.w;
    } else {
      const double2 t = *reinterpret_cast<const double2*>(src);
      v[ch * E + 0] = t.x; v[ch * E + 1] = t.y;
    }
  }
}

// Bytes of the TMA stage (a, b, c, d of one system), rounded to 1 KB.
template <typename T>
__host__ __device__ constexpr uint32_t tma_stage_bytes(int R, int W) {
  return (uint32_t)(((4u * 32u * W * R * sizeof(T)) + 1023u) & ~1023u);
}

// KB = -1: k >= log2 R (register path); KB >= 0: RD inner with k = KB
// (cta_blocked_rd).
// RAG = true: ragged and / or pitched rows (n_real <= n, system stride ss >=
// n_real, ss T a multiple of 16 B).  The tensor maps are 3-D
// {R, ceil(n_real / R), S} with strides {R T, ss T}: a system's 64-byte rows,
// the last one possibly running past the system, rows past it zero-filled by
// TMA; equations i >= n_real become the padding equations of reading R26 in
// registers and only the real ones are stored.
template <typename T, int R, int W, int INNER, int KB, bool RAG = false>
__global__ void __launch_bounds__(W * 32)
tdg_cta_tma_kernel(const __grid_constant__ CUtensorMap tmA, const __grid_constant__ CUtensorMap tmB,
                   const __grid_constant__ CUtensorMap tmC, const __grid_constant__ CUtensorMap tmD,
                   T* x, int n, long long S, int k, int dbuf, int pf, int n_real, long long ss,
                   long long* stamps) {
  static_assert(R * sizeof(T) == 64, "TMA stage rows are 64 bytes");
  constexpr int P = 32 * W;
  constexpr int LR = ilog2c(R);
  constexpr int ROWS = P > 256 ? 256 : P;  // rows per TMA box (box dims <= 256)
  constexpr int NBOX = P / ROWS;
  // L2 prefetch of this CTA's first system BEFORE waiting for the previous
  // grid: a prefetch returns nothing to the SM and L2 is the point of
  // coherence, so a later write of the previous grid still wins; it only
  // moves the first load's DRAM latency into the previous grid's tail (the
  // launch ramp of a back-to-back sweep).  The stage load itself follows the
  // wait.
  if (!RAG && (pf & 2) && threadIdx.x == 0 && blockIdx.x < S) {
#pragma unroll
    for (int bx = 0; bx < NBOX; ++bx) {
      tma_prefetch_2d(&tmA, 0, (int)(blockIdx.x * P + bx * ROWS));
      tma_prefetch_2d(&tmB, 0, (int)(blockIdx.x * P + bx * ROWS));
      tma_prefetch_2d(&tmC, 0, (int)(blockIdx.x * P + bx * ROWS));
      tma_prefetch_2d(&tmD, 0, (int)(blockIdx.x * P + bx * ROWS));
    }
  }
  pdl_entry();
  constexpr uint32_t ARR_BYTES = P * R * sizeof(T);
  constexpr uint32_t STAGE = tma_stage_bytes<T>(R, W);
  extern __shared__ __align__(1024) unsigned char smem_raw[];
  unsigned char* stage = smem_raw;
  uint64_t* bar = reinterpret_cast<uint64_t*>(smem_raw + STAGE);
  T* heads0 = reinterpret_cast<T*>(smem_raw + STAGE + 16);
  const int ls = threadIdx.x;

  const CUtensorMap* maps[4] = {&tmA, &tmB, &tmC, &tmD};
  auto issue = [&](long long sys) {
    mbar_arrive_expect_tx(bar, 4 * ARR_BYTES);
#pragma unroll
    for (int q = 0; q < 4; ++q)
#pragma unroll
      for (int bx = 0; bx < NBOX; ++bx)
        if constexpr (RAG)
          tma_load_3d(stage + q * ARR_BYTES + bx * ROWS * 64, maps[q], 0, bx * ROWS, (int)sys, bar);
        else
          tma_load_2d(stage + q * ARR_BYTES + bx * ROWS * 64, maps[q], 0,
                      (int)(sys * P + bx * ROWS), bar);
    if (!RAG && (pf & 1) && sys + gridDim.x < S) {
#pragma unroll
      for (int q = 0; q < 4; ++q)
#pragma unroll
        for (int bx = 0; bx < NBOX; ++bx)
          tma_prefetch_2d(maps[q], 0, (int)((sys + gridDim.x) * P + bx * ROWS));
    }
  };
  if (ls == 0) {
    mbar_init(bar, 1);
    if (blockIdx.x < S) issue(blockIdx.x);
  }
  __syncthreads();

  uint32_t parity = 0;
  int it = 0;
  for (long long sys = blockIdx.x; sys < S; sys += gridDim.x, ++it) {
    // dbuf > 0: the heads / survivor regions alternate between two copies of
    // dbuf elements by system parity, so the next system's writes cannot
    // race this system's reads (they are separated by the next system's
    // first barrier) and no barrier is needed at the end of a system
    T* heads = heads0 + ((dbuf > 0 && (it & 1)) ? dbuf : 0);
    // phase stamps (diagnostic, NEXT f4): warp 0 of every CTA, first
    // kStampSystems systems: [0] wait for the stage, [1] data arrived,
    // [2] in-lane forward + next-warp heads, [3] lane-level forward,
    // [4] survivors solved, [5] lane-level backward, [6] in-lane backward,
    // [7] store issued
    Stamp stp;
    if (stamps != nullptr && ls < 32 && it < kStampSystems)
      stp.p = stamps + ((long long)blockIdx.x * kStampSystems + it) * kStampSlots;
    stp.mark(0);
    mbar_wait(bar, parity);
    stp.mark(1);
    parity ^= 1;
    T ra[R], rb[R], rc[R], rd[R];
    const int sw = (ls >> 1) & 3;
    read_row<T, R>(stage + 0 * ARR_BYTES + ls * 64, sw, ra);
    read_row<T, R>(stage + 1 * ARR_BYTES + ls * 64, sw, rb);
    read_row<T, R>(stage + 2 * ARR_BYTES + ls * 64, sw, rc);
    read_row<T, R>(stage + 3 * ARR_BYTES + ls * 64, sw, rd);
    if constexpr (RAG) {
      const int i0 = ls * R;
      if (i0 + R >= n_real) {  // this lane holds c_{n_real-1} or padding rows
        const T c_pad = INNER == kRD ? T(1) : T(0);
#pragma unroll
        for (int t = 0; t < R; ++t) {
          if (i0 + t >= n_real) { ra[t] = T(0); rb[t] = T(1); rc[t] = c_pad; rd[t] = T(0); }
          if (i0 + t == n_real - 1) rc[t] = c_pad;
        }
      }
    }
    if (ls == 0) ra[0] = T(0);
    if (ls == P - 1) rc[R - 1] = T(0);
    const long long next = sys + gridDim.x;
    // every thread has read the stage once the heads barrier is passed
    constexpr int KIN = KB >= 0 ? KB : LR;
    cta_inlane_forward<T, R, W>(ra, rb, rc, rd, KIN, heads, [&] {
      if (ls == 0 && next < S) issue(next);
    });
    stp.mark(2);
    T xprev;
    if constexpr (KB >= 0) {
      xprev = cta_blocked_rd<T, R, W, (KB >= 0 ? KB : 0)>(ra, rb, rc, rd, heads + W * (LR > 0 ? LR : 1) * 4);
    } else {
      xprev = cta_register_path<T, R, W, INNER>(ra, rb, rc, rd, k, heads, stp);
    }
    stp.mark(5);
    inlane_backward<T, R>(ra, rb, rc, rd, KIN, xprev);
    stp.mark(6);
    if constexpr (RAG) {
      T* p = x + (size_t)sys * (size_t)ss + (size_t)ls * R;
      if (ls * R + R <= n_real) {
        // 16-byte aligned (n_real T and R T are multiples of 16 B): full
        // 32-byte sectors where the block allows (store_block16)
        store_block16<T, R>(p, rd);
      } else {
#pragma unroll
        for (int t = 0; t < R; ++t)
          if (ls * R + t < n_real) p[t] = rd[t];
      }
    } else {
      store_block<T, R>(x + (size_t)sys * (size_t)n + (size_t)ls * R, rd, true);
    }
    stp.mark(7);
    if (dbuf == 0) __syncthreads();  // heads / survivor regions are reused by the next system
  }
}

// Dynamic shared memory of tdg_cta_tma_kernel: stage + mbarrier + the
// register path's regions (heads, lane heads, survivors, inner).
// copies = 2: double-buffered regions (the kernel's dbuf), each rounded to 16 B.
template <typename T>
inline size_t cta_tma_region_bytes(int R, int W, int inner, int k) {
  return (cta_smem_bytes<T>(R, W, inner, k) + 15) & ~size_t(15);
}
template <typename T>
inline size_t cta_tma_smem_bytes(int R, int W, int inner, int k, int copies = 1) {
  return tma_stage_bytes<T>(R, W) + 16 + copies * cta_tma_region_bytes<T>(R, W, inner, k);
}

}  // namespace tdg
