// tridiag_ileave.cuh -- interleaved layouts (NEXT f1 of SURVEY.md 8(f)).
//
// ADI, the paper's headline application, sweeps a
// grid along rows (contiguous systems) and then along columns: element i of
// system s at ptr[s + i * es] (system stride 1, element stride es >= S).  The
// coalescing is the reverse of the contiguous layout, so this kernel stages a
// tile of G consecutive systems (G = 8: a 32-byte fp32 / 64-byte fp64 row
// segment per equation index) through shared memory:
//   * load: consecutive threads read consecutive systems of one row, so every
//     warp request is whole 32-byte sectors;
//   * the tile is stored at offset(r, g) = r*G + g + (r >> 4), which makes the
//     lane-blocked column reads of the solve (lane l reads rows l*R..l*R+R-1
//     of its system) bank-conflict free for R = 16;
//   * each system then runs exactly the contiguous kernel's warp_solve
//     (registers + shuffles), x goes back through the tile and out with the
//     same coalesced pattern.
#pragma once

#include "tridiag_kernels.cuh"

namespace tdg {

__device__ __forceinline__ int ilv_off(int r, int g, int G) { return r * G + g + (r >> 4); }

// Elements of one array's tile for G systems of n_pad rows.
__host__ __device__ constexpr int ilv_tile_elems(int n_pad, int G) {
  return n_pad * G + (n_pad >> 4) + G;
}

// ---- asynchronous 4 / 8-byte global -> shared copies (LDGSTS) ----
template <typename T>
__device__ __forceinline__ void cp_async_elem(T* dst, const T* src) {
  const unsigned s = (unsigned)__cvta_generic_to_shared(dst);
  if constexpr (sizeof(T) == 4)
    asm volatile("cp.async.ca.shared.global [%0], [%1], 4;" ::"r"(s), "l"(src) : "memory");
  else
    asm volatile("cp.async.ca.shared.global [%0], [%1], 8;" ::"r"(s), "l"(src) : "memory");
}
__device__ __forceinline__ void cp_async_commit() { asm volatile("cp.async.commit_group;" ::: "memory"); }
__device__ __forceinline__ void cp_async_wait_all() { asm volatile("cp.async.wait_group 0;" ::: "memory"); }

// Tile geometry.  NT = 2^ilv_log_threads threads; P = 2^LP lanes per
// system, G = NT / P systems per tile, ROWS = P R rows.  LP >= 0 makes every shared-memory
// offset a compile-time immediate (the kernel is integer-bound otherwise);
// LP = -1 takes log2P at run time.
// 512 threads (G = 16 systems, 64-byte fp32 row segments) at P = 32, where
// 32-byte segments over-fetch from DRAM; 256 threads for smaller P.
__host__ __device__ constexpr int ilv_log_threads(int lp) { return lp == 5 ? 9 : 8; }
// LNT >= 0: 2^LNT threads instead (the narrow-tile variant for batches with
// fewer default tiles than SMs: the paper's literal 512 x 512 column sweep has
// 32 tiles of 16 systems; tiles of 16-byte row segments give 128)
template <int LP, int LNT = -1>
struct IlvGeom {
  int lp, lnt;
  __device__ __forceinline__ explicit IlvGeom(int log2P)
      : lp(LP >= 0 ? LP : log2P), lnt(LNT >= 0 ? LNT : ilv_log_threads(LP >= 0 ? LP : log2P)) {}
  __device__ __forceinline__ int P() const { return 1 << lp; }
  __device__ __forceinline__ int lg() const { return lnt - lp; }
  __device__ __forceinline__ int G() const { return 1 << (lnt - lp); }
};

// Issue the copies of one tile: rows [row0, row0 + ROWS) of systems
// [t0, t0 + G) into the padded tile.  Thread tid owns system g = tid % G and
// rows r0 + P j (r0 = tid / G < P, j < R), so consecutive threads read
// consecutive systems of a row (whole 32-byte sectors); every offset advances
// by a constant.  Padding (rows >= n_real, systems >= S, reading R26) and
// c_{n_real-1} <- c_pad are plain shared stores.
template <typename T, int R, int LP, bool COPY_D, int LNT = -1>
__device__ __forceinline__ void ilv_issue(const T* a, const T* b, const T* c, const T* d, T* tile,
                                          int TE, long long t0, long long S, int row0, int n_real,
                                          long long es, const IlvGeom<LP, LNT>& Gm, T c_pad) {
  const int G = Gm.G(), P = Gm.P();
  const int g = threadIdx.x & (G - 1);
  const int r0 = threadIdx.x >> Gm.lg();
  const bool sys_ok = t0 + g < S;
  const long long off0 = t0 + g + (long long)(row0 + r0) * es;
  const T* pa = a + off0;
  const T* pb = b + off0;
  const T* pc = c + off0;
  const T* pd = d + off0;
  const long long step = (long long)P * es;
  unsigned so = (unsigned)__cvta_generic_to_shared(tile) + (unsigned)(r0 * G + g) * sizeof(T);
  const unsigned TB = (unsigned)TE * sizeof(T);
  const bool all_rows = row0 + P * R <= n_real - 1;  // no padding row, no c_{n_real-1} here
  if (sys_ok && all_rows) {
    // the common case (every row real, the system exists): branch-free copies
#pragma unroll 4
    for (int j = 0; j < R; ++j, pa += step, pb += step, pc += step, pd += step) {
      const int r = r0 + P * j;
      const unsigned sj = so + (unsigned)(P * j * G + (r >> 4)) * sizeof(T);
      if constexpr (sizeof(T) == 4) {
        asm volatile("cp.async.ca.shared.global [%0], [%1], 4;" ::"r"(sj), "l"(pa) : "memory");
        asm volatile("cp.async.ca.shared.global [%0], [%1], 4;" ::"r"(sj + TB), "l"(pb) : "memory");
        asm volatile("cp.async.ca.shared.global [%0], [%1], 4;" ::"r"(sj + 2 * TB), "l"(pc) : "memory");
        if (COPY_D)
          asm volatile("cp.async.ca.shared.global [%0], [%1], 4;" ::"r"(sj + 3 * TB), "l"(pd) : "memory");
      } else {
        asm volatile("cp.async.ca.shared.global [%0], [%1], 8;" ::"r"(sj), "l"(pa) : "memory");
        asm volatile("cp.async.ca.shared.global [%0], [%1], 8;" ::"r"(sj + TB), "l"(pb) : "memory");
        asm volatile("cp.async.ca.shared.global [%0], [%1], 8;" ::"r"(sj + 2 * TB), "l"(pc) : "memory");
        if (COPY_D)
          asm volatile("cp.async.ca.shared.global [%0], [%1], 8;" ::"r"(sj + 3 * TB), "l"(pd) : "memory");
      }
    }
    cp_async_commit();
    return;
  }
#pragma unroll 4
  for (int j = 0; j < R; ++j, pa += step, pb += step, pc += step, pd += step) {
    // (r0 + P j) >> 4 == (P j) >> 4 + (r0 >> 4) for P | 16 or 16 | P
    const int r = r0 + P * j;
    const unsigned sj = so + (unsigned)(P * j * G + (r >> 4)) * sizeof(T);
    const int row = row0 + r;
    if (sys_ok && (all_rows || row < n_real)) {
      if constexpr (sizeof(T) == 4) {
        asm volatile("cp.async.ca.shared.global [%0], [%1], 4;" ::"r"(sj), "l"(pa) : "memory");
        asm volatile("cp.async.ca.shared.global [%0], [%1], 4;" ::"r"(sj + TB), "l"(pb) : "memory");
        if (all_rows || row != n_real - 1)
          asm volatile("cp.async.ca.shared.global [%0], [%1], 4;" ::"r"(sj + 2 * TB), "l"(pc) : "memory");
        if (COPY_D)
          asm volatile("cp.async.ca.shared.global [%0], [%1], 4;" ::"r"(sj + 3 * TB), "l"(pd) : "memory");
      } else {
        asm volatile("cp.async.ca.shared.global [%0], [%1], 8;" ::"r"(sj), "l"(pa) : "memory");
        asm volatile("cp.async.ca.shared.global [%0], [%1], 8;" ::"r"(sj + TB), "l"(pb) : "memory");
        if (all_rows || row != n_real - 1)
          asm volatile("cp.async.ca.shared.global [%0], [%1], 8;" ::"r"(sj + 2 * TB), "l"(pc) : "memory");
        if (COPY_D)
          asm volatile("cp.async.ca.shared.global [%0], [%1], 8;" ::"r"(sj + 3 * TB), "l"(pd) : "memory");
      }
      if (!all_rows && row == n_real - 1) tile[2 * TE + ilv_off(r, g, G)] = c_pad;
    } else {
      const int o = ilv_off(r, g, G);
      tile[o] = T(0); tile[TE + o] = T(1); tile[2 * TE + o] = c_pad;
      if (COPY_D) tile[3 * TE + o] = T(0);
    }
  }
  cp_async_commit();
}

// Write the tile's x back: same element mapping, coalesced.
template <typename T, int R, int LP, int LNT = -1>
__device__ __forceinline__ void ilv_writeback(T* x, const T* tX, long long t0, long long S, int row0,
                                              int n_real, long long es, const IlvGeom<LP, LNT>& Gm) {
  const int G = Gm.G(), P = Gm.P();
  const int g = threadIdx.x & (G - 1);
  const int r0 = threadIdx.x >> Gm.lg();
  if (t0 + g >= S) return;
  T* dst = x + t0 + g + (long long)(row0 + r0) * es;
  const long long step = (long long)P * es;
  const T* srcp = tX + r0 * G + g;
  const bool all_rows = row0 + P * R <= n_real;
  if (all_rows) {
#pragma unroll 4
    for (int j = 0; j < R; ++j, dst += step) {
      const int r = r0 + P * j;
      *dst = srcp[P * j * G + (r >> 4)];
    }
    return;
  }
#pragma unroll 4
  for (int j = 0; j < R; ++j, dst += step) {
    const int r = r0 + P * j;
    if (all_rows || row0 + r < n_real) *dst = srcp[P * j * G + (r >> 4)];
  }
}

// Interleaved solve, n <= 32 R: NT threads, P = n / R lanes per system,
// G = NT / P systems per tile (NT = 512 at P = 32: 64-byte fp32 / 128-byte
// fp64 row segments; else 256).  One input tile plus an x tile: as soon as the
// lanes hold tile i in registers the copies of tile i+1 are issued into the
// same buffer (no registers held while they fly) and overlap the solve; x
// leaves through the x tile.  5 NT R elements of shared memory: 1 CTA of 16
// warps (NT = 512) or 2 CTAs of 8 warps per SM.
template <int LP, int LNT>
__host__ __device__ constexpr int ilv_threads() { return LNT >= 0 ? (1 << (LNT >= 0 ? LNT : 0)) : (LP == 5 ? 512 : 256); }
template <int LP, int LNT>
__host__ __device__ constexpr int ilv_min_blocks() {
  return LNT >= 0 ? (65536 / 128) / ilv_threads<LP, LNT>() : (LP == 5 ? 1 : 2);
}
template <typename T, int R, int INNER, int KB, int LP, int LNT = -1>
__global__ void __launch_bounds__(ilv_threads<LP, LNT>(), ilv_min_blocks<LP, LNT>())
tdg_ileave_kernel(const T* __restrict__ a, const T* __restrict__ b, const T* __restrict__ c,
                  const T* d, T* x, int n, long long S, int k, int log2P, int n_real, T c_pad,
                  long long es) {
  pdl_entry();
  extern __shared__ __align__(1024) unsigned char smem_raw[];
  T* tile = reinterpret_cast<T*>(smem_raw);
  const IlvGeom<LP, LNT> Gm(log2P);
  const int G = Gm.G(), P = Gm.P();
  const int TE = ilv_tile_elems(P * R, G);
  T* tX = tile + 4 * TE;
  // (the tiles leave no room for the cyclic PCR relayout's scratch: the
  // block-layout PCR with shuffles runs here)
  T* pcr_scr = nullptr;
  const int g = threadIdx.x >> Gm.lp;
  const int ls = threadIdx.x & (P - 1);
  // lane-blocked rows ls R + q of system g: offset base + q G (R | 16 or 16 | R)
  const int base = ls * R * G + g + ((ls * R) >> 4);
  const long long tiles = (S + G - 1) / G;
  long long t = blockIdx.x;
  if (t < tiles) ilv_issue<T, R, LP, true, LNT>(a, b, c, d, tile, TE, t * G, S, 0, n_real, es, Gm, c_pad);
  for (; t < tiles; t += gridDim.x) {
    cp_async_wait_all();
    __syncthreads();  // tile t landed; the x tile's previous write-back is done
    T ra[R], rb[R], rc[R], rd[R];
#pragma unroll
    for (int q = 0; q < R; ++q) {
      const int o = base + q * G;
      ra[q] = tile[o]; rb[q] = tile[TE + o]; rc[q] = tile[2 * TE + o]; rd[q] = tile[3 * TE + o];
    }
    __syncthreads();  // every lane holds its rows: the tile buffer is free
    const long long tn = t + gridDim.x;
    if (tn < tiles) ilv_issue<T, R, LP, true, LNT>(a, b, c, d, tile, TE, tn * G, S, 0, n_real, es, Gm, c_pad);
    if (ls == 0) ra[0] = T(0);
    if (ls == P - 1) rc[R - 1] = T(0);
    warp_solve<T, R, INNER, KB>(ra, rb, rc, rd, k, ls, P, Stamp(), pcr_scr);
#pragma unroll
    for (int q = 0; q < R; ++q) tX[base + q * G] = rd[q];
    __syncthreads();
    ilv_writeback<T, R, LP, LNT>(x, tX, t * G, S, 0, n_real, es, Gm);
  }
}

}  // namespace tdg
