// tridiag_colpass.cuh -- CR reduction / expansion passes for interleaved
// (ADI column-sweep) layouts: element i of system s at ptr[s + i * es].
//
// ADI sweeps a grid along rows and then along columns (P:L105-107,
// P:L145-147).  A column system of n = 4096 equations is 64 KB (fp32) of
// input; the coalesced unit of the column layout is a row segment of
// consecutive systems, and 8 or more systems of that size do not fit on one
// SM.  So the column sweep at n > 32 R reuses the large-n scheme (P:L656-659,
// tridiag_large.cuh) with a layout-native work unit:
//
//   * a CTA of W warps owns 32 consecutive systems (lane = system) and a
//     chunk of CH = W R consecutive rows; warp w holds rows w R .. w R + R - 1
//     of its lane's system.  Every global access of a warp is one row segment
//     of 32 systems (128 B fp32 / 256 B fp64): fully coalesced, no staging.
//   * the reduction pass runs KIN <= log2 R in-lane CR levels (the on-chip
//     kernels' inlane_forward_interior / inlane_tail_chain, so every update is
//     the same correctly rounded operation sequence) and writes the n >> KIN
//     survivors of each system to the workspace: row r of system s at
//     r es2 + s ss2 -- interleaved (es2 = S, ss2 = 1) for a further column
//     pass, or transposed into contiguous rows (es2 = 1, ss2 = n >> KIN) by
//     the last pass, whose reduced systems the fast row kernels then solve.  A
//     warp's tail needs the next warp's head equations (shared memory); the
//     last warp needs the next chunk's.  Each CTA walks a contiguous range of
//     units in descending chunk order, so those are the heads the previous
//     unit's warp 0 produced (carried in shared memory); only the first unit
//     of a CTA computes them from the next chunk's first R rows.
//   * the expansion pass recomputes the interior forward levels (the tail
//     chain only changes the tail, a survivor whose x comes from the reduced
//     solve, so no heads are needed), reads the survivors' x and runs the
//     in-lane back-substitution.  A unit reads only its own rows,
//     so x may alias d.
//
// The last pass's reduced systems (contiguous rows, at most tridiag_max_n
// equations) are solved by the row kernels (warp / TMA CTA kernels).
#pragma once

#include "tridiag_tma.cuh"  // mbarrier / cp.async.bulk.tensor helpers, Stamp

// CTAs per SM the TMA expansion pass asks for: its 64 KB stage allows 3, which
// caps registers at 80 -- a gain for fp64 (255 vs 267 us at 4096^2), a loss
// for fp32 (61 vs 59 us per pass), so fp32 keeps 2.
#ifndef TDG_COL_EXPAND_MINB
#define TDG_COL_EXPAND_MINB(T) (sizeof(T) == 8 ? 3 : 2)
#endif

namespace tdg {

// R rows of one array of column s, rows >= n_real padded (reading R26) and
// c_{n_real-1} <- last_val; columns s >= S (a ragged last group) are padding.
template <typename T, int R>
__device__ __forceinline__ void col_load(const T* p, long long es, long long s, bool sok,
                                         long long i0, long long n_real, T pad, T last_val,
                                         bool set_last, T (&v)[R]) {
  const T* q = p + s + i0 * es;
  if (sok && i0 + R < n_real) {
#pragma unroll
    for (int t = 0; t < R; ++t) v[t] = q[t * es];
  } else {
#pragma unroll
    for (int t = 0; t < R; ++t) {
      const long long i = i0 + t;
      v[t] = (sok && i < n_real) ? q[t * es] : pad;
      if (set_last && i == n_real - 1) v[t] = last_val;
    }
  }
}

template <typename T, int R>
__device__ __forceinline__ void col_load4(const T* a, const T* b, const T* c, const T* d,
                                          long long es, long long s, bool sok, long long i0,
                                          long long n_real, T c_pad, T (&ra)[R], T (&rb)[R],
                                          T (&rc)[R], T (&rd)[R]) {
  col_load<T, R>(a, es, s, sok, i0, n_real, T(0), T(0), false, ra);
  col_load<T, R>(b, es, s, sok, i0, n_real, T(1), T(0), false, rb);
  col_load<T, R>(c, es, s, sok, i0, n_real, c_pad, c_pad, true, rc);
  col_load<T, R>(d, es, s, sok, i0, n_real, T(0), T(0), false, rd);
}

// Heads of one lane: NH levels x (a, 1/b, c, d); shared layout [NH][4][32]
// (lane-contiguous: conflict-free).
template <typename T, int R>
__host__ __device__ constexpr int col_heads_elems() { return (ilog2c(R) > 0 ? ilog2c(R) : 1) * 4 * 32; }

template <typename T, int R, int KIN>
__device__ __forceinline__ void col_put_heads(T* pg, int lane, const T (&a)[R], const T (&b)[R],
                                              const T (&c)[R], const T (&d)[R]) {
#pragma unroll
  for (int l = 1; l <= KIN; ++l) {
    const int t = (1 << (l - 1)) - 1;
    T* h = pg + (l - 1) * 128 + lane;
    h[0] = a[t]; h[32] = b[t]; h[64] = c[t]; h[96] = d[t];
  }
}
template <typename T, int R, int KIN>
__device__ __forceinline__ void col_get_heads(const T* pg, int lane, Heads<T, R>& H) {
#pragma unroll
  for (int l = 1; l <= KIN; ++l) {
    const T* h = pg + (l - 1) * 128 + lane;
    H.a[l - 1] = h[0]; H.rb[l - 1] = h[32]; H.c[l - 1] = h[64]; H.d[l - 1] = h[96];
  }
}

// Dynamic shared memory of the reduction pass: two pages of W warps' heads
// plus two carry pages.
template <typename T, int R, int W>
__host__ __device__ constexpr size_t col_reduce_smem() {
  return (size_t)(2 * W + 2) * col_heads_elems<T, R>() * sizeof(T);
}

// Reduction pass: (a, b, c, d) interleaved with element stride es ->
// survivors (a2, b2, c2, d2) interleaved with element stride es2, n >> KIN rows.
template <typename T, int R, int W, int KIN>
__global__ void __launch_bounds__(W * 32, 2)
tdg_col_reduce_kernel(const T* __restrict__ a, const T* __restrict__ b, const T* __restrict__ c,
                      const T* __restrict__ d, T* __restrict__ a2, T* __restrict__ b2,
                      T* __restrict__ c2, T* __restrict__ d2, long long n, long long n_real,
                      long long es, long long S, long long es2, long long ss2, T c_pad) {
  pdl_entry();
  constexpr int HE = col_heads_elems<T, R>();
  constexpr int Q = R >> KIN;
  constexpr long long CH = (long long)W * R;
  extern __shared__ __align__(1024) unsigned char smem_raw[];
  T* pages = reinterpret_cast<T*>(smem_raw);  // [2][W][HE]
  T* carry = pages + 2 * W * HE;              // [2][HE]
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  const long long C = n / CH;
  const long long U = ((S + 31) >> 5) * C;
  const long long lo = (long long)blockIdx.x * U / gridDim.x;
  const long long hi = ((long long)blockIdx.x + 1) * U / gridDim.x;
  int j = 0;
  for (long long u = hi - 1; u >= lo; --u, ++j) {
    const long long g = u / C, ch = u - g * C;
    const long long s = g * 32 + lane;
    const bool sok = s < S;
    T* pg = pages + (j & 1) * W * HE;
    T* cin = carry + ((j + 1) & 1) * HE;  // heads of chunk ch + 1 (warp 0)
    if (j == 0 && ch + 1 < C && w == 0) {
      // first unit of this CTA: the next chunk's heads from its first R rows
      T ha[R], hb[R], hc[R], hd[R];
      col_load4<T, R>(a, b, c, d, es, s, sok, (ch + 1) * CH, n_real, c_pad, ha, hb, hc, hd);
      inlane_forward_interior<T, R, true>(ha, hb, hc, hd, KIN);
      col_put_heads<T, R, KIN>(cin, lane, ha, hb, hc, hd);
    }
    const long long i0 = ch * CH + (long long)w * R;
    T ra[R], rb[R], rc[R], rd[R];
    col_load4<T, R>(a, b, c, d, es, s, sok, i0, n_real, c_pad, ra, rb, rc, rd);
    if (i0 == 0) ra[0] = T(0);
    if (i0 + R == n) rc[R - 1] = T(0);
    inlane_forward_interior<T, R, true>(ra, rb, rc, rd, KIN);
    col_put_heads<T, R, KIN>(pg + w * HE, lane, ra, rb, rc, rd);
    __syncthreads();
    Heads<T, R> H;
    if (w + 1 < W) {
      col_get_heads<T, R, KIN>(pg + (w + 1) * HE, lane, H);
    } else if (ch + 1 < C) {
      col_get_heads<T, R, KIN>(cin, lane, H);
    } else {  // end of the system
#pragma unroll
      for (int l = 0; l < KIN; ++l) { H.a[l] = T(0); H.rb[l] = T(0); H.c[l] = T(0); H.d[l] = T(0); }
    }
    // warp 0's heads are what the next unit (chunk ch - 1) needs
    if (w == 0) col_put_heads<T, R, KIN>(carry + (j & 1) * HE, lane, ra, rb, rc, rd);
    inlane_tail_chain<T, R>(ra, rb, rc, rd, KIN, H);
    if (sok) {
      const long long o = (i0 >> KIN) * es2 + s * ss2;
#pragma unroll
      for (int q = 0; q < Q; ++q) {
        const int t = ((q + 1) << KIN) - 1;
        a2[o + q * es2] = ra[t]; b2[o + q * es2] = rb[t];
        c2[o + q * es2] = rc[t]; d2[o + q * es2] = rd[t];
      }
    }
  }
}

// Expansion pass: recompute the interior forward levels, take the survivors'
// x from x2 (interleaved, stride es2), back-substitute, write x (stride es).
template <typename T, int R, int W, int KIN>
__global__ void __launch_bounds__(W * 32, 2)
tdg_col_expand_kernel(const T* __restrict__ a, const T* __restrict__ b, const T* __restrict__ c,
                      const T* d, T* x, const T* __restrict__ x2, long long n, long long n_real,
                      long long es, long long S, long long es2, long long ss2, T c_pad) {
  pdl_entry();
  constexpr int Q = R >> KIN;
  constexpr long long CH = (long long)W * R;
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  const long long C = n / CH;
  const long long U = ((S + 31) >> 5) * C;
  for (long long u = blockIdx.x; u < U; u += gridDim.x) {
    const long long g = u / C, ch = u - g * C;
    const long long s = g * 32 + lane;
    const bool sok = s < S;
    const long long i0 = ch * CH + (long long)w * R;
    T ra[R], rb[R], rc[R], rd[R];
    col_load4<T, R>(a, b, c, d, es, s, sok, i0, n_real, c_pad, ra, rb, rc, rd);
    if (i0 == 0) ra[0] = T(0);
    if (i0 + R == n) rc[R - 1] = T(0);
    T xs[Q];
    T xprev = T(0);
    if (sok) {
      const long long o = (i0 >> KIN) * es2 + s * ss2;
#pragma unroll
      for (int q = 0; q < Q; ++q) xs[q] = x2[o + q * es2];
      if (i0 > 0) xprev = x2[o - es2];
    } else {
#pragma unroll
      for (int q = 0; q < Q; ++q) xs[q] = T(0);
    }
    inlane_forward_interior<T, R, true>(ra, rb, rc, rd, KIN);
#pragma unroll
    for (int q = 0; q < Q; ++q) rd[((q + 1) << KIN) - 1] = xs[q];
    inlane_backward<T, R>(ra, rb, rc, rd, KIN, xprev);
    if (sok) {
      T* p = x + s + i0 * es;
      if (i0 + R <= n_real) {
#pragma unroll
        for (int t = 0; t < R; ++t) p[t * es] = rd[t];
      } else {
#pragma unroll
        for (int t = 0; t < R; ++t)
          if (i0 + t < n_real) p[t * es] = rd[t];
      }
    }
  }
}

// ---------------------------------------------------------------------------
// TMA-fed versions (the default when the layout allows a tensor map: 16-byte
// aligned bases and row pitch).  A unit's 32 systems x CH rows of a, b, c, d
// arrive as four 2-D boxes {32 systems, CH rows} (128 B / 256 B rows, no
// swizzle: warp w's lanes read one row at a time, consecutive banks) by
// cp.async.bulk.tensor into a shared stage; the copy of the next unit is
// issued as soon as every thread holds the current one in registers, so HBM
// streams during the CR levels (2 CTAs per SM).  Out-of-range rows / systems
// arrive as zeros and are replaced by the padding equations in registers.
// ---------------------------------------------------------------------------
template <typename T, int R, int W>
__host__ __device__ constexpr uint32_t col_stage_bytes() { return 4u * 32u * W * R * sizeof(T); }

template <typename T, int R, int W>
__host__ __device__ constexpr size_t col_reduce_tma_smem() {
  // one page of W warps' heads (the unit-start barrier that frees the stage
  // also orders the next unit's head stores after this unit's reads) plus
  // the two carry pages
  return col_stage_bytes<T, R, W>() + 16 + (size_t)(W + 2) * col_heads_elems<T, R>() * sizeof(T) +
         (size_t)4 * W * 32 * sizeof(T);  // survivor tile of the transposed store
}

template <typename T, int R, int W>
__device__ __forceinline__ void col_read_stage(const unsigned char* stage, int w, int lane,
                                               T (&ra)[R], T (&rb)[R], T (&rc)[R], T (&rd)[R]) {
  constexpr int AE = 32 * W * R;
  const T* st = reinterpret_cast<const T*>(stage) + (w * R) * 32 + lane;
#pragma unroll
  for (int t = 0; t < R; ++t) {
    ra[t] = st[t * 32]; rb[t] = st[AE + t * 32]; rc[t] = st[2 * AE + t * 32]; rd[t] = st[3 * AE + t * 32];
  }
}

// Padding of the rows >= n_real (reading R26: a = 0, b = 1, c = c_pad, d = 0,
// c_{n_real-1} = c_pad) and of systems s >= S (same identity rows).
template <typename T, int R>
__device__ __forceinline__ void col_fix_ragged(bool sok, long long i0, long long n_real, T c_pad,
                                               T (&ra)[R], T (&rb)[R], T (&rc)[R], T (&rd)[R]) {
  if (sok && i0 + R < n_real) return;
#pragma unroll
  for (int t = 0; t < R; ++t) {
    const long long i = i0 + t;
    if (!sok || i >= n_real) { ra[t] = T(0); rb[t] = T(1); rc[t] = c_pad; rd[t] = T(0); }
    if (i == n_real - 1) rc[t] = c_pad;
  }
}

__device__ __forceinline__ void fence_proxy_async_smem() {
  asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
}

template <typename T, int R, int W, int KIN>
__global__ void __launch_bounds__(W * 32, 2)
tdg_col_reduce_tma_kernel(const __grid_constant__ CUtensorMap tmA, const __grid_constant__ CUtensorMap tmB,
                          const __grid_constant__ CUtensorMap tmC, const __grid_constant__ CUtensorMap tmD,
                          const T* __restrict__ a, const T* __restrict__ b, const T* __restrict__ c,
                          const T* __restrict__ d, T* __restrict__ a2, T* __restrict__ b2,
                          T* __restrict__ c2, T* __restrict__ d2, long long n, long long n_real,
                          long long es, long long S, long long es2, long long ss2, T c_pad, int pf,
                          long long* stamps, int pieces) {
  pdl_entry();
  constexpr int HE = col_heads_elems<T, R>();
  constexpr int Q = R >> KIN;
  constexpr long long CH = (long long)W * R;
  constexpr uint32_t ARR = col_stage_bytes<T, R, W>() / 4;
  extern __shared__ __align__(1024) unsigned char smem_raw[];
  unsigned char* stage = smem_raw;
  uint64_t* bar = reinterpret_cast<uint64_t*>(smem_raw + 4 * ARR);
  T* pages = reinterpret_cast<T*>(smem_raw + 4 * ARR + 16);  // [W][HE]
  T* carry = pages + W * HE;                                  // [2][HE]
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  const long long C = n / CH;
  const long long U = ((S + 31) >> 5) * C;
  // pieces > 0 (gridDim = groups x pieces): CTA c walks chunk range
  // [p C / pieces, (p + 1) C / pieces) of group c % groups, p = c / groups, so
  // the CTAs active together read the same rows of consecutive groups (long
  // contiguous row spans); else a contiguous split of the group-major units
  long long lo, hi;
  if (pieces > 0) {
    const long long GT = (S + 31) >> 5;
    const long long gq = blockIdx.x % GT, p = blockIdx.x / GT;
    lo = gq * C + p * C / pieces;
    hi = gq * C + (p + 1) * C / pieces;
  } else {
    lo = (long long)blockIdx.x * U / gridDim.x;
    hi = ((long long)blockIdx.x + 1) * U / gridDim.x;
  }
  const CUtensorMap* maps[4] = {&tmA, &tmB, &tmC, &tmD};
  auto issue = [&](long long uu) {
    const long long gg = uu / C, cc = uu - gg * C;
    mbar_arrive_expect_tx(bar, 4 * ARR);
#pragma unroll
    for (int q = 0; q < 4; ++q) tma_load_2d(stage + q * ARR, maps[q], (int)(gg * 32), (int)(cc * CH), bar);
    if (pf && uu - 1 >= lo) {  // the unit after: toward L2
      const long long g2 = (uu - 1) / C, c2 = (uu - 1) - g2 * C;
#pragma unroll
      for (int q = 0; q < 4; ++q) tma_prefetch_2d(maps[q], (int)(g2 * 32), (int)(c2 * CH));
    }
  };
  if (threadIdx.x == 0) {
    mbar_init(bar, 1);
    if (hi > lo) issue(hi - 1);
  }
  __syncthreads();
  uint32_t parity = 0;
  int j = 0;
  for (long long u = hi - 1; u >= lo; --u, ++j) {
    // phase stamps (NEXT f4), warp 0, first kStampSystems units: [0] unit
    // start, [1] stage arrived, [2] in-lane forward, [3] heads barrier + tail
    // chain, [4] survivors stored
    Stamp stp;
    if (stamps != nullptr && threadIdx.x < 32 && j < kStampSystems)
      stp.p = stamps + ((long long)blockIdx.x * kStampSystems + j) * kStampSlots;
    stp.mark(0);
    const long long g = u / C, ch = u - g * C;
    const long long s = g * 32 + lane;
    const bool sok = s < S;
    T* pg = pages;
    T* cin = carry + ((j + 1) & 1) * HE;
    if (j == 0 && ch + 1 < C && w == 0) {
      T ha[R], hb[R], hc[R], hd[R];
      col_load4<T, R>(a, b, c, d, es, s, sok, (ch + 1) * CH, n_real, c_pad, ha, hb, hc, hd);
      inlane_forward_interior<T, R, true>(ha, hb, hc, hd, KIN);
      col_put_heads<T, R, KIN>(cin, lane, ha, hb, hc, hd);
    }
    const long long i0 = ch * CH + (long long)w * R;
    T ra[R], rb[R], rc[R], rd[R];
    mbar_wait(bar, parity);
    parity ^= 1;
    stp.mark(1);
    col_read_stage<T, R, W>(stage, w, lane, ra, rb, rc, rd);
    __syncthreads();  // the stage is free: the next unit streams in during the CR levels
    if (threadIdx.x == 0 && u - 1 >= lo) {
      fence_proxy_async_smem();
      issue(u - 1);
    }
    col_fix_ragged<T, R>(sok, i0, n_real, c_pad, ra, rb, rc, rd);
    if (i0 == 0) ra[0] = T(0);
    if (i0 + R == n) rc[R - 1] = T(0);
    inlane_forward_interior<T, R, true>(ra, rb, rc, rd, KIN);
    stp.mark(2);
    col_put_heads<T, R, KIN>(pg + w * HE, lane, ra, rb, rc, rd);
    __syncthreads();
    Heads<T, R> H;
    if (w + 1 < W) {
      col_get_heads<T, R, KIN>(pg + (w + 1) * HE, lane, H);
    } else if (ch + 1 < C) {
      col_get_heads<T, R, KIN>(cin, lane, H);
    } else {
#pragma unroll
      for (int l = 0; l < KIN; ++l) { H.a[l] = T(0); H.rb[l] = T(0); H.c[l] = T(0); H.d[l] = T(0); }
    }
    if (w == 0) col_put_heads<T, R, KIN>(carry + (j & 1) * HE, lane, ra, rb, rc, rd);
    inlane_tail_chain<T, R>(ra, rb, rc, rd, KIN, H);
    stp.mark(3);
    if constexpr (Q == 1 && (W * sizeof(T)) % 32 == 0) {
      if (es2 == 1) {
        // the last pass writes its survivors transposed (system s's reduced
        // row, columns ch W .. ch W + W - 1 from this unit's W warps): through
        // a [4][W][32] tile so that each lane stores its system's W columns as
        // whole 32-byte sectors (one warp per array) instead of every warp
        // storing one 4-byte piece of 32 different sectors
        T* sv = carry + 2 * HE;
        sv[(0 * W + w) * 32 + lane] = ra[R - 1]; sv[(1 * W + w) * 32 + lane] = rb[R - 1];
        sv[(2 * W + w) * 32 + lane] = rc[R - 1]; sv[(3 * W + w) * 32 + lane] = rd[R - 1];
        __syncthreads();
        if (w < 4 && sok) {
          T* outp = (w == 0 ? a2 : w == 1 ? b2 : w == 2 ? c2 : d2) + ((ch * CH) >> KIN) + s * ss2;
          T v[W];
#pragma unroll
          for (int q = 0; q < W; ++q) v[q] = sv[(w * W + q) * 32 + lane];
#pragma unroll
          for (int q = 0; q < W * (int)sizeof(T) / 32; ++q) st32B(outp + q * (32 / (int)sizeof(T)), v + q * (32 / (int)sizeof(T)));
        }
        stp.mark(4);
        continue;  // (the next unit's first barrier orders the tile's reuse)
      }
    }
    if (sok) {
      const long long o = (i0 >> KIN) * es2 + s * ss2;
#pragma unroll
      for (int q = 0; q < Q; ++q) {
        const int t = ((q + 1) << KIN) - 1;
        a2[o + q * es2] = ra[t]; b2[o + q * es2] = rb[t];
        c2[o + q * es2] = rc[t]; d2[o + q * es2] = rd[t];
      }
    }
    stp.mark(4);
  }
}

template <typename T, int R, int W, int KIN>
__global__ void __launch_bounds__(W * 32, TDG_COL_EXPAND_MINB(T))
tdg_col_expand_tma_kernel(const __grid_constant__ CUtensorMap tmA, const __grid_constant__ CUtensorMap tmB,
                          const __grid_constant__ CUtensorMap tmC, const __grid_constant__ CUtensorMap tmD,
                          T* x, const T* __restrict__ x2, long long n, long long n_real,
                          long long es, long long S, long long es2, long long ss2, T c_pad, int pf,
                          long long* stamps) {
  pdl_entry();
  constexpr int Q = R >> KIN;
  constexpr long long CH = (long long)W * R;
  constexpr uint32_t ARR = col_stage_bytes<T, R, W>() / 4;
  extern __shared__ __align__(1024) unsigned char smem_raw[];
  unsigned char* stage = smem_raw;
  uint64_t* bar = reinterpret_cast<uint64_t*>(smem_raw + 4 * ARR);
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  const long long C = n / CH;
  const long long U = ((S + 31) >> 5) * C;
  const CUtensorMap* maps[4] = {&tmA, &tmB, &tmC, &tmD};
  // unit order: pf & 4 = chunk-major (the CTAs active at one time read the
  // same rows of consecutive 32-system groups: long contiguous row spans),
  // else group-major
  const long long GT = (S + 31) >> 5;
  const bool cmaj = (pf & 4) != 0;
  auto unit = [&](long long uu, long long& gg, long long& cc) {
    if (cmaj) { cc = uu / GT; gg = uu - cc * GT; } else { gg = uu / C; cc = uu - gg * C; }
  };
  auto issue = [&](long long uu) {
    long long gg, cc;
    unit(uu, gg, cc);
    mbar_arrive_expect_tx(bar, 4 * ARR);
#pragma unroll
    for (int q = 0; q < 4; ++q) tma_load_2d(stage + q * ARR, maps[q], (int)(gg * 32), (int)(cc * CH), bar);
    if ((pf & 1) && uu + gridDim.x < U) {  // the unit after: toward L2
      long long g2, c2;
      unit(uu + gridDim.x, g2, c2);
#pragma unroll
      for (int q = 0; q < 4; ++q) tma_prefetch_2d(maps[q], (int)(g2 * 32), (int)(c2 * CH));
    }
  };
  if (threadIdx.x == 0) {
    mbar_init(bar, 1);
    if (blockIdx.x < U) issue(blockIdx.x);
  }
  __syncthreads();
  uint32_t parity = 0;
  int j = 0;
  for (long long u = blockIdx.x; u < U; u += gridDim.x, ++j) {
    // phase stamps (NEXT f4): [0] unit start, [1] survivors' x loaded + stage
    // arrived, [2] forward levels recomputed, [3] back-substituted, [4] stored
    Stamp stp;
    if (stamps != nullptr && threadIdx.x < 32 && j < kStampSystems)
      stp.p = stamps + ((long long)blockIdx.x * kStampSystems + j) * kStampSlots;
    stp.mark(0);
    long long g, ch;
    unit(u, g, ch);
    const long long s = g * 32 + lane;
    const bool sok = s < S;
    const long long i0 = ch * CH + (long long)w * R;
    T xs[Q];
    T xprev = T(0);
    if (sok) {
      const long long o = (i0 >> KIN) * es2 + s * ss2;
#pragma unroll
      for (int q = 0; q < Q; ++q) xs[q] = x2[o + q * es2];
      if (i0 > 0) xprev = x2[o - es2];
    } else {
#pragma unroll
      for (int q = 0; q < Q; ++q) xs[q] = T(0);
    }
    T ra[R], rb[R], rc[R], rd[R];
    mbar_wait(bar, parity);
    parity ^= 1;
    stp.mark(1);
    col_read_stage<T, R, W>(stage, w, lane, ra, rb, rc, rd);
    __syncthreads();
    if (threadIdx.x == 0 && u + gridDim.x < U) {
      fence_proxy_async_smem();
      issue(u + gridDim.x);
    }
    col_fix_ragged<T, R>(sok, i0, n_real, c_pad, ra, rb, rc, rd);
    if (i0 == 0) ra[0] = T(0);
    if (i0 + R == n) rc[R - 1] = T(0);
    inlane_forward_interior<T, R, true>(ra, rb, rc, rd, KIN);
    stp.mark(2);
#pragma unroll
    for (int q = 0; q < Q; ++q) rd[((q + 1) << KIN) - 1] = xs[q];
    inlane_backward<T, R>(ra, rb, rc, rd, KIN, xprev);
    stp.mark(3);
    if (sok) {
      T* p = x + s + i0 * es;
      if (i0 + R <= n_real) {
#pragma unroll
        for (int t = 0; t < R; ++t) p[t * es] = rd[t];
      } else {
#pragma unroll
        for (int t = 0; t < R; ++t)
          if (i0 + t < n_real) p[t * es] = rd[t];
      }
    }
    stp.mark(4);
  }
}

}  // namespace tdg
