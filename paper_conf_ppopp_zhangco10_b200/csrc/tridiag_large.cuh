// tridiag_large.cuh -- systems larger than one CTA can hold on chip
// (n > tridiag_max_n): "accelerate larger systems with
// several first steps (as in CR) that reduce the system to fit into shared
// memory".
//
// One reduction pass applies KIN <= log2 R CR levels to every
// equation of an n-system and writes the n >> KIN survivors as a new system;
// passes repeat until the system fits the on-chip kernels, which solve it
// (including the inner PCR / RD of the hybrids).  An expansion pass then
// recomputes the same KIN forward levels from the pass's input (bitwise the
// same values: every update is the fixed cr_unit of the on-chip kernels) and
// runs the KIN backward levels from the survivors' solution.
//
// Work unit: a chunk of CH = P R consecutive equations of one system, one CTA
// of W warps, R equations per lane exactly as in the on-chip kernels.  The
// chunk's last lane needs, at every level, the level-(l-1) state of the next
// chunk's head equation 2^(l-1) - 1; those depend only on the next chunk's
// first R equations.  Each CTA of the reduction pass walks a contiguous range
// of units in DESCENDING order, so the heads it needs are the ones its
// previous unit's first lane produced (carried in shared memory); only the
// first unit of a CTA computes them from the next chunk's first R equations
// (round 2: this replaced a separate heads pass per level).  The expansion
// pass needs no heads at all: the tail chain only changes each lane's tail, a
// survivor whose x comes from the reduced solve.  No unit reads another unit's
// output, so the expansion may overwrite d with x in place.
#pragma once

#include "tridiag_kernels.cuh"  // Stamp

namespace tdg {

// Lane-slice loader for the level-0 arrays (system stride ss, only the first
// n_real equations stored: ragged n is padded with the identity rows of
// load_ragged, c_{n_real-1} <- c_pad) and for the workspace levels (vec).
template <typename T, int R, bool NC>
__device__ __forceinline__ void large_load(const T* p, long long ss, long long sys, long long i0,
                                           long long n_real, bool vec, T pad, T last_val,
                                           bool set_last, T (&v)[R]) {
  const T* base = p + sys * ss;
  if (vec) {
    load_block<T, R, NC>(base + i0, v, true);
  } else {
#pragma unroll
    for (int t = 0; t < R; ++t) {
      const long long i = i0 + t;
      v[t] = i < n_real ? base[i] : pad;
      if (set_last && i == n_real - 1) v[t] = last_val;
    }
  }
}

template <typename T, int R, bool NC_D>
__device__ __forceinline__ void large_load4(const T* a, const T* b, const T* c, const T* d,
                                            long long ss, long long sys, long long i0,
                                            long long n_real, bool vec, T c_pad, T (&ra)[R],
                                            T (&rb)[R], T (&rc)[R], T (&rd)[R]) {
  large_load<T, R, true>(a, ss, sys, i0, n_real, vec, T(0), T(0), false, ra);
  large_load<T, R, true>(b, ss, sys, i0, n_real, vec, T(1), T(0), false, rb);
  large_load<T, R, true>(c, ss, sys, i0, n_real, vec, c_pad, c_pad, true, rc);
  large_load<T, R, NC_D>(d, ss, sys, i0, n_real, vec, T(0), T(0), false, rd);
}

// Heads record per chunk boundary: NH levels x (a, 1/b, c, d).
template <int R>
__host__ __device__ constexpr int large_heads_elems() { return 4 * (ilog2c(R) > 0 ? ilog2c(R) : 1); }

// KIN in-lane CR levels of the lane's R equations, completed across lanes,
// warps (shared memory) and chunks (hbuf); on return the arrays hold the
// state the on-chip kernels reach after cta_inlane_forward with kin = KIN.
template <typename T, int R, int W, int KIN>
__device__ __forceinline__ void large_forward(T (&ra)[R], T (&rb)[R], T (&rc)[R], T (&rd)[R],
                                              const T* hrec, T (*sh)[4]) {
  constexpr int NH = large_heads_elems<R>() / 4;
  const int ls = threadIdx.x, lane = ls & 31, warp = ls >> 5;
  inlane_forward_interior<T, R, true>(ra, rb, rc, rd, KIN);
  Heads<T, R> H;
  heads_from_next_lane<T, R>(ra, rb, rc, rd, KIN, 32, false, H);
  if (lane == 0 && warp > 0) {
#pragma unroll
    for (int l = 1; l <= NH; ++l) {
      if (l <= KIN) {
        const int t = (1 << (l - 1)) - 1;
        T* hp = sh[warp * NH + (l - 1)];
        hp[0] = ra[t]; hp[1] = rb[t]; hp[2] = rc[t]; hp[3] = rd[t];
      }
    }
  }
  __syncthreads();
  if (lane == 31) {
#pragma unroll
    for (int l = 1; l <= NH; ++l) {
      if (l <= KIN) {
        if (warp + 1 < W) {
          const T* hp = sh[(warp + 1) * NH + (l - 1)];
          H.a[l - 1] = hp[0]; H.rb[l - 1] = hp[1]; H.c[l - 1] = hp[2]; H.d[l - 1] = hp[3];
        } else if (hrec) {
          const T* hp = hrec + 4 * (l - 1);
          H.a[l - 1] = hp[0]; H.rb[l - 1] = hp[1]; H.c[l - 1] = hp[2]; H.d[l - 1] = hp[3];
        } else {  // end of the system
          H.a[l - 1] = T(0); H.rb[l - 1] = T(0); H.c[l - 1] = T(0); H.d[l - 1] = T(0);
        }
      }
    }
  }
  inlane_tail_chain<T, R>(ra, rb, rc, rd, KIN, H);
}

// Reduction pass: (a, b, c, d) level j -> survivors (a2, b2, c2, d2) level
// j + 1, n2 = n >> KIN equations per system, contiguous.  CTA c walks units
// [c U / grid, (c + 1) U / grid) from the last to the first (see the header:
// the next chunk's heads are carried from the previous unit).
template <typename T, int R, int W, int KIN>
__global__ void __launch_bounds__(W * 32)
tdg_large_reduce_kernel(const T* __restrict__ a, const T* __restrict__ b, const T* __restrict__ c,
                        const T* __restrict__ d, T* __restrict__ a2, T* __restrict__ b2,
                        T* __restrict__ c2, T* __restrict__ d2, long long n, long long n_real,
                        long long ss, long long S, int vec, T c_pad, long long* stamps) {
  pdl_entry();
  constexpr int P = 32 * W;
  constexpr int NH = large_heads_elems<R>() / 4;
  constexpr int Q = R >> KIN;
  constexpr long long CH = (long long)P * R;
  __shared__ T sh[W * NH][4];
  __shared__ T carry[2][4 * NH];   // heads of the chunk walked last (its first lane)
  const long long C = n / CH;
  const long long n2 = n >> KIN;
  const long long U = S * C;
  const long long lo = (long long)blockIdx.x * U / gridDim.x;
  const long long hi = ((long long)blockIdx.x + 1) * U / gridDim.x;
  const int ls = threadIdx.x;
  int j = 0;
  for (long long u = hi - 1; u >= lo; --u, ++j) {
    // phase stamps (NEXT f4), warp 0, first kStampSystems units: [0] unit
    // start, [1] loads + KIN forward levels (lanes, warps, chunk heads),
    // [2] survivors stored
    Stamp stp;
    if (stamps != nullptr && ls < 32 && j < kStampSystems)
      stp.p = stamps + ((long long)blockIdx.x * kStampSystems + j) * kStampSlots;
    stp.mark(0);
    const long long sys = u / C, ch = u - sys * C;
    const long long i0 = ch * CH + (long long)ls * R;
    T* cnext = carry[(j + 1) & 1];   // heads of chunk ch + 1
    if (j == 0 && ch + 1 < C && ls == 0) {
      // first unit of this CTA: the next chunk's heads from its first R equations
      T ha[R], hb[R], hc[R], hd[R];
      large_load4<T, R, true>(a, b, c, d, ss, sys, (ch + 1) * CH, n_real, vec != 0, c_pad, ha, hb, hc, hd);
      inlane_forward_interior<T, R, true>(ha, hb, hc, hd, KIN);
#pragma unroll
      for (int l = 1; l <= NH; ++l) {
        if (l <= KIN) {
          const int t = (1 << (l - 1)) - 1;
          cnext[4 * (l - 1) + 0] = ha[t]; cnext[4 * (l - 1) + 1] = hb[t];
          cnext[4 * (l - 1) + 2] = hc[t]; cnext[4 * (l - 1) + 3] = hd[t];
        }
      }
    }
    T ra[R], rb[R], rc[R], rd[R];
    large_load4<T, R, true>(a, b, c, d, ss, sys, i0, n_real, vec != 0, c_pad, ra, rb, rc, rd);
    if (i0 == 0) ra[0] = T(0);
    if (i0 + R == n) rc[R - 1] = T(0);
    // (the barrier inside large_forward orders cnext's stores before its reads)
    large_forward<T, R, W, KIN>(ra, rb, rc, rd, ch + 1 < C ? cnext : nullptr, sh);
    stp.mark(1);
    if (ls == 0) {
      // this chunk's heads (its first lane's equations 2^(l-1) - 1, unchanged
      // by the tail chain) for the next unit, chunk ch - 1
      T* cme = carry[j & 1];
#pragma unroll
      for (int l = 1; l <= NH; ++l) {
        if (l <= KIN) {
          const int t = (1 << (l - 1)) - 1;
          cme[4 * (l - 1) + 0] = ra[t]; cme[4 * (l - 1) + 1] = rb[t];
          cme[4 * (l - 1) + 2] = rc[t]; cme[4 * (l - 1) + 3] = rd[t];
        }
      }
    }
    const long long o = sys * n2 + (i0 >> KIN);
#pragma unroll
    for (int q = 0; q < Q; ++q) {
      const int t = ((q + 1) << KIN) - 1;
      a2[o + q] = ra[t]; b2[o + q] = rb[t]; c2[o + q] = rc[t]; d2[o + q] = rd[t];
    }
    stp.mark(2);
    __syncthreads();  // sh / carry are reused by the next unit
  }
}

// Expansion pass: recompute the KIN forward levels of level j, take the
// survivors' x from x2 (level j + 1 solved), back-substitute, write x.
template <typename T, int R, int W, int KIN>
__global__ void __launch_bounds__(W * 32)
tdg_large_expand_kernel(const T* __restrict__ a, const T* __restrict__ b, const T* __restrict__ c,
                        const T* d, T* x, const T* __restrict__ x2, long long n,
                        long long n_real, long long ss, long long S, int vec, T c_pad,
                        long long* stamps) {
  pdl_entry();
  constexpr int P = 32 * W;
  constexpr int Q = R >> KIN;
  constexpr long long CH = (long long)P * R;
  const long long C = n / CH;
  const long long n2 = n >> KIN;
  const int ls = threadIdx.x;
  int j = 0;
  for (long long u = blockIdx.x; u < S * C; u += gridDim.x, ++j) {
    // phase stamps (NEXT f4): [0] unit start, [1] loads + KIN forward levels
    // recomputed, [2] back-substituted, [3] stored
    Stamp stp;
    if (stamps != nullptr && ls < 32 && j < kStampSystems)
      stp.p = stamps + ((long long)blockIdx.x * kStampSystems + j) * kStampSlots;
    stp.mark(0);
    const long long sys = u / C, ch = u - sys * C;
    const long long i0 = ch * CH + (long long)ls * R;
    T ra[R], rb[R], rc[R], rd[R];
    // d may alias x: coherent loads for d
    large_load4<T, R, false>(a, b, c, d, ss, sys, i0, n_real, vec != 0, c_pad, ra, rb, rc, rd);
    if (i0 == 0) ra[0] = T(0);
    if (i0 + R == n) rc[R - 1] = T(0);
    const long long o = sys * n2 + (i0 >> KIN);
    T xs[Q];
#pragma unroll
    for (int q = 0; q < Q; ++q) xs[q] = x2[o + q];
    const T xprev = i0 > 0 ? x2[o - 1] : T(0);
    // interior levels only: the tail chain (and the heads it needs) changes
    // only the tails, survivors whose x comes from x2
    inlane_forward_interior<T, R, true>(ra, rb, rc, rd, KIN);
    stp.mark(1);
#pragma unroll
    for (int q = 0; q < Q; ++q) rd[((q + 1) << KIN) - 1] = xs[q];
    inlane_backward<T, R>(ra, rb, rc, rd, KIN, xprev);
    stp.mark(2);
    T* xb = x + sys * ss;
    if (vec) {
      store_block<T, R>(xb + i0, rd, true);
    } else {
#pragma unroll
      for (int t = 0; t < R; ++t)
        if (i0 + t < n_real) xb[i0 + t] = rd[t];
    }
    stp.mark(3);
  }
}

}  // namespace tdg
