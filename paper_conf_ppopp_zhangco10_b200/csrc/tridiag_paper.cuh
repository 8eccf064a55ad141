// tridiag_paper.cuh -- the paper's own GT200 kernel schedule for CR, kept as
// the measured baseline of its Fig 9 (E5 of SURVEY.md 7.1; P:L663-696,
// P:L815-829).  NOT a product path: the library's CR runs the
// register-blocked kernels of tridiag_kernels.cuh.
//
// What the paper does:
//  * systems mapped to blocks, equations to threads: one CTA per system,
//    n/2 threads, the grid = the number of systems;
//  * the four inputs loaded from global memory into shared memory, solved
//    IN PLACE there (five arrays: a, b, c, d, x), x stored back;
//  * forward reduction with half as many active threads each step, backward
//    substitution doubling them, contiguous thread indices as the active
//    threads, a __syncthreads() between steps;
//  * in place, the access stride doubles every step, so on 32 banks the
//    accesses of a warp become 2-, 4-, ... 32-way bank conflicts (the paper's
//    16 banks: up to 16-way, Fig 9).
// MODE 0 is that schedule.  MODE 1 is the paper's timing-only control
// ("the same program modified to enforce a shared memory access
// stride of one so that it is bank-conflict-free. This results in an
// incorrect algorithm, but is for timing comparison only"): every active
// thread t addresses equation t and its neighbours t-1 / t+1 instead of the
// strided ones, with the same arithmetic, the same active-thread counts and
// the same barriers.  Its x is meaningless.
//
// Arithmetic: the paper's formulas with IEEE division (Fig 1;
// 2x2 solve by Cramer's rule, reading R5), so MODE 0 meets the G1/G2 gates.
// Stamps (optional): thread 0 of each of the first kPaperStampBlocks CTAs
// records clock64() after the load, after every forward step, after the 2x2
// solve, after every backward step and after the store -- the per-step
// times of Fig 8 / Fig 9.
#pragma once

#include "tridiag_device.cuh"

namespace tdg {

constexpr int kPaperStampBlocks = 512;
constexpr int kPaperStampSlots = 32;

template <typename T, int MODE>
__global__ void __launch_bounds__(512) tdg_paper_cr_kernel(const T* __restrict__ ga,
                                                           const T* __restrict__ gb,
                                                           const T* __restrict__ gc,
                                                           const T* __restrict__ gd, T* gx, int n,
                                                           long long* stamps) {
  pdl_entry();
  extern __shared__ __align__(16) unsigned char paper_smem[];
  T* a = reinterpret_cast<T*>(paper_smem);
  T* b = a + n;
  T* c = b + n;
  T* d = c + n;
  T* x = d + n;
  const int t = threadIdx.x;  // n / 2 threads
  const long long sys = blockIdx.x;
  long long* st = (stamps != nullptr && blockIdx.x < kPaperStampBlocks && t == 0)
                      ? stamps + (long long)blockIdx.x * kPaperStampSlots
                      : nullptr;
  int slot = 0;
  auto mark = [&] {
    if (st != nullptr && slot < kPaperStampSlots) st[slot++] = clock64();
  };
  mark();
  // load: thread t moves equations t and t + n/2 (coalesced)
  const size_t base = (size_t)sys * (size_t)n;
  const int h = n >> 1;
#pragma unroll
  for (int q = 0; q < 2; ++q) {
    const int i = t + q * h;
    a[i] = ga[base + i];
    b[i] = gb[base + i];
    c[i] = gc[base + i];
    d[i] = gd[base + i];
  }
  __syncthreads();
  if (t == 0) a[0] = T(0);          // a_0, c_{n-1} are not matrix entries (R1)
  if (t == h - 1) c[n - 1] = T(0);
  __syncthreads();
  mark();
  // forward reduction: log2 n - 1 steps, stride doubling (Fig 1)
  int delta = 1;
  const int steps = 31 - __clz(n) - 1;
  for (int s = 0; s < steps; ++s) {
    const int active = n >> (s + 1);  // equations updated this step
    if (t < active) {
      int i, lo, hi;
      if (MODE == 0) {
        i = (delta << 1) * (t + 1) - 1;  // i = 2^(s+1) (t+1) - 1 (R4)
        lo = i - delta;
        hi = i + delta;
      } else {
        i = t;
        lo = t;
        hi = t + 1;
      }
      const T k1 = a[i] / b[lo];
      T k2 = T(0), ahi = T(0), chi = T(0), dhi = T(0);
      if (hi < n) {  // absent upper neighbour contributes 0 (R3)
        k2 = c[i] / b[hi];
        ahi = a[hi]; chi = c[hi]; dhi = d[hi];
      }
      const T na = -a[lo] * k1;
      const T nc = -chi * k2;
      const T nb = b[i] - c[lo] * k1 - ahi * k2;
      const T nd = d[i] - d[lo] * k1 - dhi * k2;
      a[i] = na; b[i] = nb; c[i] = nc; d[i] = nd;
    }
    delta <<= 1;
    __syncthreads();
    mark();
  }
  // 2x2 solve of the last two unknowns p = n/2 - 1, q = n - 1 (a3, Cramer)
  if (t == 0) {
    const int p = MODE == 0 ? (n >> 1) - 1 : 0;
    const int q = MODE == 0 ? n - 1 : 1;
    const T det = b[p] * b[q] - c[p] * a[q];
    x[p] = (d[p] * b[q] - c[p] * d[q]) / det;
    x[q] = (b[p] * d[q] - d[p] * a[q]) / det;
  }
  __syncthreads();
  mark();
  // backward substitution: log2 n - 1 steps, stride halving (Fig 1)
  int active = 1;
  for (int s = 0; s < steps; ++s) {
    delta >>= 1;
    active <<= 1;
    if (t < active) {
      int i, lo, hi;
      if (MODE == 0) {
        i = (delta << 1) * t + delta - 1;  // unknowns i = delta - 1 (mod 2 delta)
        lo = i - delta;
        hi = i + delta;
      } else {
        i = t;
        lo = t;
        hi = t + 1;
      }
      const T xlo = lo >= 0 ? x[lo] : T(0);
      x[i] = (d[i] - a[i] * xlo - c[i] * x[hi]) / b[i];
    }
    __syncthreads();
    mark();
  }
#pragma unroll
  for (int q = 0; q < 2; ++q) {
    const int i = t + q * h;
    gx[base + i] = x[i];
  }
  mark();
}

}  // namespace tdg
