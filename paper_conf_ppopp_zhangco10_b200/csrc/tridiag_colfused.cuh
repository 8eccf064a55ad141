// tridiag_colfused.cuh -- single-kernel ADI column sweep for interleaved
// layouts with n > 32 R (element i of system s at ptr[s + i * es]).
//
// The column passes (tridiag_colpass.cuh) read a, b, c, d from HBM twice:
// once in the reduction pass, once more in the expansion pass (about 9.6 n T
// bytes per system against the 5 n T of Table 1).  This kernel
// runs both passes at once, in two roles of one cooperative grid, so that the
// second read is served by L2:
//
//   * forward CTAs (blockIdx.x < nf) take work units -- 32 consecutive
//     systems (lane = system: every warp access is one coalesced 128 B / 256 B
//     row segment) x CH = W R rows -- in index order, run the log2 R in-lane
//     CR levels (inlane_forward_interior / inlane_tail_chain, the
//     on-chip kernels' correctly rounded operations), write each lane's
//     surviving equation to the workspace and count the unit in its group's
//     arrival counter.  Forward CTAs never wait.
//   * reduced solves: once all C = n / CH units of a group have arrived, its
//     32 reduced systems of n / R equations (the next CR levels and the inner
//     PCR / RD; warp_solve, one warp per system) are solved as
//     TPG = 32 / W tasks of W systems: task k by the forward CTA that ran the
//     group's unit k, right after its NEXT unit (by then the group is
//     complete in all but rare cases), so the solves spread over the grid and
//     no CTA stalls on a group it just finished.
//   * expand CTAs take the same units in the same order a few microseconds
//     later: wait for the group's done flag, reload the unit's rows (TMA; the
//     forward CTA loaded them moments ago, so they come from L2), recompute
//     the interior forward levels, take the survivors' x and back-substitute
//     (P:L294-300), write x.
//
// The last warp's tail needs the head equations of the next chunk at every
// level: the forward TMA box carries the next chunk's first R rows as well.
// Synchronisation: release/acquire on per-group counters in the workspace
// (zeroed by the launcher); only expand CTAs wait, and only on forward work,
// which never waits, so with all CTAs co-resident (cooperative launch) the
// kernel cannot deadlock; a bounded poll traps instead of hanging if that
// ever fails.  x may alias d: a unit's rows are written only after every
// unit of its group has finished reading them.
#pragma once

#include "tridiag_colpass.cuh"

namespace tdg {


// Polling uses relaxed loads (an acquire load invalidates the whole L1,
// CCTL.IVALL, on every poll); one acq_rel fence after the awaited value has
// been observed makes the producers' released writes visible (fence-based
// synchronisation of the PTX memory model).
__device__ __forceinline__ unsigned ld_relaxed_gpu(const unsigned* p) {
  unsigned v;
  asm volatile("ld.relaxed.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void fence_acq_rel_gpu() { asm volatile("fence.acq_rel.gpu;" ::: "memory"); }
__device__ __forceinline__ void red_add_release_gpu(unsigned* p, unsigned v) {
  asm volatile("red.release.gpu.global.add.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}

// Thread 0 polls a counter (relaxed) until it reaches target, then fences;
// the CTA barrier orders every thread's following reads after it.
__device__ __forceinline__ void wait_count(const unsigned* f, unsigned target) {
  if (threadIdx.x == 0) {
    unsigned long long spins = 0;
    while (ld_relaxed_gpu(f) < target) {
      __nanosleep(128);
      if (++spins > (1ull << 26)) __trap();  // not co-resident: fail, never hang
    }
    fence_acq_rel_gpu();
  }
  __syncthreads();
}

// Rows per unit and TMA box height (the unit's rows + the next chunk's first R).
template <typename T, int R, int W>
__host__ __device__ constexpr int cf_box_rows() { return W * R + R; }
template <typename T, int R, int W>
__host__ __device__ constexpr uint32_t cf_arr_bytes() { return 32u * cf_box_rows<T, R, W>() * sizeof(T); }

// Shared memory: stage + mbarrier + one region reused by the forward phases
// (heads pages [W+1][HE], then the survivor transpose [4][32][W+1]) + a flag.
template <typename T, int R, int W>
__host__ __device__ constexpr size_t cf_region_bytes() {
  return ((size_t)(W + 1) * col_heads_elems<T, R>() > (size_t)4 * 32 * (W + 1)
              ? (size_t)(W + 1) * col_heads_elems<T, R>()
              : (size_t)4 * 32 * (W + 1)) * sizeof(T);
}
template <typename T, int R, int W>
__host__ __device__ constexpr size_t cf_smem_bytes() {
  return 4 * (size_t)cf_arr_bytes<T, R, W>() + 16 + cf_region_bytes<T, R, W>() + 32;
}

// One reduced-solve task: systems blk * W + w of group g, one per warp.
template <typename T, int W, int R2, int INNER>
__device__ __forceinline__ void cf_solve_task(const T* red, T* xred, long long G, long long n_red,
                                              long long g, int blk, int k2, const unsigned* arrived,
                                              unsigned C, unsigned* done) {
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  wait_count(arrived + g, C);
  const long long j = (long long)blk * W + w;
  if (j < 32) {
    T qa[R2], qb[R2], qc[R2], qd[R2];
    const long long base = (g * 32 + j) * n_red + lane * R2;
    const long long AS = G * 32 * n_red;
#pragma unroll
    for (int t = 0; t < R2; ++t) {
      qa[t] = __ldcg(red + base + t);
      qb[t] = __ldcg(red + AS + base + t);
      qc[t] = __ldcg(red + 2 * AS + base + t);
      qd[t] = __ldcg(red + 3 * AS + base + t);
    }
    warp_solve<T, R2, INNER, -1>(qa, qb, qc, qd, k2, lane, 32);
#pragma unroll
    for (int t = 0; t < R2; ++t) xred[base + t] = qd[t];
  }
  __syncthreads();
  if (threadIdx.x == 0) red_add_release_gpu(done + g, 1u);
}


// Kernel.  maps 0..3: a, b, c, d as {S, n_real} tensors, boxes {32, CH + R}
// (forward); maps 4..7: the same with boxes {32, CH} (expand).  Workspace:
// red[4][G][32][n_red] survivors, xred[G][32][n_red] their x; cnt[2 G]
// (arrivals, done flags).  R2 = n_red / 32 equations per lane of the reduced
// solve.
template <typename T, int R, int W, int R2, int INNER>
__global__ void __launch_bounds__(W * 32, 2)
tdg_col_fused_kernel(const __grid_constant__ CUtensorMap tmA, const __grid_constant__ CUtensorMap tmB,
                     const __grid_constant__ CUtensorMap tmC, const __grid_constant__ CUtensorMap tmD,
                     const __grid_constant__ CUtensorMap teA, const __grid_constant__ CUtensorMap teB,
                     const __grid_constant__ CUtensorMap teC, const __grid_constant__ CUtensorMap teD,
                     T* x, T* ws, unsigned* cnt, long long n, long long n_real, long long es,
                     long long S, int k2, T c_pad, int nf) {
  pdl_entry();
  constexpr int LR = ilog2c(R);
  constexpr int HE = col_heads_elems<T, R>();
  constexpr long long CH = (long long)W * R;
  constexpr int BR = cf_box_rows<T, R, W>();
  constexpr uint32_t ARR = cf_arr_bytes<T, R, W>();
  constexpr uint32_t ARR_E = 32u * W * R * sizeof(T);
  extern __shared__ __align__(1024) unsigned char smem_raw[];
  unsigned char* stage = smem_raw;
  uint64_t* bar = reinterpret_cast<uint64_t*>(smem_raw + 4 * ARR);
  T* region = reinterpret_cast<T*>(smem_raw + 4 * ARR + 16);
  const int tid = threadIdx.x;
  const int lane = tid & 31, w = tid >> 5;
  const long long C = n / CH;         // units per group
  const long long G = (S + 31) >> 5;  // groups
  const long long U = G * C;
  const long long n_red = n / R;      // == 32 * R2 (checked by the launcher)
  T* red = ws;                        // [4][G][32][n_red]
  T* xred = ws + 4 * G * 32 * n_red;  // [G][32][n_red]
  unsigned* arrived = cnt;            // [G]
  unsigned* done = cnt + G;           // [G] tasks finished per group
  constexpr int TPG = (32 + W - 1) / W;  // reduced-solve tasks per group
  long long pend = -1;                    // task of this CTA's previous unit
  const bool fwd = (int)blockIdx.x < nf;
  const long long first = fwd ? blockIdx.x : blockIdx.x - nf;
  const long long stride = fwd ? nf : gridDim.x - nf;

  const CUtensorMap* fmaps[4] = {&tmA, &tmB, &tmC, &tmD};
  const CUtensorMap* emaps[4] = {&teA, &teB, &teC, &teD};
  auto issue = [&](long long uu) {
    const long long gg = uu / C, cc = uu - gg * C;
    if (fwd) {
      mbar_arrive_expect_tx(bar, 4 * ARR);
#pragma unroll
      for (int q = 0; q < 4; ++q) tma_load_2d(stage + q * ARR, fmaps[q], (int)(gg * 32), (int)(cc * CH), bar);
    } else {
      mbar_arrive_expect_tx(bar, 4 * ARR_E);
#pragma unroll
      for (int q = 0; q < 4; ++q) tma_load_2d(stage + q * ARR_E, emaps[q], (int)(gg * 32), (int)(cc * CH), bar);
    }
  };
  if (tid == 0) {
    mbar_init(bar, 1);
    if (first < U) issue(first);
  }
  __syncthreads();
  uint32_t parity = 0;
  for (long long u = first; u < U; u += stride) {
    const long long g = u / C, ch = u - g * C;
    const long long s = g * 32 + lane;
    const bool sok = s < S;
    const long long i0 = ch * CH + (long long)w * R;
    if (fwd) {
      // ================= forward role =================
      T* pages = region;  // [W + 1][HE]
      mbar_wait(bar, parity);
      parity ^= 1;
      if (w == W - 1) {
        // heads of the next chunk (its first R rows, same lane), into page W
        if (ch + 1 < C) {
          T ha[R], hb[R], hc[R], hd[R];
          const T* st = reinterpret_cast<const T*>(stage) + (W * R) * 32 + lane;
#pragma unroll
          for (int t = 0; t < R; ++t) {
            ha[t] = st[t * 32]; hb[t] = st[BR * 32 + t * 32];
            hc[t] = st[2 * BR * 32 + t * 32]; hd[t] = st[3 * BR * 32 + t * 32];
          }
          col_fix_ragged<T, R>(sok, (ch + 1) * CH, n_real, c_pad, ha, hb, hc, hd);
          if ((ch + 1) * CH + R == n) hc[R - 1] = T(0);
          inlane_forward_interior<T, R>(ha, hb, hc, hd, LR);
          col_put_heads<T, R, LR>(pages + W * HE, lane, ha, hb, hc, hd);
        } else {  // end of the system
#pragma unroll
          for (int e = 0; e < HE / 32; ++e) pages[W * HE + e * 32 + lane] = T(0);
        }
      }
      T ra[R], rb[R], rc[R], rd[R];
      {
        const T* st = reinterpret_cast<const T*>(stage) + (w * R) * 32 + lane;
#pragma unroll
        for (int t = 0; t < R; ++t) {
          ra[t] = st[t * 32]; rb[t] = st[BR * 32 + t * 32];
          rc[t] = st[2 * BR * 32 + t * 32]; rd[t] = st[3 * BR * 32 + t * 32];
        }
      }
      __syncthreads();  // the stage is free: the next unit streams in from here on
      if (tid == 0 && u + stride < U) {
        fence_proxy_async_smem();
        issue(u + stride);
      }
      col_fix_ragged<T, R>(sok, i0, n_real, c_pad, ra, rb, rc, rd);
      if (i0 == 0) ra[0] = T(0);
      if (i0 + R == n) rc[R - 1] = T(0);
      inlane_forward_interior<T, R>(ra, rb, rc, rd, LR);
      col_put_heads<T, R, LR>(pages + w * HE, lane, ra, rb, rc, rd);
      __syncthreads();
      {
        Heads<T, R> H;
        col_get_heads<T, R, LR>(pages + (w + 1) * HE, lane, H);
        inlane_tail_chain<T, R>(ra, rb, rc, rd, LR, H);
      }
      __syncthreads();  // pages -> survivor transpose
      T* sv = region;   // [4][32][W + 1]
      sv[(0 * 32 + lane) * (W + 1) + w] = ra[R - 1];
      sv[(1 * 32 + lane) * (W + 1) + w] = rb[R - 1];
      sv[(2 * 32 + lane) * (W + 1) + w] = rc[R - 1];
      sv[(3 * 32 + lane) * (W + 1) + w] = rd[R - 1];
      __syncthreads();
#pragma unroll
      for (int e = tid; e < 4 * 32 * W; e += 32 * W) {
        const int q = e / (32 * W), j = (e / W) & 31, r = e % W;
        red[((q * G + g) * 32 + j) * n_red + ch * W + r] = sv[(q * 32 + j) * (W + 1) + r];
      }
      __syncthreads();
      // release (cumulative over the CTA's stores ordered by the barrier)
      if (tid == 0) red_add_release_gpu(arrived + g, 1u);
      if (pend >= 0)
        cf_solve_task<T, W, R2, INNER>(red, xred, G, n_red, pend / TPG, (int)(pend % TPG), k2, arrived,
                                       (unsigned)C, done);
      pend = ch < TPG ? g * TPG + ch : -1;
    } else {
      // ================= expand role =================
      wait_count(done + g, (unsigned)TPG);
      const long long r = ch * W + w;
      const long long xb = (g * 32 + lane) * n_red;
      const T xs = __ldcg(xred + xb + r);
      const T xprev = r > 0 ? __ldcg(xred + xb + r - 1) : T(0);
      mbar_wait(bar, parity);
      parity ^= 1;
      T ra[R], rb[R], rc[R], rd[R];
      {
        const T* st = reinterpret_cast<const T*>(stage) + (w * R) * 32 + lane;
#pragma unroll
        for (int t = 0; t < R; ++t) {
          ra[t] = st[t * 32]; rb[t] = st[W * R * 32 + t * 32];
          rc[t] = st[2 * W * R * 32 + t * 32]; rd[t] = st[3 * W * R * 32 + t * 32];
        }
      }
      __syncthreads();
      if (tid == 0 && u + stride < U) {
        fence_proxy_async_smem();
        issue(u + stride);
      }
      col_fix_ragged<T, R>(sok, i0, n_real, c_pad, ra, rb, rc, rd);
      if (i0 == 0) ra[0] = T(0);
      if (i0 + R == n) rc[R - 1] = T(0);
      inlane_forward_interior<T, R>(ra, rb, rc, rd, LR);
      rd[R - 1] = xs;
      inlane_backward<T, R>(ra, rb, rc, rd, LR, xprev);
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
  if (fwd && pend >= 0)
    cf_solve_task<T, W, R2, INNER>(red, xred, G, n_red, pend / TPG, (int)(pend % TPG), k2, arrived,
                                   (unsigned)C, done);
}

}  // namespace tdg
