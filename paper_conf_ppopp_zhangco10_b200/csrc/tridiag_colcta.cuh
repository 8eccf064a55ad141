// tridiag_colcta.cuh -- single-pass ADI column sweep for interleaved layouts
// (element i of system s at s + i es): a group of G consecutive systems is
// solved entirely on chip by a cluster of C CTAs (C = 1 or 2), so every input
// element crosses HBM once and x once: the 5 n T roofline of the row kernels,
// where the column CR passes (tridiag_colpass.cuh) read the input twice.
//
// Layout of the work (ADI: P:L105-107; CR: P:L280-304):
//   * lane = (q, g): g = lane % G is the system of the group, q = lane / G
//     (Q = 32 / G row-blocks per warp); thread (warp w, q, g) of cluster rank
//     c owns the R consecutive rows of row-block rb = (c W + w) Q + q of
//     system g.  A warp's load of one row touches Q segments of G T = 16
//     bytes (fp32 G = 4, fp64 G = 2); the neighbouring group's CTAs read the
//     other half of each 32-byte sector at the same time.
//   * the CTA's rows of the group arrive as 16-byte cp.async copies (one row
//     segment of the G systems each) in a shared stage whose row-blocks are
//     padded by 16 bytes (bank-conflict-free lane-blocked reads); the next
//     group's copies are issued as soon as every thread holds the current one
//     in registers, so HBM streams while the group computes, and its L2
//     prefetch (TMA boxes) runs a group ahead.
//   * CR levels: log2 R in-lane levels (inlane_forward_interior /
//     inlane_tail_chain, the next row-block's heads by a shuffle of G lanes,
//     from the next warp or the next cluster rank at the warp / CTA edge),
//     then kr <= log2 Q levels across the row-blocks of a warp (shuffles of
//     sg G lanes, the warp's last row-block from the next warp's lane heads),
//     leaving W C (Q >> kr) = m <= 32 survivors per system, which every rank
//     gathers (its own and its peer's through distributed shared memory) and
//     solves redundantly, one warp per system (lane_level_solve: the inner
//     PCR / RD of the hybrids), then the backward levels.  Every update is the
//     same correctly rounded cr_unit / back_unit on the same neighbours as in
//     the contiguous kernels, so x is bitwise the contiguous solve's.
//   * synchronisation per group: three cluster barriers (C = 2) or CTA
//     barriers (C = 1): heads, lane heads, survivors; one CTA barrier after
//     the redundant survivor solve.
#pragma once

#include <cooperative_groups.h>

#include "tridiag_tma.cuh"  // Stamp, tma_prefetch_2d, smem helpers

namespace tdg {

template <typename T>
__host__ __device__ constexpr int colcta_G() { return 16 / (int)sizeof(T); }

// shared memory (elements of T): in-lane heads [W][G][LR][4], lane heads
// [W][G][5][4], survivors [G][4][32], survivor x [G][32]
template <typename T, int R, int W>
__host__ __device__ constexpr int colcta_smem_elems() {
  return W * colcta_G<T>() * (ilog2c(R) > 0 ? ilog2c(R) : 1) * 4 + W * colcta_G<T>() * 5 * 4 +
         colcta_G<T>() * 4 * 32 + colcta_G<T>() * 32;
}
// Stage of one CTA's rows of a group: 4 arrays x (W Q row-blocks of R rows x
// 16 bytes, each row-block padded by 16 bytes), then the exchange regions.
// The padding makes the lane-blocked reads bank-conflict free: row-block q
// of a warp starts (R + 1) 16 bytes after row-block q - 1, i.e. 4 banks on.
template <typename T, int R>
__host__ __device__ constexpr int colcta_blk_bytes() { return (R + 1) * 16; }
template <typename T, int R, int W>
__host__ __device__ constexpr size_t colcta_arr_bytes() {
  return (size_t)W * (32 / colcta_G<T>()) * colcta_blk_bytes<T, R>();
}
template <typename T, int R, int W>
__host__ __device__ constexpr size_t colcta_smem_bytes() {
  return 4 * colcta_arr_bytes<T, R, W>() + (size_t)colcta_smem_elems<T, R, W>() * sizeof(T);
}

template <int C>
__device__ __forceinline__ void colcta_sync() {
  if constexpr (C > 1) {
    asm volatile("barrier.cluster.arrive.release.aligned;\n\tbarrier.cluster.wait.acquire.aligned;" ::: "memory");
  } else {
    __syncthreads();
  }
}

// Generic pointer to element `off` of the cluster peer's dynamic shared memory
// (the same layout); the CTA's own when C == 1.
template <typename T, int C>
__device__ __forceinline__ T* colcta_peer(T* base, int peer) {
  if constexpr (C > 1) {
    namespace cg = cooperative_groups;
    return cg::this_cluster().map_shared_rank(base, peer);
  } else {
    (void)peer;
    return base;
  }
}

template <typename T, int R, int W, int C, int INNER>
__global__ void __launch_bounds__(W * 32, W <= 8 ? 2 : 1)
tdg_colcta_kernel(const __grid_constant__ CUtensorMap tmA, const __grid_constant__ CUtensorMap tmB,
                  const __grid_constant__ CUtensorMap tmC, const __grid_constant__ CUtensorMap tmD,
                  const T* __restrict__ a, const T* __restrict__ b, const T* __restrict__ c,
                  const T* d, T* x, long long n, long long S, long long es, int k, int pf,
                  long long* stamps) {
  constexpr int G = colcta_G<T>();
  constexpr int Q = 32 / G;
  constexpr int LR = ilog2c(R);
  constexpr int LRH = LR > 0 ? LR : 1;
  constexpr int ROWS = W * Q * R;            // rows per CTA
  constexpr int PFB = ROWS < 256 ? ROWS : 256;  // rows per prefetch box
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const int q = lane / G, g = lane % G;
  int rank = 0;
  if constexpr (C > 1) {
    namespace cg = cooperative_groups;
    rank = (int)cg::this_cluster().block_rank();
  }
  const long long cluster = blockIdx.x / C, nclusters = gridDim.x / C;
  const long long groups = (S + G - 1) / G;
  const CUtensorMap* maps[4] = {&tmA, &tmB, &tmC, &tmD};
  constexpr int NB = ROWS / PFB;                  // L2 prefetch boxes per array
  constexpr int BLK = colcta_blk_bytes<T, R>();
  constexpr uint32_t ARR = (uint32_t)colcta_arr_bytes<T, R, W>();
  auto prefetch_group = [&](long long grp) {       // L2 only, lanes of warp 0
    for (int i = lane; i < 4 * NB; i += 32)
      tma_prefetch_2d(maps[i / NB], (int)(grp * G), (int)((long long)rank * ROWS + (i % NB) * PFB));
  };
  if ((pf & 2) && warp == 0 && cluster < groups) prefetch_group(cluster);
  pdl_entry();

  extern __shared__ __align__(16) unsigned char colcta_smem[];
  unsigned char* stage = colcta_smem;
  const T* arrs[4] = {a, b, c, d};
  // the group's ROWS rows x 4 arrays as 16-byte cp.async copies (one row
  // segment of the G systems each; every thread issues 4 ROWS / (32 W))
  auto issue = [&](long long grp) {
    const long long s0 = grp * G;
    const bool full = s0 + G <= S;
#pragma unroll 4
    for (int o = threadIdx.x; o < 4 * ROWS; o += W * 32) {
      const int arr = o / ROWS, row = o % ROWS;
      unsigned char* dst = stage + arr * ARR + (row / R) * BLK + (row % R) * 16;
      const T* src = arrs[arr] + s0 + ((long long)rank * ROWS + row) * es;
      if (full) {
        asm volatile("cp.async.cg.shared.global [%0], [%1], 16;" ::"r"(smem_u32(dst)), "l"(src) : "memory");
      } else {  // ragged last group: only the systems that exist
        const int valid = (int)(S - s0) * (int)sizeof(T);
        asm volatile("cp.async.ca.shared.global [%0], [%1], 16, %2;" ::"r"(smem_u32(dst)), "l"(src),
                     "r"(valid) : "memory");
      }
    }
    asm volatile("cp.async.commit_group;" ::: "memory");
  };
  if (cluster < groups) issue(cluster);
  T* heads = reinterpret_cast<T*>(colcta_smem + 4 * ARR);  // [W][G][LRH][4]
  T* heads2 = heads + W * G * LRH * 4;                    // [W][G][5][4]
  T* surv = heads2 + W * G * 5 * 4;                       // [G][4][32]
  T* xs = surv + G * 4 * 32;                              // [G][32]
  const int peer = rank ^ 1;
  const int kr = k - LR;                  // CR levels across row-blocks (<= log2 Q)
  const int per_warp = Q >> kr;           // survivors per warp per system
  const int msurv = W * C * per_warp;     // = m <= 32
  const T c_pad = INNER == kRD ? T(1) : T(0);
  (void)c_pad;
  int it = 0;
  for (long long grp = cluster; grp < groups; grp += nclusters, ++it) {
    Stamp stp;
    if (stamps != nullptr && warp == 0 && it < kStampSystems)
      stp.p = stamps + ((long long)blockIdx.x * kStampSystems + it) * kStampSlots;
    stp.mark(0);
    if ((pf & 1) && warp == 0 && grp + 2 * nclusters < groups) prefetch_group(grp + 2 * nclusters);
    const long long s = grp * G + g;
    const bool sok = s < S;
    const int rb = (rank * W + warp) * Q + q;       // row-block within the system
    const long long i0 = (long long)rb * R;
    T ra[R], rbv[R], rc[R], rd[R];
    asm volatile("cp.async.wait_all;" ::: "memory");
    __syncthreads();
    {
      // element (row t of row-block rb, system g) at rb BLK + t 16 + g T
      const uint32_t base = (uint32_t)(warp * Q + q) * BLK + (uint32_t)g * (uint32_t)sizeof(T);
#pragma unroll
      for (int t = 0; t < R; ++t) {
        const uint32_t off = base + (uint32_t)t * 16u;
        ra[t] = sok ? *reinterpret_cast<const T*>(stage + 0 * ARR + off) : T(0);
        rbv[t] = sok ? *reinterpret_cast<const T*>(stage + 1 * ARR + off) : T(1);
        rc[t] = sok ? *reinterpret_cast<const T*>(stage + 2 * ARR + off) : T(0);
        rd[t] = sok ? *reinterpret_cast<const T*>(stage + 3 * ARR + off) : T(0);
      }
    }
    if (rb == 0) ra[0] = T(0);                    // a_0, c_{n-1}: not matrix entries (R1)
    if (i0 + R == n) rc[R - 1] = T(0);
    stp.mark(1);
    // ---- in-lane CR levels 1..LR; heads of the next row-block ----
    inlane_forward_interior<T, R, true>(ra, rbv, rc, rd, LR);
    Heads<T, R> H;
#pragma unroll
    for (int l = 1; l <= LR; ++l) {
      const int t = (1 << (l - 1)) - 1;
      H.a[l - 1] = __shfl_down_sync(kFull, ra[t], G);
      H.rb[l - 1] = __shfl_down_sync(kFull, rbv[t], G);
      H.c[l - 1] = __shfl_down_sync(kFull, rc[t], G);
      H.d[l - 1] = __shfl_down_sync(kFull, rd[t], G);
    }
    // row-block q = 0 of warp w publishes its heads for warp w - 1 (or, for
    // warp 0 of rank 1, for the last warp of rank 0)
    if (q == 0) {
      T* dst = nullptr;
      if (warp > 0) dst = heads + ((warp - 1) * G + g) * LRH * 4;
      else if (rank > 0) dst = colcta_peer<T, C>(heads, peer) + ((W - 1) * G + g) * LRH * 4;
      if (dst) {
#pragma unroll
        for (int l = 1; l <= LR; ++l) {
          const int t = (1 << (l - 1)) - 1;
          dst[(l - 1) * 4 + 0] = ra[t]; dst[(l - 1) * 4 + 1] = rbv[t];
          dst[(l - 1) * 4 + 2] = rc[t]; dst[(l - 1) * 4 + 3] = rd[t];
        }
      }
    }
    colcta_sync<C>();
    // every thread of this CTA has read the stage: the next group streams in
    if (grp + nclusters < groups) issue(grp + nclusters);
    if (q == Q - 1) {
      const bool last = warp == W - 1 && rank == C - 1;   // end of the system
      const T* hp = heads + (warp * G + g) * LRH * 4;
#pragma unroll
      for (int l = 1; l <= LR; ++l) {
        H.a[l - 1] = last ? T(0) : hp[(l - 1) * 4 + 0];
        H.rb[l - 1] = last ? T(0) : hp[(l - 1) * 4 + 1];
        H.c[l - 1] = last ? T(0) : hp[(l - 1) * 4 + 2];
        H.d[l - 1] = last ? T(0) : hp[(l - 1) * 4 + 3];
      }
    }
    inlane_tail_chain<T, R>(ra, rbv, rc, rd, LR, H);
    stp.mark(2);
    // ---- kr CR levels across the row-blocks of the warp (stride sg row-blocks) ----
    T A = ra[R - 1], B = rbv[R - 1], Cc = rc[R - 1], D = rd[R - 1];
#pragma unroll
    for (int l = 1; l <= 5; ++l) {
      if (l <= kr) {
        const int sg = 1 << (l - 1);
        const int md = q & (2 * sg - 1);
        const T rcB = rcp1(B);
        if (md == sg - 1) B = rcB;
        const T la = __shfl_up_sync(kFull, A, sg * G), lb = __shfl_up_sync(kFull, B, sg * G);
        const T lc = __shfl_up_sync(kFull, Cc, sg * G), ld = __shfl_up_sync(kFull, D, sg * G);
        const T ha = __shfl_down_sync(kFull, A, sg * G), hb = __shfl_down_sync(kFull, B, sg * G);
        const T hc = __shfl_down_sync(kFull, Cc, sg * G), hd = __shfl_down_sync(kFull, D, sg * G);
        if (md == 2 * sg - 1 && q != Q - 1) cr_unit(A, B, Cc, D, la, lb, lc, ld, ha, hb, hc, hd);
      }
    }
    // lane heads of this warp (row-blocks q = 2^l - 1, final state) for the
    // previous warp's last row-block (or rank 0's last warp)
    if (kr > 0 && ((q + 1) & q) == 0 && q < (1 << (kr - 1))) {
      T* dst = nullptr;
      if (warp > 0) dst = heads2 + ((warp - 1) * G + g) * 5 * 4;
      else if (rank > 0) dst = colcta_peer<T, C>(heads2, peer) + ((W - 1) * G + g) * 5 * 4;
      if (dst) {
        const int l = ilog2c(q + 1);
        dst[l * 4 + 0] = A; dst[l * 4 + 1] = B; dst[l * 4 + 2] = Cc; dst[l * 4 + 3] = D;
      }
    }
    colcta_sync<C>();
    // the warp's last row-block (q = Q - 1) through the kr levels
#pragma unroll
    for (int l = 1; l <= 5; ++l) {
      if (l <= kr) {
        const int sg = 1 << (l - 1);
        const int src = (Q - 1 - sg) * G + g;
        const T la = __shfl_sync(kFull, A, src), lb = __shfl_sync(kFull, B, src);
        const T lc = __shfl_sync(kFull, Cc, src), ld = __shfl_sync(kFull, D, src);
        if (q == Q - 1) {
          T ha = T(0), hb = T(0), hc = T(0), hd = T(0);
          if (!(warp == W - 1 && rank == C - 1)) {
            const T* hp = heads2 + (warp * G + g) * 5 * 4 + (l - 1) * 4;
            ha = hp[0]; hb = hp[1]; hc = hp[2]; hd = hp[3];
          }
          cr_unit(A, B, Cc, D, la, lb, lc, ld, ha, hb, hc, hd);
        }
      }
    }
    stp.mark(3);
    // ---- survivors: row-blocks q = 2^kr - 1 (mod 2^kr); every rank gathers all ----
    const bool is_surv = ((q + 1) & ((1 << kr) - 1)) == 0;
    const int j = (rank * W + warp) * per_warp + (q >> kr);   // survivor index 0..m-1
    if (is_surv) {
      T* p0 = surv + g * 4 * 32 + j;
      p0[0] = A; p0[32] = B; p0[64] = Cc; p0[96] = D;
      if constexpr (C > 1) {
        T* p1 = colcta_peer<T, C>(surv, peer) + g * 4 * 32 + j;
        p1[0] = A; p1[32] = B; p1[64] = Cc; p1[96] = D;
      }
    }
    colcta_sync<C>();
    if (warp < G) {   // warp g' solves system g' (redundantly on every rank)
      const T* sp = surv + warp * 4 * 32;
      const bool v = lane < msurv;
      const T sA = v ? sp[lane] : T(0), sB = v ? sp[32 + lane] : T(1);
      const T sC = v ? sp[64 + lane] : T(0), sD = v ? sp[96 + lane] : T(0);
      const T X = lane_level_solve<T, INNER>(sA, sB, sC, sD, 0, lane & (msurv - 1), msurv);
      if (v) xs[warp * 32 + lane] = X;
    }
    __syncthreads();
    stp.mark(4);
    // ---- backward: kr levels across row-blocks, then in-lane ----
    const int jw = (rank * W + warp) * per_warp;   // this warp's first survivor
    const T xprev_warp = jw > 0 ? xs[g * 32 + jw - 1] : T(0);
    T X = is_surv ? xs[g * 32 + j] : T(0);
#pragma unroll
    for (int l = 5; l >= 1; --l) {
      if (l <= kr) {
        const int sg = 1 << (l - 1);
        T xl = __shfl_up_sync(kFull, X, sg * G);
        const T xh = __shfl_down_sync(kFull, X, sg * G);
        if ((q & (2 * sg - 1)) == sg - 1) {
          if (q < sg) xl = xprev_warp;
          X = back_unit(A, B, Cc, D, xl, xh);
        }
      }
    }
    rd[R - 1] = X;
    T xprev = __shfl_up_sync(kFull, X, G);
    if (q == 0) xprev = xprev_warp;
    inlane_backward<T, R>(ra, rbv, rc, rd, LR, xprev);
    stp.mark(5);
    if (sok) {
      T* p = x + s + i0 * es;
#pragma unroll
      for (int t = 0; t < R; ++t) p[t * es] = rd[t];
    }
    stp.mark(6);
    // the next group's head / survivor writes (after its first barrier) cannot
    // overtake this group's reads: every thread of the cluster has passed the
    // survivor barrier above, and reads of xs end before the next group's
    // survivor barrier
  }
}

}  // namespace tdg
