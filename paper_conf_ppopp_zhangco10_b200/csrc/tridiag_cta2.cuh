// tridiag_cta2.cuh -- one system per 2-CTA cluster, for the largest on-chip
// systems (fp32 n = 8192, fp64 n = 4096).  Opt-in (TRIDIAG_CTA_CLUSTER=1):
// measured slower than the single 16-warp CTA (fp32 8192: 73% vs 78% of
// HBM; fp64 4096: 69% vs 76%) -- the cross-SM hand-offs (heads, lane heads,
// survivors) sit on the per-system dependency chain, and the SM already runs
// 16 warps either way (profiles/r01_cta2_experiment.md).
//
// The TMA CTA kernel (tridiag_tma.cuh) holds such a system in one CTA of 16
// warps at ~125 registers per thread: one CTA per SM, so its barriers and its
// one-warp sections (the tails' chains, the survivors' solve) leave the SM
// idle (77-78% of HBM, against 87-97% for the 8-warp sizes that run two CTAs
// per SM).  Here the system is split over a cluster of two 8-warp CTAs on
// different SMs -- two clusters' CTAs share every SM -- and the CR steps that
// cross the split go through distributed shared memory:
//
//   * rank r holds lanes r P .. r P + P - 1 (P = 32 W, R equations per lane)
//     of the system, loaded by TMA as in the single-CTA kernel, the next
//     system's half streaming in while this one computes;
//   * in-lane CR as before; the last warp's tail chain needs the
//     next warp's head equations, which for rank 0's last warp are rank 1's
//     first warp's: rank 1 stores them into rank 0's shared memory;
//   * lane-level CR inside every warp, the same way for the lane heads;
//   * the survivors of all 2 W warps (at most 32) are exchanged, and warp 0 of
//     each rank solves them (the inner PCR / RD at m; the same
//     operations in both ranks, so the same x); back-substitution
//     (P:L294-300).
//
// The remote stores are st.async, completing transaction bytes on an
// mbarrier of the receiving CTA that only the consuming threads wait on (a
// cluster barrier per step costs a GPU-scope MEMBAR: 50% of HBM measured).
// Every operation is the one the single-CTA kernel performs on the same
// equation, so the results are bitwise identical.  The regions alternate
// between two copies by system parity: a rank writes the peer's copy of
// system s + 2 only after the peer has answered it within system s + 1,
// i.e. after the peer has finished system s.  Each mbarrier phase of system
// s completes before the peer can send anything of system s + 1 (every
// send of s + 1 waits on data the owner sends after its own waits of s).
#pragma once

#include <cooperative_groups.h>

#include "tridiag_tma.cuh"

namespace tdg {

// Remote stores into the peer CTA's shared memory that complete transaction
// bytes on the peer's mbarrier (st.async): the consumer waits on its own
// mbarrier, no cluster-wide barrier (whose release semantics cost a
// GPU-scope MEMBAR per use) is needed.
__device__ __forceinline__ uint32_t dsmem_addr(const void* local, int rank) {
  uint32_t r;
  asm volatile("mapa.shared::cluster.u32 %0, %1, %2;" : "=r"(r) : "r"(smem_u32(local)), "r"(rank));
  return r;
}
__device__ __forceinline__ void st_async(uint32_t raddr, float v, uint32_t rbar) {
  asm volatile("st.async.shared::cluster.mbarrier::complete_tx::bytes.b32 [%0], %1, [%2];" ::"r"(raddr),
               "r"(__float_as_uint(v)), "r"(rbar)
               : "memory");
}
__device__ __forceinline__ void st_async(uint32_t raddr, double v, uint32_t rbar) {
  asm volatile("st.async.shared::cluster.mbarrier::complete_tx::bytes.b64 [%0], %1, [%2];" ::"r"(raddr),
               "l"(__double_as_longlong(v)), "r"(rbar)
               : "memory");
}

// Region (elements of T): heads [W+1][LRH][4], lane heads [W+1][5][4],
// survivors [4][32], x of the survivors [32].
template <typename T, int R, int W>
__host__ __device__ constexpr int cta2_region_elems() {
  return ((W + 1) * (ilog2c(R) > 0 ? ilog2c(R) : 1) * 4 + (W + 1) * 5 * 4 + 4 * 32 + 32 + 3) & ~3;
}
template <typename T, int R, int W>
__host__ __device__ constexpr size_t cta2_smem_bytes() {
  return tma_stage_bytes<T>(R, W) + 48 + 2 * (size_t)cta2_region_elems<T, R, W>() * sizeof(T);
}

template <typename T, int R, int W, int INNER>
__global__ void __launch_bounds__(W * 32)
tdg_cta2_tma_kernel(const __grid_constant__ CUtensorMap tmA, const __grid_constant__ CUtensorMap tmB,
                    const __grid_constant__ CUtensorMap tmC, const __grid_constant__ CUtensorMap tmD,
                    T* x, int n, long long S, int k) {
  pdl_entry();
  static_assert(R * sizeof(T) == 64, "TMA stage rows are 64 bytes");
  namespace cg = cooperative_groups;
  constexpr int CL = 2;
  constexpr int P = 32 * W;  // lanes per CTA
  constexpr int LR = ilog2c(R);
  constexpr int LRH = LR > 0 ? LR : 1;
  constexpr int ROWS = P > 256 ? 256 : P;
  constexpr int NBOX = P / ROWS;
  constexpr uint32_t ARR_BYTES = P * R * sizeof(T);
  constexpr uint32_t STAGE = tma_stage_bytes<T>(R, W);
  constexpr int REG = cta2_region_elems<T, R, W>();
  extern __shared__ __align__(1024) unsigned char smem_raw[];
  unsigned char* stage = smem_raw;
  uint64_t* bar = reinterpret_cast<uint64_t*>(smem_raw + STAGE);
  // mb[0] heads, mb[1] lane heads (rank 0, from rank 1); mb[2] the peer's
  // survivors (both ranks)
  uint64_t* mb = bar + 1;
  T* region0 = reinterpret_cast<T*>(smem_raw + STAGE + 48);
  cg::cluster_group cluster = cg::this_cluster();
  const int rank = (int)cluster.block_rank();
  const long long cid = blockIdx.x / CL, ncl = gridDim.x / CL;
  const int ls = threadIdx.x, lane = ls & 31, warp = ls >> 5;
  const int gw = rank * W + warp;  // warp index within the system

  const CUtensorMap* maps[4] = {&tmA, &tmB, &tmC, &tmD};
  auto issue = [&](long long sys) {
    mbar_arrive_expect_tx(bar, 4 * ARR_BYTES);
#pragma unroll
    for (int q = 0; q < 4; ++q)
#pragma unroll
      for (int bx = 0; bx < NBOX; ++bx)
        tma_load_2d(stage + q * ARR_BYTES + bx * ROWS * 64, maps[q], 0,
                    (int)((sys * CL + rank) * P + bx * ROWS), bar);
  };
  if (ls == 0) {
    mbar_init(bar, 1);
    for (int q = 0; q < 3; ++q) mbar_init(mb + q, 1);
    if (cid < S) issue(cid);
  }
  __syncthreads();
  cluster.sync();  // the peer's mbarriers are initialised before any remote store
  const int peer = rank ^ 1;

  uint32_t parity = 0;
  int it = 0;
  for (long long sys = cid; sys < S; sys += ncl, ++it) {
    T* heads = region0 + (it & 1) * REG;          // [W+1][LRH][4]
    T* heads2 = heads + (W + 1) * LRH * 4;         // [W+1][5][4]
    T* surv = heads2 + (W + 1) * 5 * 4;            // [4][32]
    T* xs = surv + 4 * 32;                         // [32]
    mbar_wait(bar, parity);
    parity ^= 1;
    T ra[R], rb[R], rc[R], rd[R];
    const int sw = (ls >> 1) & 3;
    read_row<T, R>(stage + 0 * ARR_BYTES + ls * 64, sw, ra);
    read_row<T, R>(stage + 1 * ARR_BYTES + ls * 64, sw, rb);
    read_row<T, R>(stage + 2 * ARR_BYTES + ls * 64, sw, rc);
    read_row<T, R>(stage + 3 * ARR_BYTES + ls * 64, sw, rd);
    if (rank == 0 && ls == 0) ra[0] = T(0);
    if (rank == CL - 1 && ls == P - 1) rc[R - 1] = T(0);

    const int kr = k - LR;
    const int kl = kr < 5 ? kr : 5;
    const int per_warp = 32 >> kl;
    const int msurv = CL * W * per_warp;  // <= 32 (checked by the launcher)
    const uint32_t ph = (uint32_t)(it & 1);
    if (ls == 0) {
      // this system's transaction bytes on the mbarriers the peer completes
      if (rank == 0) {
        mbar_arrive_expect_tx(mb + 0, LR * 4 * (uint32_t)sizeof(T));
        mbar_arrive_expect_tx(mb + 1, kl * 4 * (uint32_t)sizeof(T));
      }
      mbar_arrive_expect_tx(mb + 2, W * per_warp * 4 * (uint32_t)sizeof(T));
    }

    // ---- in-lane CR forward (k >= log2 R: all in-lane levels) ----
    inlane_forward_interior<T, R>(ra, rb, rc, rd, LR);
    Heads<T, R> H;
    heads_from_next_lane<T, R>(ra, rb, rc, rd, LR, 32, false, H);
    if (lane == 0 && warp > 0) {
      // this warp's head equations are what the previous warp's tail needs
#pragma unroll
      for (int l = 1; l <= LR; ++l) {
        const int t = (1 << (l - 1)) - 1;
        T* hp = heads + (warp * LRH + (l - 1)) * 4;
        hp[0] = ra[t]; hp[1] = rb[t]; hp[2] = rc[t]; hp[3] = rd[t];
      }
    } else if (lane == 0 && rank > 0) {
      // rank 1's first warp: into rank 0's slot W
      const uint32_t rh = dsmem_addr(heads + W * LRH * 4, peer), rbar = dsmem_addr(mb + 0, peer);
#pragma unroll
      for (int l = 1; l <= LR; ++l) {
        const int t = (1 << (l - 1)) - 1;
        const uint32_t hp = rh + (uint32_t)((l - 1) * 4 * sizeof(T));
        st_async(hp, ra[t], rbar); st_async(hp + sizeof(T), rb[t], rbar);
        st_async(hp + 2 * sizeof(T), rc[t], rbar); st_async(hp + 3 * sizeof(T), rd[t], rbar);
      }
    }
    __syncthreads();  // B1 (local): heads visible; every thread has read its stage
    if (ls == 0 && sys + ncl < S) issue(sys + ncl);
    const bool has_next = warp + 1 < W || rank + 1 < CL;
    if (lane == 31) {
      if (warp + 1 == W && has_next) mbar_wait(mb + 0, ph);  // rank 0's last warp
#pragma unroll
      for (int l = 1; l <= LR; ++l) {
        if (has_next) {
          const T* hp = heads + ((warp + 1) * LRH + (l - 1)) * 4;
          H.a[l - 1] = hp[0]; H.rb[l - 1] = hp[1]; H.c[l - 1] = hp[2]; H.d[l - 1] = hp[3];
        } else {
          H.a[l - 1] = T(0); H.rb[l - 1] = T(0); H.c[l - 1] = T(0); H.d[l - 1] = T(0);
        }
      }
    }
    inlane_tail_chain<T, R>(ra, rb, rc, rd, LR, H);

    // ---- lane-level CR inside every warp (the register path of the CTA kernel) ----
    T A = ra[R - 1], B = rb[R - 1], C = rc[R - 1], D = rd[R - 1];
#pragma unroll
    for (int l = 1; l <= 5; ++l) {
      if (l <= kl) {
        const int sg = 1 << (l - 1);
        const int md = lane & (2 * sg - 1);
        if (md == sg - 1) B = Arith<T>::rcp(B);
        const T la = shup(A, sg, 32), lb = shup(B, sg, 32), lc = shup(C, sg, 32), ld = shup(D, sg, 32);
        const T ha = shdn(A, sg, 32), hb = shdn(B, sg, 32), hc = shdn(C, sg, 32), hd = shdn(D, sg, 32);
        if (md == 2 * sg - 1 && lane != 31) cr_unit(A, B, C, D, la, lb, lc, ld, ha, hb, hc, hd);
      }
    }
    if (((lane + 1) & lane) == 0 && lane < (1 << (kl - 1))) {
      const int l = ilog2c(lane + 1);  // lane = 2^l - 1 -> level l + 1
      if (warp > 0) {
        T* hp = heads2 + (warp * 5 + l) * 4;
        hp[0] = A; hp[1] = B; hp[2] = C; hp[3] = D;
      } else if (rank > 0) {
        const uint32_t hp = dsmem_addr(heads2 + (W * 5 + l) * 4, peer), rbar = dsmem_addr(mb + 1, peer);
        st_async(hp, A, rbar); st_async(hp + sizeof(T), B, rbar);
        st_async(hp + 2 * sizeof(T), C, rbar); st_async(hp + 3 * sizeof(T), D, rbar);
      }
    }
    __syncthreads();  // B2 (local): lane heads visible
    if (lane == 31 && warp + 1 == W && has_next) mbar_wait(mb + 1, ph);
#pragma unroll
    for (int l = 1; l <= 5; ++l) {
      if (l <= kl) {
        const int sg = 1 << (l - 1);
        const T la = __shfl_sync(kFull, A, 31 - sg), lb = __shfl_sync(kFull, B, 31 - sg);
        const T lc = __shfl_sync(kFull, C, 31 - sg), ld = __shfl_sync(kFull, D, 31 - sg);
        if (lane == 31) {
          T ha = T(0), hb = T(0), hc = T(0), hd = T(0);
          if (has_next) {
            const T* hp = heads2 + ((warp + 1) * 5 + (l - 1)) * 4;
            ha = hp[0]; hb = hp[1]; hc = hp[2]; hd = hp[3];
          }
          cr_unit(A, B, C, D, la, lb, lc, ld, ha, hb, hc, hd);
        }
      }
    }
    // survivors: lanes 2^kl - 1 (mod 2^kl) of every warp of both ranks, to rank 0
    const bool is_surv = ((lane + 1) & ((1 << kl) - 1)) == 0;
    const int j = gw * per_warp + (lane >> kl);
    if (is_surv) {
      // both ranks hold all survivors: own ones locally, the peer's by st.async
      surv[j] = A; surv[32 + j] = B; surv[64 + j] = C; surv[96 + j] = D;
      const uint32_t sv = dsmem_addr(surv, peer), rbar = dsmem_addr(mb + 2, peer);
      st_async(sv + (uint32_t)(j * sizeof(T)), A, rbar);
      st_async(sv + (uint32_t)((32 + j) * sizeof(T)), B, rbar);
      st_async(sv + (uint32_t)((64 + j) * sizeof(T)), C, rbar);
      st_async(sv + (uint32_t)((96 + j) * sizeof(T)), D, rbar);
    }
    __syncthreads();  // B3 (local): this rank's survivors
    if (warp == 0) {
      // each rank solves the survivors itself (same operations: same bits),
      // so no x travels between the SMs
      mbar_wait(mb + 2, ph);  // the peer's survivors
      const bool v = lane < msurv;
      const T sA = v ? surv[lane] : T(0), sB = v ? surv[32 + lane] : T(1);
      const T sC = v ? surv[64 + lane] : T(0), sD = v ? surv[96 + lane] : T(0);
      const T X = lane_level_solve<T, INNER>(sA, sB, sC, sD, kr - kl, lane & (msurv - 1), msurv);
      if (v) xs[lane] = X;
    }
    __syncthreads();  // B4 (local): x of the survivors
    const T xprev_warp = gw > 0 ? xs[gw * per_warp - 1] : T(0);
    T X = is_surv ? xs[j] : T(0);
#pragma unroll
    for (int l = 5; l >= 1; --l) {
      if (l <= kl) {
        const int sg = 1 << (l - 1);
        T xl = shup(X, sg, 32);
        const T xh = shdn(X, sg, 32);
        if ((lane & (2 * sg - 1)) == sg - 1) {
          if (lane < sg) xl = xprev_warp;
          X = back_unit(A, B, C, D, xl, xh);
        }
      }
    }
    rd[R - 1] = X;
    const T xup = shup(X, 1, 32);
    const T xprev = lane > 0 ? xup : xprev_warp;
    inlane_backward<T, R>(ra, rb, rc, rd, LR, xprev);
    store_block<T, R>(x + (size_t)sys * (size_t)n + (size_t)(rank * P + ls) * R, rd, true);
  }
  // no CTA may exit while its peer can still store into its shared memory
  cluster.sync();
}

}  // namespace tdg
