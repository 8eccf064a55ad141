// tridiag_colcluster.cuh -- single-pass ADI column sweep: a thread-block
// cluster keeps a group of 32 interleaved systems on chip from load to store.
//
// The two-pass column sweep (tridiag_colpass.cuh) reads a, b, c, d twice
// (~9.3 n T per system).  Here a cluster of CL CTAs owns 32
// consecutive systems (lane = system) and ALL their n = CL W R rows: CTA c
// holds rows [c W R, (c + 1) W R), warp w of it rows c W R + w R .. + R - 1,
// R per lane in registers (the column passes' unit, CL of them side by side).
// Per group of 32 systems:
//   1. the group arrives by TMA (one box {32 systems, W R rows} per array and
//      CTA, issued while the previous group computed) and moves to registers;
//      the next group's copy is issued at once (the stage is free);
//   2. the log2 R in-lane CR levels (the column passes' and the
//      on-chip kernels' inlane_forward_interior), the next warp's heads
//      through shared memory and the next CTA's through distributed shared
//      memory (cluster barrier 1), the tail chain: one survivor per warp and
//      system, n / R per system;
//   3. every survivor goes to the CTA that solves its system (system g on
//      CTA g % CL, cluster barrier 2), which solves its 32 / CL reduced systems
//      of n / R equations with the row kernels' warp_solve (the same
//      operations as the passes' reduced-row launch: bitwise the same x) and
//      sends each survivor's x back to its owner (cluster barrier 3);
//   4. the in-lane back-substitution from the registers -- no
//      second read of the input -- and x goes out as 128-byte row segments.
// HBM traffic is the algorithmic 5 n T.  One group computes per cluster at a
// time (a system's coefficients fill a register file); the stage overlaps the
// next group's load.
#pragma once

#include <cooperative_groups.h>

#include "tridiag_colpass.cuh"  // col_read_stage, col_put_heads / col_get_heads, TMA helpers

namespace tdg {

constexpr int kClusterW = 16;  // warps per CTA (512 threads, one CTA per SM)

template <typename T, int R, int CL>
struct ColCluster {
  static constexpr int W = kClusterW;
  static constexpr int LR = ilog2c(R);
  static constexpr int CH = W * R;                   // rows per CTA
  static constexpr int N = CL * CH;                  // rows per system
  static constexpr int N2 = N / R;                   // reduced equations per system
  static constexpr int NSYS = 32 / CL;               // reduced systems solved per CTA
  static constexpr int P2 = N2 / R;                  // lanes per reduced system (solve: R per lane)
  static constexpr int NSW = NSYS * P2 / 32;         // solver warps
  static constexpr int NP = N2 + N2 / W;             // padded reduced row pitch (one per CTA's W rows)
  static constexpr int HE = col_heads_elems<T, R>(); // one warp's heads [LR][4][32]
  static constexpr uint32_t ARR = 32u * CH * sizeof(T);  // one array of the stage
  static_assert(NSW >= 1 && NSYS * P2 == NSW * 32, "solver lanes must fill whole warps");
  // shared memory layout (bytes)
  static constexpr size_t OFF_BAR = 4 * (size_t)ARR;
  static constexpr size_t OFF_PAGES = OFF_BAR + 16;                          // [W][HE] (also the solver park)
  static constexpr size_t OFF_NXT = OFF_PAGES + (size_t)W * HE * sizeof(T);  // [HE] next CTA's warp-0 heads
  static constexpr size_t OFF_SURV = OFF_NXT + (size_t)HE * sizeof(T);       // [4][NSYS][NP]
  static constexpr size_t OFF_XS = OFF_SURV + 4 * (size_t)NSYS * NP * sizeof(T);  // [W + 1][32]
  static constexpr size_t OFF_LOC = OFF_XS + (size_t)(W + 1) * 32 * sizeof(T);    // [4][32][W + 1]
  static constexpr size_t OFF_SCR = (OFF_LOC + 4 * (size_t)32 * (W + 1) * sizeof(T) + 15) & ~size_t(15);
  template <int KB2>
  static constexpr size_t smem_bytes() {
    return OFF_SCR + (size_t)NSW * pcr_scratch_bytes<T, R, kPCR, KB2>();
  }
  static_assert((size_t)NSW * 32 * 4 * R * sizeof(T) <= (size_t)W * HE * sizeof(T),
                "the solver warps park their rows in the heads pages");
  static_assert(NSW * 32 * R <= 4 * 32 * (W + 1), "the solvers' x staging fits the local tile");
};

// KB2: the reduced solve's KB (as the row kernel the two-pass path launches
// for n / R equations at this m: -1 register path, else register-blocked).
template <typename T, int R, int CL, int KB2>
__global__ void __launch_bounds__(kClusterW * 32, 1)
tdg_col_cluster_kernel(const __grid_constant__ CUtensorMap tmA, const __grid_constant__ CUtensorMap tmB,
                       const __grid_constant__ CUtensorMap tmC, const __grid_constant__ CUtensorMap tmD,
                       T* x, long long es, long long S, int k2, long long* stamps) {
  namespace cg = cooperative_groups;
  using G = ColCluster<T, R, CL>;
  constexpr int W = G::W, LR = G::LR, HE = G::HE;
  pdl_entry();
  cg::cluster_group cluster = cg::this_cluster();
  const int crank = (int)cluster.block_rank();
  const long long cid = blockIdx.x / CL;
  const long long ncl = gridDim.x / CL;
  const long long groups = S >> 5;
  extern __shared__ __align__(1024) unsigned char smem_raw[];
  unsigned char* stage = smem_raw;
  uint64_t* bar = reinterpret_cast<uint64_t*>(smem_raw + G::OFF_BAR);
  T* pages = reinterpret_cast<T*>(smem_raw + G::OFF_PAGES);
  T* nxt = reinterpret_cast<T*>(smem_raw + G::OFF_NXT);
  T* surv = reinterpret_cast<T*>(smem_raw + G::OFF_SURV);
  T* xs = reinterpret_cast<T*>(smem_raw + G::OFF_XS);
  T* scr = reinterpret_cast<T*>(smem_raw + G::OFF_SCR);
  T* loc = reinterpret_cast<T*>(smem_raw + G::OFF_LOC);
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  const CUtensorMap* maps[4] = {&tmA, &tmB, &tmC, &tmD};
  auto issue = [&](long long g) {
    mbar_arrive_expect_tx(bar, 4 * G::ARR);
#pragma unroll
    for (int q = 0; q < 4; ++q)
      tma_load_2d(stage + q * G::ARR, maps[q], (int)(g * 32), crank * G::CH, bar);
  };
  if (threadIdx.x == 0) {
    mbar_init(bar, 1);
    if (cid < groups) issue(cid);
  }
  __syncthreads();
  // remote views (distributed shared memory) of the neighbours' regions
  T* nxt_prev = crank > 0 ? cluster.map_shared_rank(nxt, crank - 1) : nullptr;
  uint32_t parity = 0;
  int it = 0;
  for (long long g = cid; g < groups; g += ncl, ++it) {
    Stamp stp;
    if (stamps != nullptr && threadIdx.x < 32 && it < kStampSystems)
      stp.p = stamps + ((long long)blockIdx.x * kStampSystems + it) * kStampSlots;
    stp.mark(0);
    T ra[R], rb[R], rc[R], rd[R];
    mbar_wait(bar, parity);
    parity ^= 1;
    stp.mark(1);
    col_read_stage<T, R, W>(stage, w, lane, ra, rb, rc, rd);
    __syncthreads();  // the stage is free: the next group streams in during the solve
    if (threadIdx.x == 0 && g + ncl < groups) {
      fence_proxy_async_smem();
      issue(g + ncl);
    }
#ifdef CLU_DIAG
    stp.mark(2);
#endif
    const long long i0 = (long long)crank * G::CH + (long long)w * R;
    if (i0 == 0) ra[0] = T(0);                // a_0, c_{n-1}: not matrix entries
    if (i0 + R == G::N) rc[R - 1] = T(0);
    inlane_forward_interior<T, R, true>(ra, rb, rc, rd, LR);
#ifdef CLU_DIAG
    stp.mark(3);
#endif
    // heads of this warp for warp w - 1 (warp 0's for the previous CTA's last warp)
    if (w > 0) col_put_heads<T, R, LR>(pages + w * HE, lane, ra, rb, rc, rd);
    else if (crank > 0) col_put_heads<T, R, LR>(nxt_prev, lane, ra, rb, rc, rd);
#ifdef CLU_DIAG
    stp.mark(4);
#endif
    cluster.sync();   // 1: heads visible CTA- and cluster-wide
#ifdef CLU_DIAG
    stp.mark(5);
#else
    stp.mark(2);
#endif
    Heads<T, R> H;
    if (w + 1 < W) {
      col_get_heads<T, R, LR>(pages + (w + 1) * HE, lane, H);
    } else if (crank + 1 < CL) {
      col_get_heads<T, R, LR>(nxt, lane, H);
    } else {  // end of the system
#pragma unroll
      for (int l = 0; l < LR; ++l) { H.a[l] = T(0); H.rb[l] = T(0); H.c[l] = T(0); H.d[l] = T(0); }
    }
    inlane_tail_chain<T, R>(ra, rb, rc, rd, LR, H);
    {
      // survivors: first into a local [comp][system][warp] tile, then every
      // (solver CTA, system, comp) run of W consecutive reduced rows goes out
      // as W contiguous values (remote stores grouped by destination, not
      // 16 destinations per warp instruction)
      constexpr int WP = W + 1;
      T* lo = loc + lane * WP + w;
      lo[0] = ra[R - 1]; lo[32 * WP] = rb[R - 1]; lo[2 * 32 * WP] = rc[R - 1]; lo[3 * 32 * WP] = rd[R - 1];
      __syncthreads();
      constexpr int ITEMS = 4 * 32 * W;           // (comp, system, warp)
      for (int q = threadIdx.x; q < ITEMS; q += W * 32) {
        const int ww = q % W, gq = (q / W) % 32, comp = q / (32 * W);
        const int r2 = crank * W + ww;
        T* sv = cluster.map_shared_rank(surv, gq % CL);
        sv[comp * G::NSYS * G::NP + (gq / CL) * G::NP + r2 + r2 / W] = loc[(comp * 32 + gq) * WP + ww];
      }
    }
    cluster.sync();   // 2: this CTA's reduced systems are complete
#ifdef CLU_DIAG
    stp.mark(6);
#else
    stp.mark(3);
#endif
    if (w < G::NSW) {
      // park this warp's rows (the heads pages are free), solve, unpark
      T* pk = pages + (size_t)w * 32 * 4 * R;
#pragma unroll
      for (int t = 0; t < R; ++t) {
        pk[(4 * t + 0) * 32 + lane] = ra[t]; pk[(4 * t + 1) * 32 + lane] = rb[t];
        pk[(4 * t + 2) * 32 + lane] = rc[t]; pk[(4 * t + 3) * 32 + lane] = rd[t];
      }
      const int L = w * 32 + lane;
      const int j = L / G::P2, p = L % G::P2;      // reduced system j, lane p of it
      T sa[R], sb[R], sc[R], sd[R];
#pragma unroll
      for (int t = 0; t < R; ++t) {               // rows p R .. p R + R - 1 (padded)
        const int r2 = p * R + t;
        const int ob = j * G::NP + r2 + r2 / W;
        sa[t] = surv[ob]; sb[t] = surv[G::NSYS * G::NP + ob];
        sc[t] = surv[2 * G::NSYS * G::NP + ob]; sd[t] = surv[3 * G::NSYS * G::NP + ob];
      }
      if (p == 0) sa[0] = T(0);
      if (p == G::P2 - 1) sc[R - 1] = T(0);
      constexpr bool CYC = pcr_scratch_bytes<T, R, kPCR, KB2>() > 0;
      warp_solve<T, R, kPCR, KB2, CYC>(sa, sb, sc, sd, k2, p, G::P2, Stamp(),
                                        CYC ? scr + (size_t)w * (pcr_scratch_bytes<T, R, kPCR, KB2>() / sizeof(T)) : nullptr);
      // x of reduced row r2 belongs to CTA r2 / W, warp r2 % W, system
      // j CL + crank; the last warp's also to the next CTA (its xprev).  Staged
      // in this warp's rows of the local tile, then sent with consecutive lanes
      // on consecutive rows (one or two destinations per warp instruction).
      constexpr int SPW = 32 / G::P2;              // reduced systems per solver warp
      T* xl = loc + (size_t)w * SPW * G::N2;
#pragma unroll
      for (int t = 0; t < R; ++t) xl[(j - w * SPW) * G::N2 + p * R + t] = sd[t];
      __syncwarp();
#pragma unroll
      for (int t = 0; t < R; ++t) {
        const int item = t * 32 + lane;            // (system of this warp, row)
        const int jj = item / G::N2, r2 = item % G::N2;
        const int gs = (w * SPW + jj) * CL + crank;
        const int oc = r2 / W, ow = r2 % W;
        const T xv = xl[item];
        T* xr = cluster.map_shared_rank(xs, oc);
        xr[(ow + 1) * 32 + gs] = xv;
        if (ow == W - 1 && oc + 1 < CL) {
          T* xn = cluster.map_shared_rank(xs, oc + 1);
          xn[gs] = xv;
        }
      }
#pragma unroll
      for (int t = 0; t < R; ++t) {
        ra[t] = pk[(4 * t + 0) * 32 + lane]; rb[t] = pk[(4 * t + 1) * 32 + lane];
        rc[t] = pk[(4 * t + 2) * 32 + lane]; rd[t] = pk[(4 * t + 3) * 32 + lane];
      }
    }
    cluster.sync();   // 3: every survivor's x is home
#ifdef CLU_DIAG
    stp.mark(7);
#else
    stp.mark(4);
#endif
    const T xprev = (w == 0 && crank == 0) ? T(0) : xs[w * 32 + lane];
    rd[R - 1] = xs[(w + 1) * 32 + lane];
    inlane_backward<T, R>(ra, rb, rc, rd, LR, xprev);
    T* p = x + (g * 32 + lane) + i0 * es;
#pragma unroll
    for (int t = 0; t < R; ++t) p[t * es] = rd[t];
#ifndef CLU_DIAG
    stp.mark(5);
#endif
  }
  // no CTA may exit while a peer can still write into its shared memory
  cluster.sync();
}

}  // namespace tdg
