// tridiag_kernels.cuh -- the two kernel families of libtridiag (sm_100a).
//
// Both run ONE algorithm template for all five methods of the paper: k CR
// levels around an inner PCR or RD on
// the m = n >> k intermediate equations (Fig 4).  CR is the case
// m = 2 with the PCR inner (a single 2-unknown solve); PCR and RD
// are k = 0.  The endpoint identities of Fig 17 therefore hold
// bitwise by construction.
//
//  * tdg_warp_kernel<T, R, INNER>: P = n/R <= 32 lanes per system (32/P
//    systems per warp), registers + shuffles only when m <= P; persistent
//    grid-stride loop over warp-groups of systems.
//  * tdg_cta_kernel<T, R, W, INNER>: P = 32W lanes (W warps) per system, one
//    system per CTA at a time: in-lane CR in registers, the P surviving
//    equations are reduced in shared memory with even/odd-compacted CR levels
//    (conflict-light; the fix the paper suggests at P:L822-824) down to 32 (or
//    m), then one warp finishes with shuffles.
#pragma once

#include "tridiag_device.cuh"

#ifndef TDG_BLOCKED_MINB
#define TDG_BLOCKED_MINB 2
#endif
// 4-warp CTAs per SM of the small-CTA PCR kernels (pcr_small_cta): 3 for PCR
// alone (151 registers, no spills), one more for CR+PCR with one CR level
// (127 registers, no spills): measured 44.0 vs 41.8% and 82.7 vs 75.1% of HBM
#ifndef TDG_PCR_SMALL_MINB
#define TDG_PCR_SMALL_MINB 3
#endif
#ifndef TDG_PCR_SMALL_MINB_K1
#define TDG_PCR_SMALL_MINB_K1 4
#endif
// CTAs per SM the LU-form RD kernel asks for (its three scans want ~185
// registers: 1 CTA of 8 warps, or 2 with spills)
#ifndef TDG_STONE_MINB
#define TDG_STONE_MINB 2
#endif

namespace tdg {

// ============================================================================
// Warp kernel.
// ============================================================================
// Phase stamps: the paper times its solvers phase
// by phase (Figs 8, 11, 13, 15, 16).  When the launch passes a
// stamp buffer, lane 0 of warp 0 of every CTA records clock64() at the phase
// boundaries of its first kStampSystems system groups (no effect otherwise).
constexpr int kStampSystems = 4;
constexpr int kStampSlots = 8;
struct Stamp {
  long long* p = nullptr;
  __device__ __forceinline__ void mark(int slot) const {
    if (p != nullptr && (threadIdx.x & 31) == 0) p[slot] = clock64();
  }
};

// KB < 0: k >= LR (all in-lane levels; m <= P, lane-level inner solve).
// KB >= 0: k == KB < LR (m = P * (R >> KB) > P, register-blocked inner solve).
// PCR_CYC: pcr_scratch is the warp's cyclic-relayout scratch (blocked PCR).
template <typename T, int R, int INNER, int KB, bool PCR_CYC = false>
__device__ __forceinline__ void warp_solve(T (&a)[R], T (&b)[R], T (&c)[R], T (&d)[R], int k,
                                           int ls, int P, Stamp st = Stamp(),
                                           T* pcr_scratch = nullptr) {
  constexpr int LR = ilog2c(R);
  constexpr int kin = KB < 0 ? LR : KB;
  inlane_forward_interior<T, R>(a, b, c, d, kin);
  st.mark(1);
  Heads<T, R> H;
  heads_from_next_lane<T, R>(a, b, c, d, kin, P, ls == P - 1, H);
  inlane_tail_chain<T, R>(a, b, c, d, kin, H);
  st.mark(2);
  if constexpr (INNER == kSTONE) {
    // overflow-free LU-form RD on the whole system (k = 0, kin = 0)
    blocked_stone<T, R>(a, b, c, d, ls, P);
  } else if constexpr (KB < 0) {
    d[R - 1] = lane_level_solve<T, INNER>(a[R - 1], b[R - 1], c[R - 1], d[R - 1], k - LR, ls, P);
  } else {
    // m = P * (R >> KB) > P: the intermediate system stays block-distributed
    // in registers (no copy; the paper copies it to 5 extra arrays).
    if constexpr (INNER == kPCR) blocked_pcr<T, R, (KB < 0 ? 0 : KB), PCR_CYC>(a, b, c, d, ls, P, pcr_scratch);
    else blocked_rd<T, R, (KB < 0 ? 0 : KB)>(a, b, c, d, ls, P);
  }
  st.mark(3);
  T xprev = __shfl_up_sync(kFull, d[R - 1], 1, P);
  if (ls == 0) xprev = T(0);
  inlane_backward<T, R>(a, b, c, d, kin, xprev);
  st.mark(4);
}

// ---- warp-staged general path (contiguous rows of any length / alignment) ----
// Per-warp shared tile of 32R elements per array (the warp's G systems of
// n_pad = P R equations, back to back), element q at q + (q >> 5).
template <typename T, int R>
__host__ __device__ constexpr int warp_tile_elems() { return 32 * R + R + 1; }
template <typename T, int R>
__device__ __forceinline__ T* warp_tile(int warp) {
  extern __shared__ __align__(1024) unsigned char smem_raw[];
  return reinterpret_cast<T*>(smem_raw) + (size_t)warp * 4 * warp_tile_elems<T, R>();
}
__device__ __forceinline__ int wt_off(int q) { return q + (q >> 5); }

// The warp's tile holds 32R elements per array, so every lane moves exactly R
// of them: element q = lane + 32 j (j < R, unrolled so all 4R loads are in
// flight together) is equation i = q mod n_pad of system s0 + q / n_pad.
template <typename T, int R>
__device__ __forceinline__ void staged_load(const T* a, const T* b, const T* c, const T* d,
                                            long long s0, long long S, long long ss, int n_pad,
                                            int n_real, T c_pad, int log2n, int lane,
                                            T (&ra)[R], T (&rb)[R], T (&rc)[R], T (&rd)[R],
                                            T* tile) {
  constexpr int TE = warp_tile_elems<T, R>();
  T* tA = tile;
  T* tB = tile + TE;
  T* tC = tile + 2 * TE;
  T* tD = tile + 3 * TE;
  T va[R], vb[R], vc[R], vd[R];
#pragma unroll
  for (int j = 0; j < R; ++j) {
    const int q = lane + 32 * j;
    const int g = q >> log2n, i = q & (n_pad - 1);
    const long long sys = s0 + g;
    const bool v = sys < S && i < n_real;
    const size_t e = (size_t)sys * (size_t)ss + i;
    va[j] = v ? a[e] : T(0);
    vb[j] = v ? b[e] : T(1);
    vc[j] = v ? (i == n_real - 1 ? c_pad : c[e]) : c_pad;
    vd[j] = v ? d[e] : T(0);
  }
#pragma unroll
  for (int j = 0; j < R; ++j) {
    const int o = wt_off(lane + 32 * j);
    tA[o] = va[j]; tB[o] = vb[j]; tC[o] = vc[j]; tD[o] = vd[j];
  }
  __syncwarp();
#pragma unroll
  for (int t = 0; t < R; ++t) {
    const int o = wt_off(lane * R + t);
    ra[t] = tA[o]; rb[t] = tB[o]; rc[t] = tC[o]; rd[t] = tD[o];
  }
  __syncwarp();
}

template <typename T, int R>
__device__ __forceinline__ void staged_store(T* x, long long s0, long long S, long long ss,
                                             int n_pad, int n_real, int log2n, int lane,
                                             const T (&rd)[R], T* tile) {
  T* tD = tile + 3 * warp_tile_elems<T, R>();
#pragma unroll
  for (int t = 0; t < R; ++t) tD[wt_off(lane * R + t)] = rd[t];
  __syncwarp();
#pragma unroll
  for (int j = 0; j < R; ++j) {
    const int q = lane + 32 * j;
    const int g = q >> log2n, i = q & (n_pad - 1);
    const long long sys = s0 + g;
    if (sys < S && i < n_real) x[(size_t)sys * (size_t)ss + i] = tD[wt_off(q)];
  }
  __syncwarp();
}

// GEN = false: contiguous power-of-two systems with aligned pointers (vector
// loads only).  GEN = true: the general path -- scalar loads, element / system
// strides, padded (ragged) n -- compiled separately so the fast path carries
// none of its registers.
// RAG = true (with GEN = false): ragged contiguous rows (system stride
// n_real, n_real T a multiple of 16 B, 16-byte aligned pointers): each lane
// moves its R equations with 16-byte vector accesses when they are all real,
// element by element (padding equations of reading R26 past n_real) at the
// end of a system -- no shared-memory staging.
template <typename T, bool NC>
__device__ __forceinline__ void ld16B(const T* p, T* v) {
  if constexpr (sizeof(T) == 4) {
    const float4 t = NC ? __ldg(reinterpret_cast<const float4*>(p)) : *reinterpret_cast<const float4*>(p);
    v[0] = t.x; v[1] = t.y; v[2] = t.z; v[3] = t.w;
  } else {
    const double2 t = NC ? __ldg(reinterpret_cast<const double2*>(p)) : *reinterpret_cast<const double2*>(p);
    v[0] = t.x; v[1] = t.y;
  }
}
template <typename T>
__device__ __forceinline__ void st16B(T* p, const T* v) {
  if constexpr (sizeof(T) == 4)
    *reinterpret_cast<float4*>(p) = make_float4(v[0], v[1], v[2], v[3]);
  else
    *reinterpret_cast<double2*>(p) = make_double2(v[0], v[1]);
}

// A lane block of B = R T bytes at a 16-byte aligned address: 32-byte
// accesses (one full sector each) wherever the block allows -- all of it when
// the address is 32-byte aligned, else a 16-byte head, (B - 32) / 32 full
// sectors and a 16-byte tail -- instead of B / 16 half-sector accesses (which
// cost twice the L1 / L2 requests: ragged n = 500 fp32 measured 1.3x slower
// than n = 512).
template <typename T, int R, bool NC>
__device__ __forceinline__ void load_block16(const T* p, T (&v)[R]) {
  constexpr int E = 16 / (int)sizeof(T);
  constexpr int B = R * (int)sizeof(T);
  if constexpr (R % E != 0) {  // (not launched: the host requires 16-byte lane blocks)
#pragma unroll
    for (int t = 0; t < R; ++t) v[t] = p[t];
  } else if constexpr (B % 32 == 0 && B >= 64) {
    if ((reinterpret_cast<uintptr_t>(p) & 31) == 0) {
#pragma unroll
      for (int q = 0; q < B / 32; ++q) ld32B<NC>(p + q * 2 * E, v + q * 2 * E);
    } else {
      ld16B<T, NC>(p, v);
#pragma unroll
      for (int q = 0; q < B / 32 - 1; ++q) ld32B<NC>(p + E + q * 2 * E, v + E + q * 2 * E);
      ld16B<T, NC>(p + R - E, v + R - E);
    }
  } else {
#pragma unroll
    for (int q = 0; q < R / E; ++q) ld16B<T, NC>(p + q * E, v + q * E);
  }
}
template <typename T, int R>
__device__ __forceinline__ void store_block16(T* p, const T (&v)[R]) {
  constexpr int E = 16 / (int)sizeof(T);
  constexpr int B = R * (int)sizeof(T);
  if constexpr (R % E != 0) {  // (not launched: the host requires 16-byte lane blocks)
#pragma unroll
    for (int t = 0; t < R; ++t) p[t] = v[t];
  } else if constexpr (B % 32 == 0 && B >= 64) {
    if ((reinterpret_cast<uintptr_t>(p) & 31) == 0) {
#pragma unroll
      for (int q = 0; q < B / 32; ++q) st32B(p + q * 2 * E, v + q * 2 * E);
    } else {
      st16B<T>(p, v);
#pragma unroll
      for (int q = 0; q < B / 32 - 1; ++q) st32B(p + E + q * 2 * E, v + E + q * 2 * E);
      st16B<T>(p + R - E, v + R - E);
    }
  } else {
#pragma unroll
    for (int q = 0; q < R / E; ++q) st16B<T>(p + q * E, v + q * E);
  }
}

// L2 prefetch of a warp kernel's first system group before the dependent-launch
// wait (see tdg_cta_tma_kernel): contiguous power-of-two rows only.
template <typename T, int R>
__device__ __forceinline__ void warp_prefetch_first(const T* a, const T* b, const T* c, const T* d,
                                                    int n, long long S, int log2P, int vec, int pf,
                                                    long long ss) {
  const int lane = threadIdx.x & 31;
  if (!vec || !(pf & 2) || ss != n || lane >= 4) return;
  const int wpb = blockDim.x >> 5;
  const int G = 32 >> log2P;
  const long long s0 = ((long long)blockIdx.x * wpb + (threadIdx.x >> 5)) * G;
  if (s0 >= S) return;
  const long long cnt = (S - s0) < G ? (S - s0) : G;
  const T* base = lane == 0 ? a : lane == 1 ? b : lane == 2 ? c : d;
  const uint32_t bytes = (uint32_t)(cnt * n * sizeof(T));
  if (bytes % 16 == 0) prefetch_l2(base + (size_t)s0 * n, bytes);
}

// LP >= 0: lanes per system P = 2^LP fixed at compile time (log2P ignored), so
// every step guard of the blocked inner solvers folds and their shuffles
// have a compile-time width (no divergent-shuffle fallbacks).
template <typename T, int R, int INNER, int KB, bool GEN, bool RAG = false, int LP = -1>
__device__ __forceinline__ void warp_kernel_body(
    const T* __restrict__ a, const T* __restrict__ b, const T* __restrict__ c, const T* d, T* x,
    int n, long long S, int k, int log2P_rt, int vec, int pf, int n_real, T c_pad, long long es,
    long long ss, long long* stamps) {
  const int log2P = LP >= 0 ? LP : log2P_rt;
  const int P = 1 << log2P;
  const int lane = threadIdx.x & 31;
  const int warp = threadIdx.x >> 5;
  const int wpb = blockDim.x >> 5;
  const int G = 32 >> log2P;  // systems per warp
  const int sub = lane >> log2P;
  const int ls = lane & (P - 1);
  const long long step = (long long)gridDim.x * wpb * G;
  // per-warp scratch of the cyclic PCR relayout, after the GEN warp tiles
  T* pcr_scr = nullptr;
  if constexpr (pcr_scratch_bytes<T, R, INNER, KB>() > 0) {
    extern __shared__ __align__(1024) unsigned char smem_raw[];
    const size_t off = GEN ? (((size_t)wpb * 4 * warp_tile_elems<T, R>() * sizeof(T) + 15) & ~size_t(15)) : 0;
    pcr_scr = reinterpret_cast<T*>(smem_raw + off + (size_t)warp * pcr_scratch_bytes<T, R, INNER, KB>());
  }
  int iter = 0;
  for (long long s0 = ((long long)blockIdx.x * wpb + warp) * G; s0 < S; s0 += step, ++iter) {
    Stamp stp;
    if (stamps != nullptr && warp == 0 && iter < kStampSystems)
      stp.p = stamps + ((long long)blockIdx.x * kStampSystems + iter) * kStampSlots;
    stp.mark(0);
    if ((pf & 1) && lane < 4 && s0 + step < S) {
      // lanes 0..3 prefetch array a, b, c, d of this warp's next group
      const long long nx = s0 + step;
      const long long cnt = (S - nx) < G ? (S - nx) : G;
      const T* base = lane == 0 ? a : lane == 1 ? b : lane == 2 ? c : d;
      prefetch_l2(base + (size_t)nx * n, (uint32_t)(cnt * n * sizeof(T)));
    }
    const long long sys = s0 + sub;
    const bool valid = sys < S;
    const size_t sbase = (size_t)sys * (size_t)ss;
    const size_t off = sbase + (size_t)ls * R;
    T ra[R], rb[R], rc[R], rd[R];
    if constexpr (RAG) {
      const int i0 = ls * R;
      if (valid && i0 + R <= n_real) {
        load_block16<T, R, true>(a + off, ra);
        load_block16<T, R, true>(b + off, rb);
        load_block16<T, R, true>(c + off, rc);
        load_block16<T, R, false>(d + off, rd);
      } else {
#pragma unroll
        for (int t = 0; t < R; ++t) {
          const bool in = valid && i0 + t < n_real;
          ra[t] = in ? a[off + t] : T(0);
          rb[t] = in ? b[off + t] : T(1);
          rc[t] = in ? c[off + t] : c_pad;
          rd[t] = in ? d[off + t] : T(0);
        }
      }
      if (i0 + R >= n_real) {
#pragma unroll
        for (int t = 0; t < R; ++t)
          if (i0 + t == n_real - 1) rc[t] = c_pad;  // c_{n_real-1} (R26)
      }
    } else if constexpr (!GEN) {
      if (valid) {
        load_block<T, R, true>(a + off, ra, vec);
        load_block<T, R, true>(b + off, rb, vec);
        load_block<T, R, true>(c + off, rc, vec);
        load_block<T, R, false>(d + off, rd, vec);
      } else {
#pragma unroll
        for (int i = 0; i < R; ++i) { ra[i] = T(0); rb[i] = T(1); rc[i] = T(0); rd[i] = T(0); }
      }
    } else {
      // General contiguous rows (ragged n, misaligned or pitched): the warp
      // reads its G systems with coalesced, lane-consecutive loads into a
      // per-warp shared tile (padded one element per 32, so the lane-blocked
      // reads below are bank-conflict free), padding included.
      staged_load<T, R>(a, b, c, d, s0, S, ss, n, n_real, c_pad, log2P + ilog2c(R), lane, ra, rb,
                        rc, rd, warp_tile<T, R>(warp));
    }
    // a_0 and c_{n-1} are not matrix entries: never read.
    if (ls == 0) ra[0] = T(0);
    if (ls == P - 1) rc[R - 1] = T(0);
    warp_solve<T, R, INNER, KB, (pcr_scratch_bytes<T, R, INNER, KB>() > 0)>(ra, rb, rc, rd, k, ls, P, stp, pcr_scr);
    if constexpr (RAG) {
      const int i0 = ls * R;
      if (valid) {
        if (i0 + R <= n_real) {
          store_block16<T, R>(x + off, rd);
        } else {
#pragma unroll
          for (int t = 0; t < R; ++t)
            if (i0 + t < n_real) x[off + t] = rd[t];
        }
      }
    } else if constexpr (!GEN) {
      if (valid) store_block<T, R>(x + off, rd, vec);
    } else {
      staged_store<T, R>(x, s0, S, ss, n, n_real, log2P + ilog2c(R), lane, rd, warp_tile<T, R>(warp));
    }
    stp.mark(5);
  }
}

// KB < 0 (the register path of the tuned hybrids and CR): ptxas picks ~127
// registers for 256 threads, two CTAs (16 warps) per SM.
template <typename T, int R, int INNER, int KB, bool GEN, bool RAG = false>
__global__ void __launch_bounds__(256)
tdg_warp_kernel(const T* __restrict__ a, const T* __restrict__ b, const T* __restrict__ c,
                const T* d, T* x, int n, long long S, int k, int log2P, int vec, int pf,
                int n_real, T c_pad, long long es, long long ss, long long* stamps) {
  if constexpr (!GEN && !RAG) warp_prefetch_first<T, R>(a, b, c, d, n, S, log2P, vec, pf, ss);
  pdl_entry();
  warp_kernel_body<T, R, INNER, KB, GEN, RAG>(a, b, c, d, x, n, S, k, log2P, vec, pf, n_real, c_pad,
                                              es, ss, stamps);
}

// KB >= 0 (register-blocked inner: PCR, RD, large m) is latency bound with
// one 8-warp CTA per SM at ~170 registers; asking for two CTAs (<= 128
// registers; the few spills land in the otherwise unused L1) doubles the
// warps that hide the shuffle / MUFU latency.
// SMALL: PCR alone in fp32 (k = 0, vector path, P >= 16 lanes per system):
// 4-warp CTAs, 3 per SM, 170 registers (12 warps per SM, fewer spills than
// at the 2-CTA cap); n = 64 / 128 (P < 16) are faster with the default.
template <typename T, int R, int INNER, int KB, bool GEN>
__host__ __device__ constexpr bool pcr_small_cta() {
  return INNER == kPCR && (KB == 0 || KB == 1) && !GEN &&
         ((sizeof(T) == 4 && R == 16) || (sizeof(T) == 8 && R == 8));
}
template <typename T, int R, int INNER, int KB, bool GEN, bool SMALL = false, int LP = -1>
__global__ void __launch_bounds__(SMALL ? 128 : 256,
                                  SMALL ? (KB == 0 ? TDG_PCR_SMALL_MINB : TDG_PCR_SMALL_MINB_K1) : (R >= 8 && INNER != kSTONE) ? TDG_BLOCKED_MINB : TDG_STONE_MINB)
tdg_warp_blocked_kernel(const T* __restrict__ a, const T* __restrict__ b, const T* __restrict__ c,
                        const T* d, T* x, int n, long long S, int k, int log2P, int vec, int pf,
                        int n_real, T c_pad, long long es, long long ss, long long* stamps) {
  if constexpr (!GEN) warp_prefetch_first<T, R>(a, b, c, d, n, S, LP >= 0 ? LP : log2P, vec, pf, ss);
  pdl_entry();
  warp_kernel_body<T, R, INNER, KB, GEN, false, LP>(a, b, c, d, x, n, S, k, log2P, vec, pf, n_real, c_pad,
                                         es, ss, stamps);
}

// ============================================================================
// CTA kernel (n > 32 R): W warps per system.
// Shared memory layout (elements of T):
//   heads  [W][LR][4]                      next-warp head equations
//   case k >= LR:  lev[5][2P]  (A, B, C, D, X of the compacted CR levels;
//                   level l of P>>l equations at offset 2P - 2(P>>l))
//                  + inner region for m > 32
//   case k <  LR:  inner region for m = P * (R >> k)
// ============================================================================
// In-lane CR (heads of the next warp through shared memory, one barrier) for
// a CTA that owns one system; AfterB1 runs right after that barrier (the TMA
// kernel issues the next system's copy there: every thread has consumed its
// staged input by then).
template <typename T, int R, int W, class AfterB1>
__device__ __forceinline__ void cta_inlane_forward(T (&ra)[R], T (&rb)[R], T (&rc)[R], T (&rd)[R],
                                                   int kin, T* heads, AfterB1 after_b1) {
  constexpr int LR = ilog2c(R);
  constexpr int LRH = LR > 0 ? LR : 1;
  const int ls = threadIdx.x;
  const int lane = ls & 31;
  const int warp = ls >> 5;
    inlane_forward_interior<T, R, true>(ra, rb, rc, rd, kin);
    // Heads: lanes 0..30 take them from lane+1 by shuffle; lane 31 of warp w
    // takes warp w+1's lane 0 through shared memory.
    Heads<T, R> H;
    heads_from_next_lane<T, R>(ra, rb, rc, rd, kin, 32, false, H);
    if (lane == 0 && warp > 0) {
#pragma unroll
      for (int l = 1; l <= LR; ++l) {
        if (l <= kin) {
          const int t = (1 << (l - 1)) - 1;
          T* hp = heads + (warp * LRH + (l - 1)) * 4;
          hp[0] = ra[t]; hp[1] = rb[t]; hp[2] = rc[t]; hp[3] = rd[t];
        }
      }
    }
    __syncthreads();
    after_b1();
    if (lane == 31) {
#pragma unroll
      for (int l = 1; l <= LR; ++l) {
        if (l <= kin) {
          if (warp + 1 < W) {
            const T* hp = heads + ((warp + 1) * LRH + (l - 1)) * 4;
            H.a[l - 1] = hp[0]; H.rb[l - 1] = hp[1]; H.c[l - 1] = hp[2]; H.d[l - 1] = hp[3];
          } else {
            H.a[l - 1] = T(0); H.rb[l - 1] = T(0); H.c[l - 1] = T(0); H.d[l - 1] = T(0);
          }
        }
      }
    }
    inlane_tail_chain<T, R>(ra, rb, rc, rd, kin, H);

}

// Survivor hand-off on a named barrier (producer warps arrive, the solver
// warp waits) instead of a CTA barrier + warp 0 (A/B: 0 = the round-1 path).
#ifndef TDG_SURV_NAMED_BARRIER
#define TDG_SURV_NAMED_BARRIER 1
#endif
// Register path (k >= log2 R, m <= 32 lanes or m = survivors): lane-level CR
// inside every warp, survivors solved by one warp or by the CTA in shared
// memory, back-substitution.  Returns xprev for the in-lane back-substitution
// and leaves x of the lane's tail in rd[R-1].
template <typename T, int R, int W, int INNER>
__device__ __forceinline__ T cta_register_path(T (&ra)[R], T (&rb)[R], T (&rc)[R], T (&rd)[R],
                                               int k, T* heads, Stamp stp = Stamp()) {
  constexpr int P = 32 * W;
  constexpr int LR = ilog2c(R);
  constexpr int LRH = LR > 0 ? LR : 1;
  const int ls = threadIdx.x;
  const int lane = ls & 31;
  const int warp = ls >> 5;
  T xprev;
    // ---- lane-level CR inside every warp (shuffles), kl levels ----
    const int kr = k - LR;                 // CR levels left after the in-lane ones
    const int kl = kr < 5 ? kr : 5;        // of which across the lanes of a warp
    T A = ra[R - 1], B = rb[R - 1], C = rc[R - 1], D = rd[R - 1];
    // interior: every update lane except the warp's tail (lane 31)
#pragma unroll
    for (int l = 1; l <= 5; ++l) {
      if (l <= kl) {
        const int sg = 1 << (l - 1);
        const int md = lane & (2 * sg - 1);
        const T rcB = rcp1(B);  // every lane (no divergent slow-path branch)
        if (md == sg - 1) B = rcB;
        const T la = shup(A, sg, 32), lb = shup(B, sg, 32), lc = shup(C, sg, 32), ld = shup(D, sg, 32);
        const T ha = shdn(A, sg, 32), hb = shdn(B, sg, 32), hc = shdn(C, sg, 32), hd = shdn(D, sg, 32);
        if (md == 2 * sg - 1 && lane != 31) cr_unit(A, B, C, D, la, lb, lc, ld, ha, hb, hc, hd);
      }
    }
    // lane heads of warp w (lanes 2^(l-1)-1, final state) for warp w-1's tail
    T* heads2 = heads + W * LRH * 4;                 // [W][5][4]
    T* surv = heads2 + W * 5 * 4;                    // [4][P] survivors (m_surv <= 32)
    T* xs = surv + 4 * P;                            // [P]
    T* inner = xs + P;                               // inner region (m_surv > 32)
    if (warp > 0 && ((lane + 1) & lane) == 0 && lane < (1 << (kl - 1))) {
      const int l = ilog2c(lane + 1);               // lane = 2^l - 1 -> level l+1
      T* hp = heads2 + (warp * 5 + l) * 4;
      hp[0] = A; hp[1] = B; hp[2] = C; hp[3] = D;
    }
    __syncthreads();
    // tail chain of lane 31: lower neighbour lane 31-sg (final), upper = next warp's head
#pragma unroll
    for (int l = 1; l <= 5; ++l) {
      if (l <= kl) {
        const int sg = 1 << (l - 1);
        const T la = __shfl_sync(kFull, A, 31 - sg), lb = __shfl_sync(kFull, B, 31 - sg);
        const T lc = __shfl_sync(kFull, C, 31 - sg), ld = __shfl_sync(kFull, D, 31 - sg);
        if (lane == 31) {
          T ha = T(0), hb = T(0), hc = T(0), hd = T(0);
          if (warp + 1 < W) {
            const T* hp = heads2 + ((warp + 1) * 5 + (l - 1)) * 4;
            ha = hp[0]; hb = hp[1]; hc = hp[2]; hd = hp[3];
          }
          cr_unit(A, B, C, D, la, lb, lc, ld, ha, hb, hc, hd);
        }
      }
    }
    stp.mark(3);
    // survivors: lanes 2^kl - 1 (mod 2^kl) of every warp
    const int per_warp = 32 >> kl;
    const int msurv = W * per_warp;
    const bool is_surv = ((lane + 1) & ((1 << kl) - 1)) == 0;
    const int j = warp * per_warp + (lane >> kl);
    if (msurv <= 32) {
      if (is_surv) { surv[j] = A; surv[P + j] = B; surv[2 * P + j] = C; surv[3 * P + j] = D; }
    } else if (is_surv) {
      // kl == kr: the survivors are the m-system; shared-memory inner on the CTA
      if constexpr (INNER == kPCR) {
        inner[j] = A; inner[msurv + j] = B; inner[2 * msurv + j] = C; inner[3 * msurv + j] = D;
      } else {
        rd_setup(A, B, C, D, j, msurv, inner + j, msurv);
      }
    }
#if TDG_SURV_NAMED_BARRIER
    // producer / consumer hand-off on named barrier 1: warps 0 .. W-2 arrive
    // (no wait) once their survivors are stored, the last warp -- under the
    // oldest-first warp scheduling the last to get there anyway -- waits for
    // all of them and solves; everyone meets at the barrier that publishes x
    const int solver = W - 1;
    if (msurv <= 32) {
      if (warp != solver)
        asm volatile("bar.arrive 1, %0;" ::"r"(W * 32) : "memory");
      else
        asm volatile("bar.sync 1, %0;" ::"r"(W * 32) : "memory");
    } else {
      __syncthreads();
    }
#else
    const int solver = 0;
    __syncthreads();
#endif
    if (msurv <= 32) {
      if (warp == solver) {
        const bool v = lane < msurv;
        const T sA = v ? surv[lane] : T(0), sB = v ? surv[P + lane] : T(1);
        const T sC = v ? surv[2 * P + lane] : T(0), sD = v ? surv[3 * P + lane] : T(0);
        const T X = lane_level_solve<T, INNER>(sA, sB, sC, sD, kr - kl, lane & (msurv - 1), msurv);
        if (v) xs[lane] = X;
      }
    } else {
      if constexpr (INNER == kPCR) smem_pcr<T>(inner, xs, msurv, ls, P, SyncCta());
      else smem_rd<T>(inner, xs, msurv, ls, P, SyncCta());
    }
    __syncthreads();
    stp.mark(4);
    // lane-level backward inside the warp
    const T xprev_warp = warp > 0 ? xs[warp * per_warp - 1] : T(0);
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
    xprev = lane > 0 ? xup : xprev_warp;
  return xprev;
}

// RD on the register-blocked m-system of a whole CTA (P = 32 W lanes, Q =
// R >> K survivors per lane): in-lane sequential scan, Hillis-Steele over the
// 32 lane aggregates of each warp (shuffles), one more over the W warp
// aggregates (shared memory, warp 0), fix-up composes, evaluation (R25).
// Returns x of the previous lane's tail for the in-lane back-substitution;
// d[t_u] <- x of the survivors.
template <typename T, int R, int W, int K>
__device__ __forceinline__ T cta_blocked_rd(T (&a)[R], T (&b)[R], T (&c)[R], T (&d)[R], T* sm) {
  constexpr int Q = R >> K;
  constexpr int P = 32 * W;
  const int ls = threadIdx.x;
  const int lane = ls & 31;
  const int warp = ls >> 5;
  const int m = P * Q;
  T* wagg = sm;              // [W][6] warp aggregates -> exclusive warp prefixes
  T* tail = sm + 6 * W;      // [W][2] C[0][0], C[0][2] of every warp's last element
  T* misc = tail + 2 * W;    // [0..1] last element's C (x0), [2 + w] last x of warp w
  T M[Q][6];
#pragma unroll
  for (int u = 0; u < Q; ++u) {
    const int t = Blocked<T, R, K>::t(u);
    const int g = ls * Q + u;
    rd_setup6(a[t], b[t], c[t], d[t], g == 0, g == m - 1, M[u]);
  }
  auto op = [](T (&p)[6], const T (&q)[6]) { mat_compose(p, q); };
#pragma unroll
  for (int u = 1; u < Q; ++u) op(M[u], M[u - 1]);
  T agg[6];
#pragma unroll
  for (int e = 0; e < 6; ++e) agg[e] = M[Q - 1][e];
#pragma unroll
  for (int s = 1; s < 32; s <<= 1) {
    T F[6];
#pragma unroll
    for (int e = 0; e < 6; ++e) F[e] = shup(agg[e], s, 32);
    if (lane >= s) op(agg, F);
  }
  T lex[6];  // exclusive prefix within the warp
#pragma unroll
  for (int e = 0; e < 6; ++e) lex[e] = shup(agg[e], 1, 32);
  if (lane == 31) {
#pragma unroll
    for (int e = 0; e < 6; ++e) wagg[warp * 6 + e] = agg[e];
  }
  __syncthreads();
  if (warp == 0) {
    T wv[6];
#pragma unroll
    for (int e = 0; e < 6; ++e) wv[e] = lane < W ? wagg[lane * 6 + e] : T(0);
#pragma unroll
    for (int s = 1; s < 32; s <<= 1) {
      if (s < W) {
        T F[6];
#pragma unroll
        for (int e = 0; e < 6; ++e) F[e] = shup(wv[e], s, 32);
        if (lane >= s) op(wv, F);
      }
    }
    T wx[6];
#pragma unroll
    for (int e = 0; e < 6; ++e) wx[e] = shup(wv[e], 1, 32);
    __syncwarp();
    if (lane < W) {
#pragma unroll
      for (int e = 0; e < 6; ++e) wagg[lane * 6 + e] = wx[e];
    }
  }
  __syncthreads();
  // prefix of everything before this lane = (earlier lanes of the warp) o (earlier warps)
  if (ls > 0) {
    T ex[6];
    if (warp > 0) {
      T wx[6];
#pragma unroll
      for (int e = 0; e < 6; ++e) wx[e] = wagg[warp * 6 + e];
      if (lane > 0) {
#pragma unroll
        for (int e = 0; e < 6; ++e) ex[e] = lex[e];
        op(ex, wx);
      } else {
#pragma unroll
        for (int e = 0; e < 6; ++e) ex[e] = wx[e];
      }
    } else {
#pragma unroll
      for (int e = 0; e < 6; ++e) ex[e] = lex[e];
    }
#pragma unroll
    for (int u = 0; u < Q; ++u) op(M[u], ex);
  }
  // evaluation: x_0 from the last element, x_g from C_{g-1}
  if (ls == P - 1) { misc[0] = M[Q - 1][0]; misc[1] = M[Q - 1][2]; }
  if (lane == 31) { tail[warp * 2] = M[Q - 1][0]; tail[warp * 2 + 1] = M[Q - 1][2]; }
  __syncthreads();
  const T x0 = rd_x0(misc[0], misc[1]);
  T p00 = shup(M[Q - 1][0], 1, 32), p02 = shup(M[Q - 1][2], 1, 32);
  if (lane == 0 && warp > 0) { p00 = tail[(warp - 1) * 2]; p02 = tail[(warp - 1) * 2 + 1]; }
#pragma unroll
  for (int u = Q - 1; u >= 0; --u) {
    const int t = Blocked<T, R, K>::t(u);
    if (u > 0) d[t] = rd_eval(M[u - 1][0], M[u - 1][2], x0);
    else d[t] = (ls == 0) ? x0 : rd_eval(p00, p02, x0);
  }
  // x of the previous lane's tail (its last survivor) for the back-substitution
  if (lane == 31) misc[2 + warp] = d[R - 1];
  __syncthreads();
  T xprev = shup(d[R - 1], 1, 32);
  if (lane == 0) xprev = warp > 0 ? misc[2 + warp - 1] : T(0);
  return xprev;
}

// KB = -1: register path (k >= log2 R).  KB = -2: shared-memory inner for
// k < log2 R (runtime k; PCR).  KB >= 0: k = KB < log2 R with the register-
// blocked inner across the CTA (RD: cta_blocked_rd).
template <typename T, int R, int W, int INNER, int KB>
__global__ void __launch_bounds__(W * 32)
tdg_cta_kernel(const T* __restrict__ a, const T* __restrict__ b, const T* __restrict__ c,
               const T* d, T* x, int n, long long S, int k, int vec, int pf, int n_real,
               T c_pad, long long es, long long ss) {
  pdl_entry();
  constexpr int P = 32 * W;
  constexpr int LR = ilog2c(R);
  constexpr int LRH = LR > 0 ? LR : 1;
  extern __shared__ __align__(1024) unsigned char smem_raw[];
  T* smem = reinterpret_cast<T*>(smem_raw);
  T* heads = smem;                        // W * LRH * 4
  T* work = smem + W * LRH * 4;
  const int ls = threadIdx.x;
  const int lane = ls & 31;
  const int warp = ls >> 5;
  constexpr bool SMEM = KB != -1;
  const int kin = KB >= 0 ? KB : SMEM ? (k < LR ? k : LR) : LR;

  for (long long sys = blockIdx.x; sys < S; sys += gridDim.x) {
    if (pf && lane < 4 && sys + gridDim.x < S) {
      // lanes 0..3 of every warp prefetch this warp's slice of the next system
      const T* base = lane == 0 ? a : lane == 1 ? b : lane == 2 ? c : d;
      prefetch_l2(base + (size_t)(sys + gridDim.x) * n + (size_t)warp * 32 * R,
                  (uint32_t)(32 * R * sizeof(T)));
    }
    const bool ragged = n_real != n || es != 1 || !vec;
    // contiguous rows (any length / alignment / pitch): CTA-cooperative
    // coalesced loads through a padded shared tile; element-strided rows
    // (interleaved layouts with n > 32R) fall back to scalar loads.
    const bool staged = ragged && es == 1;
    const size_t sbase = (size_t)sys * (size_t)ss;
    const size_t off = sbase + (size_t)ls * R;
    T ra[R], rb[R], rc[R], rd[R];
    if (!ragged) {
      load_block<T, R, true>(a + off, ra, vec);
      load_block<T, R, true>(b + off, rb, vec);
      load_block<T, R, true>(c + off, rc, vec);
      load_block<T, R, false>(d + off, rd, vec);
    } else if (staged) {
      const int TE = n + (n >> 5) + 1;
      T* tA = work;
      T* tB = work + TE;
      T* tC = work + 2 * TE;
      T* tD = work + 3 * TE;
      T va[R], vb[R], vc[R], vd[R];
#pragma unroll
      for (int j = 0; j < R; ++j) {  // element ls + P j: all 4R loads in flight
        const int i = ls + P * j;
        const bool v = i < n_real;
        va[j] = v ? a[sbase + i] : T(0);
        vb[j] = v ? b[sbase + i] : T(1);
        vc[j] = v ? (i == n_real - 1 ? c_pad : c[sbase + i]) : c_pad;
        vd[j] = v ? d[sbase + i] : T(0);
      }
#pragma unroll
      for (int j = 0; j < R; ++j) {
        const int o = wt_off(ls + P * j);
        tA[o] = va[j]; tB[o] = vb[j]; tC[o] = vc[j]; tD[o] = vd[j];
      }
      __syncthreads();
#pragma unroll
      for (int t = 0; t < R; ++t) {
        const int o = wt_off(ls * R + t);
        ra[t] = tA[o]; rb[t] = tB[o]; rc[t] = tC[o]; rd[t] = tD[o];
      }
      __syncthreads();  // the tile is reused by the heads / survivor regions
    } else {
      load_ragged<T, R>(a + sbase, es, ls * R, n_real, ra, T(0), T(0), false);
      load_ragged<T, R>(b + sbase, es, ls * R, n_real, rb, T(1), T(0), false);
      load_ragged<T, R>(c + sbase, es, ls * R, n_real, rc, c_pad, c_pad, true);
      load_ragged<T, R>(d + sbase, es, ls * R, n_real, rd, T(0), T(0), false);
    }
    if (ls == 0) ra[0] = T(0);
    if (ls == P - 1) rc[R - 1] = T(0);

    cta_inlane_forward<T, R, W>(ra, rb, rc, rd, kin, heads, [] {});
    T xprev;
    if constexpr (!SMEM) {
      xprev = cta_register_path<T, R, W, INNER>(ra, rb, rc, rd, k, heads);
    } else if constexpr (KB >= 0 && INNER == kRD) {
      xprev = cta_blocked_rd<T, R, W, (KB >= 0 ? KB : 0)>(ra, rb, rc, rd, work);
    } else {
      // ---- m = P * q > P: shared-memory inner on the whole CTA ----
      const int q = R >> k;
      const int m = P * q;
      const int mask = (1 << k) - 1;
      T* inner = work;
      T* X = inner + (INNER == kPCR ? 8 * m : 12 * m);
#pragma unroll
      for (int t = 0; t < R; ++t) {
        if (((t + 1) & mask) == 0) {
          const int j = ls * q + ((t + 1) >> k) - 1;
          if constexpr (INNER == kPCR) {
            inner[j] = ra[t]; inner[m + j] = rb[t]; inner[2 * m + j] = rc[t]; inner[3 * m + j] = rd[t];
          } else {
            rd_setup(ra[t], rb[t], rc[t], rd[t], j, m, inner + j, m);
          }
        }
      }
      __syncthreads();
      if constexpr (INNER == kPCR) smem_pcr<T>(inner, X, m, ls, P, SyncCta());
      else smem_rd<T>(inner, X, m, ls, P, SyncCta());
#pragma unroll
      for (int t = 0; t < R; ++t) {
        if (((t + 1) & mask) == 0) rd[t] = X[ls * q + ((t + 1) >> k) - 1];
      }
      xprev = ls > 0 ? X[ls * q - 1] : T(0);
    }
    inlane_backward<T, R>(ra, rb, rc, rd, kin, xprev);
    if (!ragged) {
      store_block<T, R>(x + off, rd, vec);
    } else if (staged) {
      __syncthreads();  // every thread is done with the survivor regions
      T* tD = work + 3 * (n + (n >> 5) + 1);
#pragma unroll
      for (int t = 0; t < R; ++t) tD[wt_off(ls * R + t)] = rd[t];
      __syncthreads();
#pragma unroll
      for (int j = 0; j < R; ++j) {
        const int i = ls + P * j;
        if (i < n_real) x[sbase + i] = tD[wt_off(i)];
      }
    } else {
      store_ragged<T, R>(x + sbase, es, ls * R, n_real, rd);
    }
    __syncthreads();  // shared memory is reused by the next system
  }
}

template <typename T>
inline size_t cta_smem_bytes_core(int R, int W, int inner, int k) {
  const int P = 32 * W;
  const int LR = ilog2c(R);
  const int LRH = LR > 0 ? LR : 1;
  int64_t e = (int64_t)W * LRH * 4;
  if (k > LR || (k == LR && inner != kRD)) {
    const int kr = k - LR;
    const int kl = kr < 5 ? kr : 5;
    const int64_t msurv = (int64_t)W * (32 >> kl);
    e += (int64_t)W * 5 * 4 + 4LL * P + P;
    if (msurv > 32) e += inner_region_elems(inner, msurv);
  } else {
    const int64_t m = (int64_t)P * (R >> k);
    // RD: cta_blocked_rd's warp aggregates, tails and broadcasts only
    e += inner == kRD ? 9LL * W + 2 : inner_region_elems(inner, m);
  }
  return (size_t)e * sizeof(T);
}

// Shared-memory bytes of tdg_cta_kernel for a given k (staged: room for the
// coalesced staging tile of the general path, 4 (n + n/32 + 1) elements).
template <typename T>
inline size_t cta_smem_bytes(int R, int W, int inner, int k, bool staged = false) {
  const size_t base = cta_smem_bytes_core<T>(R, W, inner, k);
  const int64_t n = 32LL * W * R;
  const size_t tile = (size_t)(W * (ilog2c(R) > 0 ? ilog2c(R) : 1) * 4 + 4 * (n + (n >> 5) + 1)) * sizeof(T);
  return staged && tile > base ? tile : base;
}

}  // namespace tdg
