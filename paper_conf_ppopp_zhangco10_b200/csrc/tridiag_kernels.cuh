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

namespace tdg {

// ============================================================================
// Warp kernel.
// ============================================================================
// KB < 0: k >= LR (all in-lane levels; m <= P, lane-level inner solve).
// KB >= 0: k == KB < LR (m = P * (R >> KB) > P, register-blocked inner solve).
template <typename T, int R, int INNER, int KB>
__device__ __forceinline__ void warp_solve(T (&a)[R], T (&b)[R], T (&c)[R], T (&d)[R], int k,
                                           int ls, int P) {
  constexpr int LR = ilog2c(R);
  constexpr int kin = KB < 0 ? LR : KB;
  inlane_forward_interior<T, R>(a, b, c, d, kin);
  Heads<T, R> H;
  heads_from_next_lane<T, R>(a, b, c, d, kin, P, ls == P - 1, H);
  inlane_tail_chain<T, R>(a, b, c, d, kin, H);
  if constexpr (KB < 0) {
    d[R - 1] = lane_level_solve<T, INNER>(a[R - 1], b[R - 1], c[R - 1], d[R - 1], k - LR, ls, P);
  } else {
    // m = P * (R >> KB) > P: the intermediate system stays block-distributed
    // in registers (no copy; the paper copies it to 5 extra arrays).
    if constexpr (INNER == kPCR) blocked_pcr<T, R, (KB < 0 ? 0 : KB)>(a, b, c, d, ls, P);
    else blocked_rd<T, R, (KB < 0 ? 0 : KB)>(a, b, c, d, ls, P);
  }
  T xprev = __shfl_up_sync(kFull, d[R - 1], 1, P);
  if (ls == 0) xprev = T(0);
  inlane_backward<T, R>(a, b, c, d, kin, xprev);
}

template <typename T, int R, int INNER, int KB>
__global__ void __launch_bounds__(256)
tdg_warp_kernel(const T* __restrict__ a, const T* __restrict__ b, const T* __restrict__ c,
                const T* d, T* x, int n, long long S, int k, int log2P, int vec, int pf) {
  const int P = 1 << log2P;
  const int lane = threadIdx.x & 31;
  const int warp = threadIdx.x >> 5;
  const int wpb = blockDim.x >> 5;
  const int G = 32 >> log2P;  // systems per warp
  const int sub = lane >> log2P;
  const int ls = lane & (P - 1);
  const long long step = (long long)gridDim.x * wpb * G;
  for (long long s0 = ((long long)blockIdx.x * wpb + warp) * G; s0 < S; s0 += step) {
    if (pf && lane < 4 && s0 + step < S) {
      // lanes 0..3 prefetch array a, b, c, d of this warp's next group
      const long long nx = s0 + step;
      const long long cnt = (S - nx) < G ? (S - nx) : G;
      const T* base = lane == 0 ? a : lane == 1 ? b : lane == 2 ? c : d;
      prefetch_l2(base + (size_t)nx * n, (uint32_t)(cnt * n * sizeof(T)));
    }
    const long long sys = s0 + sub;
    const bool valid = sys < S;
    const size_t off = (size_t)sys * (size_t)n + (size_t)ls * R;
    T ra[R], rb[R], rc[R], rd[R];
    if (valid) {
      load_block<T, R, true>(a + off, ra, vec);
      load_block<T, R, true>(b + off, rb, vec);
      load_block<T, R, true>(c + off, rc, vec);
      load_block<T, R, false>(d + off, rd, vec);
    } else {
#pragma unroll
      for (int i = 0; i < R; ++i) { ra[i] = T(0); rb[i] = T(1); rc[i] = T(0); rd[i] = T(0); }
    }
    // a_0 and c_{n-1} are not matrix entries: never read.
    if (ls == 0) ra[0] = T(0);
    if (ls == P - 1) rc[R - 1] = T(0);
    warp_solve<T, R, INNER, KB>(ra, rb, rc, rd, k, ls, P);
    if (valid) store_block<T, R>(x + off, rd, vec);
  }
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
template <typename T, int R, int W, int INNER, bool SMEM>
__global__ void __launch_bounds__(W * 32)
tdg_cta_kernel(const T* __restrict__ a, const T* __restrict__ b, const T* __restrict__ c,
               const T* d, T* x, int n, long long S, int k, int vec, int pf) {
  constexpr int P = 32 * W;
  constexpr int LR = ilog2c(R);
  constexpr int LRH = LR > 0 ? LR : 1;
  extern __shared__ __align__(16) unsigned char smem_raw[];
  T* smem = reinterpret_cast<T*>(smem_raw);
  T* heads = smem;                        // W * LRH * 4
  T* work = smem + W * LRH * 4;
  const int ls = threadIdx.x;
  const int lane = ls & 31;
  const int warp = ls >> 5;
  const int kin = SMEM ? (k < LR ? k : LR) : LR;

  for (long long sys = blockIdx.x; sys < S; sys += gridDim.x) {
    if (pf && lane < 4 && sys + gridDim.x < S) {
      // lanes 0..3 of every warp prefetch this warp's slice of the next system
      const T* base = lane == 0 ? a : lane == 1 ? b : lane == 2 ? c : d;
      prefetch_l2(base + (size_t)(sys + gridDim.x) * n + (size_t)warp * 32 * R,
                  (uint32_t)(32 * R * sizeof(T)));
    }
    const size_t off = (size_t)sys * (size_t)n + (size_t)ls * R;
    T ra[R], rb[R], rc[R], rd[R];
    load_block<T, R, true>(a + off, ra, vec);
    load_block<T, R, true>(b + off, rb, vec);
    load_block<T, R, true>(c + off, rc, vec);
    load_block<T, R, false>(d + off, rd, vec);
    if (ls == 0) ra[0] = T(0);
    if (ls == P - 1) rc[R - 1] = T(0);

    inlane_forward_interior<T, R>(ra, rb, rc, rd, kin);
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

    T xprev;
    if constexpr (!SMEM) {
      // ---- P survivors (one per lane) -> compacted CR levels in smem ----
      const int kr = k - LR;                 // CR levels left
      const int m = P >> kr;                 // intermediate size
      const int mt = m > 32 ? m : 32;        // reduce in smem down to mt
      const int kmid = ilog2c(P) - ilog2c(mt);
      T* LA = work;
      T* LB = LA + 2 * P;
      T* LC = LB + 2 * P;
      T* LD = LC + 2 * P;
      T* LX = LD + 2 * P;
      T* inner = LX + 2 * P;
      LA[ls] = ra[R - 1]; LB[ls] = rb[R - 1]; LC[ls] = rc[R - 1]; LD[ls] = rd[R - 1];
      __syncthreads();
      int offp = 0;  // offset of level l-1
      for (int l = 1; l <= kmid; ++l) {
        const int np = P >> (l - 1);  // equations at level l-1
        const int offn = offp + np;   // offset of level l
        const int j = ls;
        if (j < (np >> 1)) {
          const int i = offp + 2 * j + 1, lo = i - 1, hi = i + 1;
          T ai = LA[i], bi = LB[i], ci = LC[i], di = LD[i];
          const T rl = Arith<T>::rcp(LB[lo]);
          T ha = T(0), hr = T(0), hc = T(0), hd = T(0);
          if (2 * j + 2 < np) { ha = LA[hi]; hr = Arith<T>::rcp(LB[hi]); hc = LC[hi]; hd = LD[hi]; }
          cr_unit(ai, bi, ci, di, LA[lo], rl, LC[lo], LD[lo], ha, hr, hc, hd);
          LA[offn + j] = ai; LB[offn + j] = bi; LC[offn + j] = ci; LD[offn + j] = di;
        }
        __syncthreads();
        offp = offn;
      }
      // level kmid (mt equations) at offset offp
      if (m <= 32) {
        if (warp == 0) {
          const T X = lane_level_solve<T, INNER>(LA[offp + lane], LB[offp + lane],
                                                 LC[offp + lane], LD[offp + lane],
                                                 ilog2c(32) - ilog2c(m), lane, 32);
          LX[offp + lane] = X;
        }
      } else {
        if constexpr (INNER == kPCR) {
          for (int j = ls; j < m; j += P) {
            inner[j] = LA[offp + j]; inner[m + j] = LB[offp + j];
            inner[2 * m + j] = LC[offp + j]; inner[3 * m + j] = LD[offp + j];
          }
        } else {
          for (int j = ls; j < m; j += P)
            rd_setup(LA[offp + j], LB[offp + j], LC[offp + j], LD[offp + j], j, m, inner + j, m);
        }
        __syncthreads();
        T* X = inner + (INNER == kPCR ? 8 * m : 12 * m);
        if constexpr (INNER == kPCR) smem_pcr<T>(inner, X, m, ls, P, SyncCta());
        else smem_rd<T>(inner, X, m, ls, P, SyncCta());
        for (int j = ls; j < m; j += P) LX[offp + j] = X[j];
      }
      __syncthreads();
      // backward through the compacted levels: level l-1 from level l
      for (int l = kmid; l >= 1; --l) {
        const int np = P >> (l - 1);
        const int offl = 2 * P - 2 * (P >> l);       // level l
        const int offm = 2 * P - 2 * np;             // level l-1
        const int j = ls;
        if (j < (np >> 1)) {
          const T xo = LX[offl + j];                  // x of equation 2j+1 of level l-1
          const T xl = (j > 0) ? LX[offl + j - 1] : T(0);
          const int e = offm + 2 * j;
          LX[e] = Arith<T>::div(LD[e] - LA[e] * xl - LC[e] * xo, LB[e]);
          LX[e + 1] = xo;
        }
        __syncthreads();
      }
      rd[R - 1] = LX[ls];
      xprev = ls > 0 ? LX[ls - 1] : T(0);
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
    store_block<T, R>(x + off, rd, vec);
    __syncthreads();  // shared memory is reused by the next system
  }
}

// Shared-memory bytes of tdg_cta_kernel for a given k.
template <typename T>
inline size_t cta_smem_bytes(int R, int W, int inner, int k) {
  const int P = 32 * W;
  const int LR = ilog2c(R);
  const int LRH = LR > 0 ? LR : 1;
  int64_t e = (int64_t)W * LRH * 4;
  if (k >= LR) {
    const int m = P >> (k - LR);
    e += 10LL * P;
    if (m > 32) e += inner_region_elems(inner, m);
  } else {
    const int64_t m = (int64_t)P * (R >> k);
    e += inner_region_elems(inner, m);
  }
  return (size_t)e * sizeof(T);
}

}  // namespace tdg
