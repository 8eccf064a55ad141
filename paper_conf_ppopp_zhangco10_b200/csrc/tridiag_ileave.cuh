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

template <typename T, int R, int INNER, int KB>
__global__ void __launch_bounds__(256, 2)
tdg_ileave_kernel(const T* __restrict__ a, const T* __restrict__ b, const T* __restrict__ c,
                  const T* d, T* x, int n, long long S, int k, int log2P, int log2G, int n_real,
                  T c_pad, long long es, int vec16) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  T* tile = reinterpret_cast<T*>(smem_raw);
  const int G = 1 << log2G;
  const int TE = ilv_tile_elems(n, G);
  T* tA = tile;
  T* tB = tile + TE;
  T* tC = tile + 2 * TE;
  T* tD = tile + 3 * TE;
  const int P = 1 << log2P;
  const int NT = blockDim.x;  // = G * P
  const int g = threadIdx.x >> log2P;
  const int ls = threadIdx.x & (P - 1);
  // Row-segment mapping for the coalesced phases: V consecutive systems per
  // thread (one 16-byte vector when aligned, else V = 1).
  constexpr int V16 = 16 / (int)sizeof(T);
  const int V = vec16 ? V16 : 1;
  const int lv = vec16 ? (V16 == 4 ? 2 : 1) : 0;
  const int qpr = G >> lv;                     // threads per row segment
  const int lq = log2G - lv;
  const int q = threadIdx.x & (qpr - 1);       // which V-group of the row
  const int r0 = threadIdx.x >> lq;            // first row of this thread
  const int RS = NT >> lq;                     // rows per sweep
  for (long long t0 = (long long)blockIdx.x * G; t0 < S; t0 += (long long)gridDim.x * G) {
    const long long s0 = t0 + q * V;           // first system of this thread's group
    // ---- coalesced load of the tile ----
    // Each thread moves R / V row segments (compile-time count: n G / NT =
    // R rows of V systems, unrolled so all loads are in flight together).
    if (vec16) {
      constexpr int NSEG = R / V16 > 0 ? R / V16 : 1;
      T va[NSEG][V16], vb[NSEG][V16], vc[NSEG][V16], vd[NSEG][V16];
#pragma unroll
      for (int j = 0; j < NSEG; ++j) {
        const int r = r0 + j * RS;
        const long long e = s0 + (long long)r * es;
        const bool full = r < n_real && s0 + V16 <= S;
        if (full) {
          if constexpr (sizeof(T) == 4) {
            const float4 A4 = __ldg(reinterpret_cast<const float4*>(a + e));
            const float4 B4 = __ldg(reinterpret_cast<const float4*>(b + e));
            const float4 C4 = __ldg(reinterpret_cast<const float4*>(c + e));
            const float4 D4 = *reinterpret_cast<const float4*>(d + e);
            va[j][0] = A4.x; va[j][1] = A4.y; va[j][2] = A4.z; va[j][3] = A4.w;
            vb[j][0] = B4.x; vb[j][1] = B4.y; vb[j][2] = B4.z; vb[j][3] = B4.w;
            vc[j][0] = C4.x; vc[j][1] = C4.y; vc[j][2] = C4.z; vc[j][3] = C4.w;
            vd[j][0] = D4.x; vd[j][1] = D4.y; vd[j][2] = D4.z; vd[j][3] = D4.w;
          } else {
            const double2 A2 = __ldg(reinterpret_cast<const double2*>(a + e));
            const double2 B2 = __ldg(reinterpret_cast<const double2*>(b + e));
            const double2 C2 = __ldg(reinterpret_cast<const double2*>(c + e));
            const double2 D2 = *reinterpret_cast<const double2*>(d + e);
            va[j][0] = A2.x; va[j][1] = A2.y; vb[j][0] = B2.x; vb[j][1] = B2.y;
            vc[j][0] = C2.x; vc[j][1] = C2.y; vd[j][0] = D2.x; vd[j][1] = D2.y;
          }
        } else {
#pragma unroll
          for (int v = 0; v < V16; ++v) {
            const bool ok = r < n_real && s0 + v < S;
            va[j][v] = ok ? a[e + v] : T(0);
            vb[j][v] = ok ? b[e + v] : T(1);
            vc[j][v] = ok ? c[e + v] : c_pad;
            vd[j][v] = ok ? d[e + v] : T(0);
          }
        }
      }
#pragma unroll
      for (int j = 0; j < NSEG; ++j) {
        const int r = r0 + j * RS;
        const int o = ilv_off(r, q * V16, G);
#pragma unroll
        for (int v = 0; v < V16; ++v) {
          tA[o + v] = va[j][v]; tB[o + v] = vb[j][v];
          tC[o + v] = (r == n_real - 1) ? c_pad : vc[j][v];
          tD[o + v] = vd[j][v];
        }
      }
    } else {
      T va[R], vb[R], vc[R], vd[R];
#pragma unroll
      for (int j = 0; j < R; ++j) {
        const int r = r0 + j * RS;
        const long long e = s0 + (long long)r * es;
        const bool ok = r < n_real && s0 < S;
        va[j] = ok ? a[e] : T(0);
        vb[j] = ok ? b[e] : T(1);
        vc[j] = ok ? (r == n_real - 1 ? c_pad : c[e]) : c_pad;
        vd[j] = ok ? d[e] : T(0);
      }
#pragma unroll
      for (int j = 0; j < R; ++j) {
        const int o = ilv_off(r0 + j * RS, q, G);
        tA[o] = va[j]; tB[o] = vb[j]; tC[o] = vc[j]; tD[o] = vd[j];
      }
    }
    __syncthreads();
    T ra[R], rb[R], rc[R], rd[R];
#pragma unroll
    for (int t = 0; t < R; ++t) {
      const int o = ilv_off(ls * R + t, g, G);
      ra[t] = tA[o]; rb[t] = tB[o]; rc[t] = tC[o]; rd[t] = tD[o];
    }
    if (ls == 0) ra[0] = T(0);
    if (ls == P - 1) rc[R - 1] = T(0);
    warp_solve<T, R, INNER, KB>(ra, rb, rc, rd, k, ls, P);
#pragma unroll
    for (int t = 0; t < R; ++t) tD[ilv_off(ls * R + t, g, G)] = rd[t];
    __syncthreads();
    if (vec16) {
      constexpr int NSEG = R / V16 > 0 ? R / V16 : 1;
#pragma unroll
      for (int j = 0; j < NSEG; ++j) {
        const int r = r0 + j * RS;
        if (r >= n_real) continue;
        const long long e = s0 + (long long)r * es;
        const int o = ilv_off(r, q * V16, G);
        if (s0 + V16 <= S) {
          if constexpr (sizeof(T) == 4)
            *reinterpret_cast<float4*>(x + e) = make_float4(tD[o], tD[o + 1], tD[o + 2], tD[o + 3]);
          else
            *reinterpret_cast<double2*>(x + e) = make_double2(tD[o], tD[o + 1]);
        } else {
          for (int v = 0; v < V16; ++v)
            if (s0 + v < S) x[e + v] = tD[o + v];
        }
      }
    } else {
#pragma unroll
      for (int j = 0; j < R; ++j) {
        const int r = r0 + j * RS;
        if (r < n_real && s0 < S) x[s0 + (long long)r * es] = tD[ilv_off(r, q, G)];
      }
    }
    __syncthreads();
  }
}

}  // namespace tdg
