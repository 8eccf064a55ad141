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
__global__ void __launch_bounds__(256)
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
  const long long step = (long long)RS * es;
  for (long long t0 = (long long)blockIdx.x * G; t0 < S; t0 += (long long)gridDim.x * G) {
    const long long s0 = t0 + q * V;           // first system of this thread's group
    // ---- coalesced load of the tile ----
    {
      long long e = s0 + (long long)r0 * es;
      for (int r = r0; r < n; r += RS, e += step) {
        const int o = ilv_off(r, q * V, G);
        if (r < n_real && s0 + V <= S) {
          T va[V16], vb[V16], vc[V16], vd[V16];
          if (vec16) {
            if constexpr (sizeof(T) == 4) {
              const float4 A4 = __ldg(reinterpret_cast<const float4*>(a + e));
              const float4 B4 = __ldg(reinterpret_cast<const float4*>(b + e));
              const float4 C4 = __ldg(reinterpret_cast<const float4*>(c + e));
              const float4 D4 = *reinterpret_cast<const float4*>(d + e);
              va[0] = A4.x; va[1] = A4.y; va[2] = A4.z; va[3] = A4.w;
              vb[0] = B4.x; vb[1] = B4.y; vb[2] = B4.z; vb[3] = B4.w;
              vc[0] = C4.x; vc[1] = C4.y; vc[2] = C4.z; vc[3] = C4.w;
              vd[0] = D4.x; vd[1] = D4.y; vd[2] = D4.z; vd[3] = D4.w;
            } else {
              const double2 A2 = __ldg(reinterpret_cast<const double2*>(a + e));
              const double2 B2 = __ldg(reinterpret_cast<const double2*>(b + e));
              const double2 C2 = __ldg(reinterpret_cast<const double2*>(c + e));
              const double2 D2 = *reinterpret_cast<const double2*>(d + e);
              va[0] = A2.x; va[1] = A2.y; vb[0] = B2.x; vb[1] = B2.y;
              vc[0] = C2.x; vc[1] = C2.y; vd[0] = D2.x; vd[1] = D2.y;
            }
#pragma unroll
            for (int j = 0; j < V16; ++j) {
              tA[o + j] = va[j]; tB[o + j] = vb[j];
              tC[o + j] = (r == n_real - 1) ? c_pad : vc[j];
              tD[o + j] = vd[j];
            }
          } else {
            tA[o] = a[e]; tB[o] = b[e]; tC[o] = (r == n_real - 1) ? c_pad : c[e]; tD[o] = d[e];
          }
        } else {
          for (int j = 0; j < V; ++j) {
            const bool ok = r < n_real && s0 + j < S;
            tA[o + j] = ok ? a[e + j] : T(0);
            tB[o + j] = ok ? b[e + j] : T(1);
            tC[o + j] = ok ? ((r == n_real - 1) ? c_pad : c[e + j]) : c_pad;
            tD[o + j] = ok ? d[e + j] : T(0);
          }
        }
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
    {
      long long e = s0 + (long long)r0 * es;
      for (int r = r0; r < n_real; r += RS, e += step) {
        const int o = ilv_off(r, q * V, G);
        if (vec16 && s0 + V <= S) {
          if constexpr (sizeof(T) == 4)
            *reinterpret_cast<float4*>(x + e) = make_float4(tD[o], tD[o + 1], tD[o + 2], tD[o + 3]);
          else
            *reinterpret_cast<double2*>(x + e) = make_double2(tD[o], tD[o + 1]);
        } else {
          for (int j = 0; j < V; ++j)
            if (s0 + j < S) x[e + j] = tD[o + j];
        }
      }
    }
    __syncthreads();
  }
}

}  // namespace tdg
