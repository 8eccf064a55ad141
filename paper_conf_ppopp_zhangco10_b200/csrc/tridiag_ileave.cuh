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
                  const T* d, T* x, int n, long long S, int k, int log2P, int G, int n_real,
                  T c_pad, long long es) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  T* tile = reinterpret_cast<T*>(smem_raw);
  const int TE = ilv_tile_elems(n, G);
  T* tA = tile;
  T* tB = tile + TE;
  T* tC = tile + 2 * TE;
  T* tD = tile + 3 * TE;
  const int P = 1 << log2P;
  const int NT = blockDim.x;  // = G * P
  const int g = threadIdx.x >> log2P;
  const int ls = threadIdx.x & (P - 1);
  const int rows = n * G;
  for (long long t0 = (long long)blockIdx.x * G; t0 < S; t0 += (long long)gridDim.x * G) {
    // ---- coalesced load of the tile (rows of G consecutive systems) ----
    for (int idx = threadIdx.x; idx < rows; idx += NT) {
      const int r = idx / G, gg = idx - r * G;
      const long long s = t0 + gg;
      const int o = ilv_off(r, gg, G);
      if (s < S && r < n_real) {
        const long long e = s + (long long)r * es;
        tA[o] = a[e]; tB[o] = b[e];
        tC[o] = (r == n_real - 1) ? c_pad : c[e];
        tD[o] = d[e];
      } else {
        tA[o] = T(0); tB[o] = T(1); tC[o] = c_pad; tD[o] = T(0);
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
    for (int idx = threadIdx.x; idx < rows; idx += NT) {
      const int r = idx / G, gg = idx - r * G;
      const long long s = t0 + gg;
      if (s < S && r < n_real) x[s + (long long)r * es] = tD[ilv_off(r, gg, G)];
    }
    __syncthreads();
  }
}

}  // namespace tdg
