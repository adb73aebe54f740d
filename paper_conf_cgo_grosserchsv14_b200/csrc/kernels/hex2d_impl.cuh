// hex2d_impl.cuh -- the specialised sm_100a phase kernel for 2D single-field stencils of
// radius 1 (jacobi2d5, star2d5, box2d9, gradient2d) under the hybrid schedule with
// delta0 = delta1 = 1 (Sec. 3.3-3.6, Fig. 6).
//
// Mapping:
//   * one CTA per hexagon S0 of the launch's (T, p) (Sec. 4.1);
//   * the classical dimension j is streamed in super-chunks of C = NW*32*V columns; the
//     super-chunk k at local level a covers j in [k*C - a, k*C - a + C - 1] -- exactly the
//     classical tile of eq. (14) with w1 = C and u = a -- and the chunks run sequentially
//     inside the CTA, as the paper's S1 loop does;
//   * a thread owns V consecutive columns of the chunk and ALL hexagon rows b of the
//     current level in registers (the time wavefront lives in registers: Fig. 2's
//     "values ... reused in registers across sequential time steps", PAPER.md:135-141,
//     taken to its limit -- no shared-memory copy of the tile at all);
//   * horizontal neighbours come from the left lane by two warp shuffles per row and
//     level; lane 0 takes them from a tiny shared-memory "tail" written by the last lane of
//     the previous warp (or of the previous super-chunk) -- the paper's inter-tile reuse
//     (Sec. 4.2.2) in registers;
//   * HBM is touched only for the hexagon's In set (w0+4h+5 values per column: the bottom
//     row and the slanted-edge inputs) and Out set (w0+4h+3 values per column: the slanted
//     upper edges and the top row), plus every value of the final time level -- the
//     interleaved copy-out of Sec. 4.2.1;
//   * the level loop and the row loop are fully unrolled from the compile-time hexagon
//     shape (constraint-based unrolling, Sec. 4.3.2); full tiles run the
//     branch-free instantiation, tiles cut by the domain run the predicated one
//     (full/partial separation, Sec. 4.3.1).
#pragma once
#include <cstdint>
#include <type_traits>

#include "../stencil_ops.cuh"
#include "launch.h"

namespace hexs {
namespace fast2d {

// Compile-time loop: f(std::integral_constant<int, I>) for I in [A, N).
template <int A, int N, class F>
__device__ __forceinline__ void static_for(F&& f) {
  if constexpr (A < N) {
    f(std::integral_constant<int, A>{});
    static_for<A + 1, N>(f);
  }
}

template <typename T> struct VecInfo;
template <> struct VecInfo<float> { static constexpr int V = 4, VB = 4; };   // 16-B blocks
template <> struct VecInfo<double> { static constexpr int V = 2, VB = 2; };

__host__ __device__ constexpr int lo_row(int H, int W0, int a) { return a <= H ? H - a : a - H - 1; }
__host__ __device__ constexpr int hi_row(int H, int W0, int a) { return a <= H ? H + W0 + a : 3 * H + 1 + W0 - a; }

template <typename T, int KIND>
__device__ __forceinline__ T apply(const T (&x)[3][3], const Coef<T>& k) {
  // x[r][c]: r = row b-1, b, b+1 ; c = column j-1, j, j+1
  if constexpr (KIND == K_JACOBI2D5) return jacobi2d5<T>(x[1][1], x[0][1], x[2][1], x[1][0], x[1][2], k);
  else if constexpr (KIND == K_STAR2D5) return star2d5<T>(x[1][1], x[0][1], x[2][1], x[1][0], x[1][2], k);
  else if constexpr (KIND == K_GRADIENT2D) return gradient2d<T>(x[1][1], x[0][1], x[2][1], x[1][0], x[1][2], k);
  else return box2d9<T>(x[0][0], x[0][1], x[0][2], x[1][0], x[1][1], x[1][2], x[2][0], x[2][1], x[2][2], k);
}

template <typename T, int KIND, int H, int W0, int NW>
struct Kernel {
  static constexpr int V = VecInfo<T>::V;
  static constexpr int VB = VecInfo<T>::VB;
  static constexpr int L = 2 * H + 2;        // levels per hexagon
  static constexpr int R = W0 + 2 * H + 1;   // max hexagon rows; local rows b in [0, R)
  static constexpr int Q = R + 2;            // register rows q = b + 1, b in [-1, R]
  static constexpr int NT = NW * 32;
  static constexpr int C = NT * V;           // super-chunk width (classical tile w1)
  static constexpr int HALO = 2;             // two left-halo columns per row
  static constexpr int MINB = sizeof(T) == 8 ? 2 : 3;  // resident CTAs/SM the register budget targets

  struct Smem {
    T tail[2][L][NW][Q][2];  // [chunk parity][level][warp][row][2 last columns]
  };

  // kind of register row q at level a
  __host__ __device__ static constexpr bool is_in_row(int a, int q) {   // loaded from global at level a
    const int b = q - 1;
    if (a == 0) return b >= lo_row(H, W0, 0) - 1 && b <= hi_row(H, W0, 0) + 1;
    if (a <= H) return b == lo_row(H, W0, a) - 1 || b == lo_row(H, W0, a) ||
                       b == hi_row(H, W0, a) || b == hi_row(H, W0, a) + 1;
    if (a == H + 1) return b == -1 || b == R;
    return false;
  }
  __host__ __device__ static constexpr bool is_input_row(int a, int q) {  // any input row of level a
    const int b = q - 1;
    return b >= lo_row(H, W0, a) - 1 && b <= hi_row(H, W0, a) + 1;
  }
  __host__ __device__ static constexpr bool is_out_row(int a, int q) {  // in the Out set (stored) at level a
    const int b = q - 1, lo = lo_row(H, W0, a), hi = hi_row(H, W0, a);
    if (b < lo || b > hi) return false;
    if (a < H) return false;
    if (a == H) return b == lo || b == hi;
    if (a < L - 1) return b <= lo + 1 || b >= hi - 1;
    return true;
  }
  __host__ __device__ static constexpr bool is_comp_row(int a, int q) {
    const int b = q - 1;
    return b >= lo_row(H, W0, a) && b <= hi_row(H, W0, a);
  }

  // Load V+2 consecutive elements starting at column `start` (= thread's first halo
  // column) of global row `row` into dst[0..V+1].  aligned: row pitch is 16-B granular so
  // aligned 16-B block loads are legal; the misalignment (start mod VB) is the
  // compile-time constant M.
  template <int M, bool PART>
  static __device__ __forceinline__ void load_window(const T* __restrict__ src, int64_t N1, int64_t row,
                                                     int start, bool aligned, T (&dst)[V + 2]) {
    const T* rp = src + row * N1;
    if (aligned && (!PART || (start - M >= 0 && start - M + 3 * VB <= N1))) {
      constexpr int NB = (M + V + 2 + VB - 1) / VB;  // 16-B blocks covering [M, M+V+2)
      T blk[NB * VB];
      const T* bp = rp + (start - M);
#pragma unroll
      for (int i = 0; i < NB; ++i) {
        if constexpr (VB == 4) {
          const float4 v = *(reinterpret_cast<const float4*>(bp) + i);
          blk[4 * i] = v.x; blk[4 * i + 1] = v.y; blk[4 * i + 2] = v.z; blk[4 * i + 3] = v.w;
        } else {
          const double2 v = *(reinterpret_cast<const double2*>(bp) + i);
          blk[2 * i] = v.x; blk[2 * i + 1] = v.y;
        }
      }
#pragma unroll
      for (int i = 0; i < V + 2; ++i) dst[i] = blk[M + i];
    } else {
#pragma unroll
      for (int i = 0; i < V + 2; ++i) {
        int64_t col = (int64_t)start + i;
        if constexpr (PART) col = col < 0 ? 0 : (col >= N1 ? N1 - 1 : col);
        dst[i] = rp[col];
      }
    }
  }

  // One super-chunk: all levels a in [a_lo, a_hi] of columns [k*C - a, k*C - a + C).
  // PART: tile cut by the domain (predicated points); TCUT: tile cut in time (levels
  // outside [a_lo, a_hi] are skipped at run time).  Full tiles run <false, false>, which is
  // free of any run-time level control so every register row has a static live range.
  template <bool PART, bool TCUT>
  static __device__ __forceinline__ void chunk(const Fast2DArgs& g, Smem& sm, int64_t k, int64_t i0,
                                               int a_final, bool aligned, const Coef<T>& cf) {
    const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
    const int64_t N0 = g.N0, N1 = g.N1;
    T in[Q][V + 2];  // input array of the current level: [row][halo0, halo1, own V]
#pragma unroll
    for (int q = 0; q < Q; ++q)
#pragma unroll
      for (int v = 0; v < V + 2; ++v) in[q][v] = T(0);

    static_for<0, L>([&](auto a_c) {
      constexpr int a = decltype(a_c)::value;
      if constexpr (TCUT) {
        if (a < g.a_lo || a > g.a_hi) return;  // time-cut tiles (uniform)
      }
      const int64_t tau = g.tau0 + a;
      const T* src = static_cast<const T*>(g.buf[tau & 1]);
      T* dst = static_cast<T*>(g.buf[(tau + 1) & 1]);
      const int colbase = (int)k * C - a + tid * V;  // first output column (N1 < 2^30)
      const int wstart = colbase - 1;                // first input column (halo)
      constexpr int M = ((-a - 1) % VB + VB) % VB;             // wstart mod VB (k*C, tid*V are multiples of VB)
      const bool first = TCUT ? (a == g.a_lo) : (a == 0);

      // ---- (1) inputs: In rows from global (all input rows at the first level) ----
#pragma unroll
      for (int q = 0; q < Q; ++q) {
        if (!is_input_row(a, q)) continue;
        if (first || is_in_row(a, q)) {
          int64_t row = i0 + (q - 1);
          if constexpr (PART) row = row < 0 ? 0 : (row >= N0 ? N0 - 1 : row);
          load_window<M, PART>(src, N1, row, wstart, aligned, in[q]);
        }
      }
      // ---- (2)-(5) rows ascending: left halo just in time, compute, copy out, tail ----
      const int pw = warp == 0 ? NW - 1 : warp - 1;
      const int pk = warp == 0 ? (int)((k - 1) & 1) : (int)(k & 1);
      // Left halo of input row q: rows computed at the previous level take the two last
      // columns of the left lane (shuffle) or, in lane 0, of the previous warp / chunk
      // (shared-memory tail).  Rows loaded from global already carry their halo.
      auto halo = [&](auto q_c) {
        constexpr int q = decltype(q_c)::value;
        if constexpr (is_input_row(a, q) && !is_in_row(a, q) && a > 0) {
          if (!first) {
            T h0 = __shfl_up_sync(0xffffffffu, in[q][V], 1);
            T h1 = __shfl_up_sync(0xffffffffu, in[q][V + 1], 1);
            if (lane == 0) {
              h0 = sm.tail[pk][a - 1][pw][q][0];
              h1 = sm.tail[pk][a - 1][pw][q][1];
            }
            in[q][0] = h0;
            in[q][1] = h1;
          }
        }
      };
      constexpr int qlo = lo_row(H, W0, a) + 1, qhi = hi_row(H, W0, a) + 1;
      halo(std::integral_constant<int, qlo - 1>{});
      halo(std::integral_constant<int, qlo>{});
      T out[Q][V];
      bool colok[V];
#pragma unroll
      for (int v = 0; v < V; ++v) {
        const int c = colbase + v;
        colok[v] = !PART || (c >= 1 && c <= (int)N1 - 2);
      }
      const bool fin = TCUT && (a == a_final);
      static_for<qlo, qhi + 1>([&](auto q_c) {
        constexpr int q = decltype(q_c)::value;
        halo(std::integral_constant<int, q + 1>{});
        const int64_t row = i0 + (q - 1);
        const bool rowok = !PART || (row >= 1 && row <= N0 - 2);
#pragma unroll
        for (int v = 0; v < V; ++v) {
          T x[3][3];
#pragma unroll
          for (int r = 0; r < 3; ++r)
#pragma unroll
            for (int c = 0; c < 3; ++c) x[r][c] = in[q - 1 + r][v + c];
          const T val = apply<T, KIND>(x, cf);
          if constexpr (PART) out[q][v] = (rowok && colok[v]) ? val : in[q][v + 1];
          else out[q][v] = val;
        }
        // interleaved copy-out of the Out set (every row at the final level)
        if (is_out_row(a, q) || fin) {
          if (!PART || rowok) {
            T* rp = dst + row * N1 + colbase;
#pragma unroll
            for (int v = 0; v < V; ++v)
              if (!PART || colok[v]) rp[v] = out[q][v];
          }
        }
        // tail for the next warp / next super-chunk
        if constexpr (a < L - 1) {
          if (lane == 31) {
            sm.tail[k & 1][a][warp][q][0] = out[q][V - 2];
            sm.tail[k & 1][a][warp][q][1] = out[q][V - 1];
          }
        }
      });
      __syncthreads();
      // ---- (6) the outputs become the next level's inputs ----
#pragma unroll
      for (int q = qlo; q <= qhi; ++q)
#pragma unroll
        for (int v = 0; v < V; ++v) in[q][v + 2] = out[q][v];
    });
  }

  template <bool TCUT>
  static __device__ __forceinline__ void run(const Fast2DArgs& g, Smem& sm) {
    const int64_t S0 = g.S0_lo + blockIdx.x;
    const int64_t i0 = S0 * g.W - g.row_off;  // global row of local row b = 0
    const Coef<T> cf{(T)g.k0, (T)g.k1};
    const int64_t N0 = g.N0, N1 = g.N1;
    const bool aligned = ((N1 * (int64_t)sizeof(T)) % 16) == 0;
    const bool rowpart = (i0 - 1 < 1) || (i0 + R > N0 - 2);
    const int64_t K = (N1 + L - 2 + C - 1) / C;
    for (int64_t k = 0; k < K; ++k) {
      const bool colpart = (k == 0) || ((k + 1) * C > N1 - 1) || (k * C - (L - 1) < 1);
      if constexpr (TCUT) chunk<true, true>(g, sm, k, i0, g.a_final, aligned, cf);
      else if (rowpart || colpart) chunk<true, false>(g, sm, k, i0, g.a_final, aligned, cf);
      else chunk<false, false>(g, sm, k, i0, g.a_final, aligned, cf);
    }
  }
};

}  // namespace fast2d
}  // namespace hexs
