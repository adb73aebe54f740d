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
//   * the In rows of the NEXT super-chunk are staged into shared memory by 1-D bulk TMA
//     copies (one per row, 16-B aligned windows -- the aligned loads of Sec. 4.2.3,
//     PAPER.md:749-767), refilled level by level as soon as the current chunk has consumed
//     them and tracked by one mbarrier per level, so no warp waits on HBM latency;
//   * the level loop and the row loop are fully unrolled from the compile-time hexagon
//     shape (constraint-based unrolling, Sec. 4.3.2); full tiles run the
//     branch-free instantiation, tiles cut by the domain run predicated ones
//     (full/partial separation, Sec. 4.3.1).
#pragma once
#include <cstdint>
#include <type_traits>

#include "../stencil_ops.cuh"
#include "launch.h"
#include "tma.cuh"

#ifndef HEXS_MERGE_ROWP
#define HEXS_MERGE_ROWP 1
#endif
#ifndef HEXS_2D_DRIFT
#define HEXS_2D_DRIFT 0  // 1: no CTA barrier per level -- tail hand-off by mbarrier, last-arriver refill:
                         // bit-exact but measured slower (heat2d5 1672 -> 1212: warps serialise on
                         // their predecessor's tail, 168 vs 147 registers)
#endif
#ifndef HEXS_F2_2D
#define HEXS_F2_2D 0  // 1 measured slower: heat2d5 1551 -> 1379 GUp/s, box2d9 1151 -> 946 (FADD2 holds
                      // the FMA pipe 2 cycles, and the pair moves are IMADs on the same pipe)
#endif
#ifndef HEXS_MERGE_COLP
#define HEXS_MERGE_COLP 0  // 1 (all classes) measured slower: 1514 -> 1250 GUp/s star2d5 in round 1 (per-element
                           // selects), 1689 -> 1624 with the round-2 repair; gradient2d merges always
#endif

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
  using Elem = T;
  static constexpr int V = VecInfo<T>::V;
  static constexpr int VB = VecInfo<T>::VB;
  static constexpr int L = 2 * H + 2;        // levels per hexagon
  static constexpr int R = W0 + 2 * H + 1;   // max hexagon rows; local rows b in [0, R)
  static constexpr int Q = R + 2;            // register rows q = b + 1, b in [-1, R]
  static constexpr int NT = NW * 32;
  static constexpr int C = NT * V;           // super-chunk width (classical tile w1)
  // resident CTAs/SM the register budget targets: 12 (fp32) / 8 (fp64) warps per SM
  static constexpr int MINB = (sizeof(T) == 8 ? 8 : 12) / NW > 0 ? (sizeof(T) == 8 ? 8 : 12) / NW : 1;
  static constexpr int NIN = W0 + 4 * H + 5; // In rows per chunk (= In values per column)
  static constexpr int SW = C + 8;           // staged row width (elements), 16-B granular
  // fp32 linear classes can sweep two columns per instruction (F2 pairs: FADD2 / FFMA2, see
  // chunk_packed; the gradient's sqrt / div have no packed form) -- off by default, measured
  // slower (HEXS_F2_2D above)
  static constexpr bool kPacked = HEXS_F2_2D && std::is_same<T, float>::value && KIND != K_GRADIENT2D;
  // one body for column-partial chunks as well: measured faster for the gradient's small (1,1)
  // body (472 -> 518 GUp/s), slower for star / box (1689 -> 1624, 1381 -> 1331: two bodies fit)
  static constexpr bool kMergeColp = HEXS_MERGE_COLP || KIND == K_GRADIENT2D;

  struct Smem {
    uint64_t mbar[L];                 // one transaction barrier per level's In rows
#if HEXS_2D_DRIFT
    uint64_t tailbar[2][L][NW];       // (drift mode) tail of [chunk parity][level][warp] written
    unsigned cnt[L];                  // (drift mode) warps done with a level's In rows
#endif
    T tail[2][L][NW][Q][2];           // [chunk parity][level][warp][row][2 last columns]
    alignas(16) T inrows[NIN][SW];    // In rows of the current chunk (TMA-staged)
  };

  // ---- compile-time hexagon shape ----
  __host__ __device__ static constexpr int n_in(int a) {
    return a == 0 ? W0 + 3 : (a <= H ? 4 : (a == H + 1 ? 2 : 0));
  }
  __host__ __device__ static constexpr int slot_base(int a) {
    return a == 0 ? 0 : (a <= H ? W0 + 3 + 4 * (a - 1) : W0 + 3 + 4 * H);
  }
  // local row b of the i-th In row of level a
  __host__ __device__ static constexpr int in_row_b(int a, int i) {
    if (a == 0) return lo_row(H, W0, 0) - 1 + i;
    if (a <= H) {
      const int lo = lo_row(H, W0, a), hi = hi_row(H, W0, a);
      return i == 0 ? lo - 1 : (i == 1 ? lo : (i == 2 ? hi : hi + 1));
    }
    return i == 0 ? -1 : R;
  }
  __host__ __device__ static constexpr bool is_in_row(int a, int q) {   // loaded at level a
    for (int i = 0; i < n_in(a); ++i)
      if (in_row_b(a, i) == q - 1) return true;
    return false;
  }
  __host__ __device__ static constexpr int in_slot(int a, int q) {
    for (int i = 0; i < n_in(a); ++i)
      if (in_row_b(a, i) == q - 1) return slot_base(a) + i;
    return -1;
  }
  __host__ __device__ static constexpr bool is_input_row(int a, int q) {
    const int b = q - 1;
    return b >= lo_row(H, W0, a) - 1 && b <= hi_row(H, W0, a) + 1;
  }
  __host__ __device__ static constexpr bool is_out_row(int a, int q) {  // Out set (stored) at level a
    const int b = q - 1, lo = lo_row(H, W0, a), hi = hi_row(H, W0, a);
    if (b < lo || b > hi) return false;
    if (a < H) return false;
    if (a == H) return b == lo || b == hi;
    if (a < L - 1) return b <= lo + 1 || b >= hi - 1;
    return true;
  }
  // first column of the staged window of level a (16-B aligned: k*C and C are multiples of VB)
  __host__ __device__ static constexpr int win_shift(int a) {  // window start = k*C - win_shift(a)
    return a + 1 + (((-a - 1) % VB + VB) % VB);
  }

  // ---- producer: TMA the In rows of (chunk k, level a) into their slots (thread 0) ----
  static __device__ __forceinline__ void issue_level(const Fast2DArgs& g, Smem& sm, int64_t k, int a,
                                                     int64_t i0) {
    const int na = n_in(a);
    if (na == 0) return;
    const T* src = static_cast<const T*>(g.buf[(g.tau0 + a) & 1]);  // input level tau0 + a
    const int64_t N0 = g.N0, N1 = g.N1;
    const int64_t c0 = k * C - win_shift(a);
    const int64_t lo_c = c0 < 0 ? 0 : c0;
    const int64_t hi_c = (c0 + SW) > N1 ? N1 : (c0 + SW);
    const uint32_t bytes = hi_c > lo_c ? (uint32_t)((hi_c - lo_c) * sizeof(T)) : 0u;
    mbar_arrive_expect_tx(&sm.mbar[a], bytes * na);
    if (bytes == 0) return;
    for (int i = 0; i < na; ++i) {
      int64_t row = i0 + in_row_b(a, i);
      row = row < 0 ? 0 : (row >= N0 ? N0 - 1 : row);
      tma_load_1d(&sm.inrows[slot_base(a) + i][lo_c - c0], src + row * N1 + lo_c, bytes, &sm.mbar[a]);
    }
  }

  // Direct (non-TMA) load of V+2 consecutive elements starting at column `start` of global
  // row `row` (unaligned rows or time-cut tiles); clamped into the grid.
  static __device__ __forceinline__ void load_direct(const T* src, int64_t N1, int64_t row, int start,
                                                     T (&dst)[V + 2]) {
    const T* rp = src + row * N1;
#pragma unroll
    for (int i = 0; i < V + 2; ++i) {
      int64_t col = (int64_t)start + i;
      col = col < 0 ? 0 : (col >= N1 ? N1 - 1 : col);
      dst[i] = rp[col];
    }
  }

  // One super-chunk: all levels of columns [k*C - a, k*C - a + C).
  //   TMA : In rows come from the TMA-staged slots (else direct global loads)
  //   ROWP: hexagon rows cross the domain's row boundary (per-row uniform predicate)
  //   COLP: chunk crosses a column boundary (per-element predicate)
  //   TCUT: tile cut at t = 0 / t = T (levels outside [a_lo, a_hi] skipped at run time)
  template <bool TMA, bool ROWP, bool COLP, bool TCUT>
  static __device__ __forceinline__ void chunk(const Fast2DArgs& g, Smem& sm, int64_t k, int64_t K,
                                               int64_t i0, const Coef<T>& cf) {
    if constexpr (kPacked) {
      chunk_packed<TMA, ROWP, COLP, TCUT>(g, sm, k, K, i0, cf);
      return;
    }
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
      const bool first = TCUT ? (a == g.a_lo) : (a == 0);

      // ---- (1) the In rows of this level have landed (TMA mode) ----
      if constexpr (TMA) {
        static_assert(!TCUT, "TMA staging runs full-time tiles only");
        if constexpr (n_in(a) > 0) mbar_wait_parity(&sm.mbar[a], (uint32_t)(k & 1));
      }
#if HEXS_2D_DRIFT
      // drift mode: the previous warp's (previous chunk's last warp's) level a-1 tail is written
      if constexpr (TMA && a > 0) {
        if (warp > 0) {
          mbar_wait_parity(&sm.tailbar[k & 1][a - 1][warp - 1], (uint32_t)((k >> 1) & 1));
        } else if (k > 0) {
          mbar_wait_parity(&sm.tailbar[(k - 1) & 1][a - 1][NW - 1], (uint32_t)(((k - 1) >> 1) & 1));
        }
      }
#endif

      // ---- (2)-(5) rows ascending: inputs just in time, compute, copy out, tail ----
      const int pw = warp == 0 ? NW - 1 : warp - 1;
      const int pk = warp == 0 ? (int)((k - 1) & 1) : (int)(k & 1);
      // Input row q of level a, fetched right before its first use (keeps the register
      // footprint at ~one level of rows): In rows come from the TMA-staged slot (or global
      // memory) with their two left-halo columns; rows computed at the previous level take
      // the two last columns of the left lane (shuffle) or, in lane 0, of the previous warp /
      // chunk (shared-memory tail).
      auto halo = [&](auto q_c) {
        constexpr int q = decltype(q_c)::value;
        if constexpr (TMA && is_in_row(a, q)) {
          constexpr int M = win_shift(a) - a - 1;  // window offset of the thread's first input column
          constexpr int NB = (M + V + 2 + VB - 1) / VB;
          const T* rowp = &sm.inrows[in_slot(a, q)][tid * V];
          T blk[NB * VB];
#pragma unroll
          for (int i = 0; i < NB; ++i) {
            if constexpr (VB == 4) {
              const float4 v4 = reinterpret_cast<const float4*>(rowp)[i];
              blk[4 * i] = v4.x; blk[4 * i + 1] = v4.y; blk[4 * i + 2] = v4.z; blk[4 * i + 3] = v4.w;
            } else {
              const double2 v2 = reinterpret_cast<const double2*>(rowp)[i];
              blk[2 * i] = v2.x; blk[2 * i + 1] = v2.y;
            }
          }
#pragma unroll
          for (int i = 0; i < V + 2; ++i) in[q][i] = blk[M + i];
        } else if constexpr (!TMA && is_input_row(a, q)) {
          if (first || is_in_row(a, q)) {
            int64_t row = i0 + (q - 1);
            row = row < 0 ? 0 : (row >= N0 ? N0 - 1 : row);
            load_direct(src, N1, row, colbase - 1, in[q]);
          }
        }
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
        colok[v] = !COLP || (c >= 1 && c <= (int)N1 - 2);
      }
      const bool fin = TCUT && (a == g.a_final);
      T* dbase = dst + i0 * N1 + colbase;
      static_for<qlo, qhi + 1>([&](auto q_c) {
        constexpr int q = decltype(q_c)::value;
        halo(std::integral_constant<int, q + 1>{});
        const int64_t row = i0 + (q - 1);
        const bool rowok = !ROWP || (row >= 1 && row <= N0 - 2);
#pragma unroll
        for (int v = 0; v < V; ++v) {
          T x[3][3];
#pragma unroll
          for (int r = 0; r < 3; ++r)
#pragma unroll
            for (int c = 0; c < 3; ++c) x[r][c] = in[q - 1 + r][v + c];
          out[q][v] = apply<T, KIND>(x, cf);
        }
        // interleaved copy-out of the Out set (every row at the final level); Dirichlet and
        // out-of-domain cells are never stored
        if (is_out_row(a, q) || fin) {
          if (rowok) {
            T* rp = dbase + (int64_t)(q - 1) * N1;
#pragma unroll
            for (int v = 0; v < V; ++v)
              if (colok[v]) rp[v] = out[q][v];
          }
        }
      });
      // Dirichlet cells keep their value: one branch per level instead of a select per
      // element -- only the edge hexagons' levels that reach row 0 / N0-1 (CTA-uniform) and
      // the threads holding a column outside [1, N1-2] enter it; the repaired values are the
      // ones the next level and the tail see (out-of-domain cells feed only repaired cells)
      if constexpr (ROWP || COLP) {
        const bool rfix = ROWP && (i0 + (qlo - 1) < 1 || i0 + (qhi - 1) > N0 - 2);
        bool cfix = false;
#pragma unroll
        for (int v = 0; v < V; ++v) cfix |= !colok[v];
        if (rfix || cfix) {
#pragma unroll
          for (int q = qlo; q <= qhi; ++q) {
            const int64_t row = i0 + (q - 1);
            const bool rowok = !ROWP || (row >= 1 && row <= N0 - 2);
#pragma unroll
            for (int v = 0; v < V; ++v)
              if (!(rowok && colok[v])) out[q][v] = in[q][v + 1];
          }
        }
      }
      // tail for the next warp / next super-chunk (one branch for all rows)
      if constexpr (a < L - 1) {
        if (lane == 31) {
#pragma unroll
          for (int q = qlo; q <= qhi; ++q) {
            sm.tail[k & 1][a][warp][q][0] = out[q][V - 2];
            sm.tail[k & 1][a][warp][q][1] = out[q][V - 1];
          }
#if HEXS_2D_DRIFT
          if constexpr (TMA) mbar_arrive(&sm.tailbar[k & 1][a][warp]);  // release
#endif
        }
      }
#if HEXS_2D_DRIFT
      constexpr bool kDrift = TMA;
#else
      constexpr bool kDrift = false;
#endif
      if constexpr (kDrift) {
#if HEXS_2D_DRIFT
        // ---- refill without a CTA barrier: the last warp done with level a's In rows issues
        // chunk k+1's (its fence orders every warp's reads before the async-proxy writes) ----
        if constexpr (n_in(a) > 0) {
          __syncwarp();
          if (lane == 0) {
            __threadfence_block();
            const unsigned old = atomicAdd(&sm.cnt[a], 1u);
            if (old == NW - 1) {
              sm.cnt[a] = 0u;
              __threadfence_block();
              if (k + 1 < K) {
                fence_proxy_async_smem();
                issue_level(g, sm, k + 1, a, i0);
              }
            }
          }
        }
#endif
      } else {
      __syncthreads();
      // ---- refill: the consumed slots of level a take chunk k+1's In rows ----
      if constexpr (TMA && n_in(a) > 0) {
        if (tid == 0 && k + 1 < K) {
          fence_proxy_async_smem();
          issue_level(g, sm, k + 1, a, i0);
        }
      }
      }
      // ---- (6) the outputs become the next level's inputs ----
#pragma unroll
      for (int q = qlo; q <= qhi; ++q)
#pragma unroll
        for (int v = 0; v < V; ++v) in[q][v + 2] = out[q][v];
    });
  }

  // The same super-chunk with the level held as F2 pairs (fp32 linear classes).  With in[0..5]
  // the scalar path's input row (2 halo columns + the thread's 4), a row is held as
  //   P[q][0] = (in0, in2), P[q][1] = (in1, in3), P[q][2] = (in2, in4), P[q][3] = (in3, in5)
  // so the 3x3 operand window of outputs v and v+2 (p = v = 0, 1) is the pairs P[q-1..q+1]
  // [p .. p+2] with no data movement, and the two output pairs (out0, out2), (out1, out3)
  // ARE the next level's P[q][2], P[q][3]; P[q][0], P[q][1] take the left lane's out2 /
  // out3 by shuffle plus one move each.  Every point is the scalar expression (stencil_ops,
  // instantiated on F2), so results are bit-identical to the scalar sweep.
  template <bool TMA, bool ROWP, bool COLP, bool TCUT>
  static __device__ __forceinline__ void chunk_packed(const Fast2DArgs& g, Smem& sm, int64_t k, int64_t K,
                                                      int64_t i0, const Coef<T>& cf) {
    static_assert(V == 4, "packed sweep: fp32 quads");
    const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
    const int64_t N0 = g.N0, N1 = g.N1;
    const Coef<F2> cf2{f2_pack((float)cf.k0, (float)cf.k0), f2_pack((float)cf.k1, (float)cf.k1)};
    F2 P[Q][4];
    auto set_row = [&](F2 (&r)[4], const T (&x)[V + 2]) {
      r[0] = f2_pack(x[0], x[2]);
      r[1] = f2_pack(x[1], x[3]);
      r[2] = f2_pack(x[2], x[4]);
      r[3] = f2_pack(x[3], x[5]);
    };
#pragma unroll
    for (int q = 0; q < Q; ++q)
#pragma unroll
      for (int v = 0; v < 4; ++v) P[q][v] = f2_pack(0.f, 0.f);

    static_for<0, L>([&](auto a_c) {
      constexpr int a = decltype(a_c)::value;
      if constexpr (TCUT) {
        if (a < g.a_lo || a > g.a_hi) return;
      }
      const int64_t tau = g.tau0 + a;
      const T* src = static_cast<const T*>(g.buf[tau & 1]);
      T* dst = static_cast<T*>(g.buf[(tau + 1) & 1]);
      const int colbase = (int)k * C - a + tid * V;
      const bool first = TCUT ? (a == g.a_lo) : (a == 0);
      if constexpr (TMA) {
        static_assert(!TCUT, "TMA staging runs full-time tiles only");
        if constexpr (n_in(a) > 0) mbar_wait_parity(&sm.mbar[a], (uint32_t)(k & 1));
      }
      const int pw = warp == 0 ? NW - 1 : warp - 1;
      const int pk = warp == 0 ? (int)((k - 1) & 1) : (int)(k & 1);
      auto halo = [&](auto q_c) {
        constexpr int q = decltype(q_c)::value;
        if constexpr (TMA && is_in_row(a, q)) {
          constexpr int M = win_shift(a) - a - 1;
          constexpr int NB = (M + V + 2 + VB - 1) / VB;
          const T* rowp = &sm.inrows[in_slot(a, q)][tid * V];
          T blk[NB * VB];
#pragma unroll
          for (int i = 0; i < NB; ++i) {
            const float4 v4 = reinterpret_cast<const float4*>(rowp)[i];
            blk[4 * i] = v4.x; blk[4 * i + 1] = v4.y; blk[4 * i + 2] = v4.z; blk[4 * i + 3] = v4.w;
          }
          T x[V + 2];
#pragma unroll
          for (int i = 0; i < V + 2; ++i) x[i] = blk[M + i];
          set_row(P[q], x);
        } else if constexpr (!TMA && is_input_row(a, q)) {
          if (first || is_in_row(a, q)) {
            int64_t row = i0 + (q - 1);
            row = row < 0 ? 0 : (row >= N0 ? N0 - 1 : row);
            T x[V + 2];
            load_direct(src, N1, row, colbase - 1, x);
            set_row(P[q], x);
          }
        }
        if constexpr (is_input_row(a, q) && !is_in_row(a, q) && a > 0) {
          if (!first) {
            float c0, c2, c1, c3;
            f2_unpack(P[q][2], c0, c2);  // own out0, out2 of level a-1
            f2_unpack(P[q][3], c1, c3);  // own out1, out3
            T h0 = __shfl_up_sync(0xffffffffu, c2, 1);
            T h1 = __shfl_up_sync(0xffffffffu, c3, 1);
            if (lane == 0) {
              h0 = sm.tail[pk][a - 1][pw][q][0];
              h1 = sm.tail[pk][a - 1][pw][q][1];
            }
            P[q][0] = f2_pack(h0, c0);
            P[q][1] = f2_pack(h1, c1);
          }
        }
      };
      constexpr int qlo = lo_row(H, W0, a) + 1, qhi = hi_row(H, W0, a) + 1;
      halo(std::integral_constant<int, qlo - 1>{});
      halo(std::integral_constant<int, qlo>{});
      F2 O[Q][2];
      bool colok[V];
#pragma unroll
      for (int v = 0; v < V; ++v) {
        const int c = colbase + v;
        colok[v] = !COLP || (c >= 1 && c <= (int)N1 - 2);
      }
      const bool fin = TCUT && (a == g.a_final);
      T* dbase = dst + i0 * N1 + colbase;
      static_for<qlo, qhi + 1>([&](auto q_c) {
        constexpr int q = decltype(q_c)::value;
        halo(std::integral_constant<int, q + 1>{});
        const int64_t row = i0 + (q - 1);
        const bool rowok = !ROWP || (row >= 1 && row <= N0 - 2);
        static_for<0, 2>([&](auto p_c) {
          constexpr int p = decltype(p_c)::value;
          F2 x[3][3];
#pragma unroll
          for (int r = 0; r < 3; ++r)
#pragma unroll
            for (int c = 0; c < 3; ++c) x[r][c] = P[q - 1 + r][p + c];
          F2 val = apply<F2, KIND>(x, cf2);
          if constexpr (ROWP || COLP) {
            // keep (Dirichlet) old values: outputs p, p+2 hold in[p+1], in[p+3] = P[q][p+1]
            float v0, v2, o0, o2;
            f2_unpack(val, v0, v2);
            f2_unpack(P[q][p + 1], o0, o2);
            v0 = (rowok && colok[p]) ? v0 : o0;
            v2 = (rowok && colok[p + 2]) ? v2 : o2;
            val = f2_pack(v0, v2);
          }
          O[q][p] = val;
        });
        if (is_out_row(a, q) || fin) {
          if (rowok) {
            float o[4];
            f2_unpack(O[q][0], o[0], o[2]);
            f2_unpack(O[q][1], o[1], o[3]);
            T* rp = dbase + (int64_t)(q - 1) * N1;
#pragma unroll
            for (int v = 0; v < V; ++v)
              if (colok[v]) rp[v] = o[v];
          }
        }
        if constexpr (a < L - 1) {
          if (lane == 31) {
            float o0, o2, o1, o3;
            f2_unpack(O[q][0], o0, o2);
            f2_unpack(O[q][1], o1, o3);
            sm.tail[k & 1][a][warp][q][0] = o2;
            sm.tail[k & 1][a][warp][q][1] = o3;
          }
        }
      });
      __syncthreads();
      if constexpr (TMA && n_in(a) > 0) {
        if (tid == 0 && k + 1 < K) {
          fence_proxy_async_smem();
          issue_level(g, sm, k + 1, a, i0);
        }
      }
#pragma unroll
      for (int q = qlo; q <= qhi; ++q) {
        P[q][2] = O[q][0];
        P[q][3] = O[q][1];
      }
    });
  }

  static __device__ __forceinline__ int64_t n_chunks(const Fast2DArgs& g) {
    return (g.N1 + L - 2 + C - 1) / C;
  }
  static __device__ __forceinline__ bool col_partial(const Fast2DArgs& g, int64_t k) {
    return (k == 0) || ((k + 1) * C > g.N1 - 1) || (k * C - (L - 1) < 1);
  }

  // Full-time tiles, 16-B aligned rows: TMA-staged In rows.
  static __device__ __forceinline__ void run_tma(const Fast2DArgs& g, Smem& sm) {
    const int64_t S0 = g.S0_lo + blockIdx.x;
    const int64_t i0 = S0 * g.W - g.row_off;  // global row of local row b = 0
    const Coef<T> cf{(T)g.k0, (T)g.k1};
    const bool rowpart = (i0 - 1 < 1) || (i0 + R > g.N0 - 2);
    const int64_t K = n_chunks(g);
    if (threadIdx.x == 0) {
#pragma unroll
      for (int a = 0; a < L; ++a) mbar_init(&sm.mbar[a], 1);
#if HEXS_2D_DRIFT
      for (int a = 0; a < L; ++a) {
        sm.cnt[a] = 0u;
        for (int w = 0; w < NW; ++w) {
          mbar_init(&sm.tailbar[0][a][w], 1);
          mbar_init(&sm.tailbar[1][a][w], 1);
        }
      }
#endif
      mbar_fence_init();
    }
    __syncthreads();
    if (threadIdx.x == 0) {
#pragma unroll
      for (int a = 0; a < L; ++a) issue_level(g, sm, 0, a, i0);
    }
    for (int64_t k = 0; k < K; ++k) {
      const bool colpart = col_partial(g, k);
#if HEXS_MERGE_ROWP
      // One code body for interior and row-partial hexagons (a per-element select on the
      // row predicate): co-resident CTAs then share the instruction stream instead of
      // thrashing the instruction cache with two ~70 KB bodies.
      (void)rowpart;
      if constexpr (kMergeColp) {
        // column-partial chunks share the body too (column repair per level, store predicates)
        (void)colpart;
        chunk<true, true, true, false>(g, sm, k, K, i0, cf);
      } else {
        if (colpart) chunk<true, true, true, false>(g, sm, k, K, i0, cf);
        else chunk<true, true, false, false>(g, sm, k, K, i0, cf);
      }
#else
      if (rowpart) {
        if (colpart) chunk<true, true, true, false>(g, sm, k, K, i0, cf);
        else chunk<true, true, false, false>(g, sm, k, K, i0, cf);
      } else {
        if (colpart) chunk<true, false, true, false>(g, sm, k, K, i0, cf);
        else chunk<true, false, false, false>(g, sm, k, K, i0, cf);
      }
#endif
    }
  }

  // Unaligned rows (TCUT = false) or time-cut tiles (TCUT = true): direct loads, predicated.
  template <bool TCUT>
  static __device__ __forceinline__ void run_direct(const Fast2DArgs& g, Smem& sm) {
    const int64_t S0 = g.S0_lo + blockIdx.x;
    const int64_t i0 = S0 * g.W - g.row_off;
    const Coef<T> cf{(T)g.k0, (T)g.k1};
    const int64_t K = n_chunks(g);
    for (int64_t k = 0; k < K; ++k) chunk<false, true, true, TCUT>(g, sm, k, K, i0, cf);
  }
};

}  // namespace fast2d
}  // namespace hexs
