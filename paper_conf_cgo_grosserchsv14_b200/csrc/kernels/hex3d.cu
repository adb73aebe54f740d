// hex3d.cu -- the specialised sm_100a phase kernel for 3D single-field stencils of radius 1
// (star3d7, gradient3d, box3d27) under the hybrid schedule: hexagonal over (t, z), classical
// parallelogram tiles over y and x (eq. (14)).
//
// Mapping:
//   * work item = one classical tile (S1, S2) of one hexagon S0 of the launch's (T, p): an
//     NY x NX (y, x) parallelogram over the hexagon's 2h+2 levels and its rows z.  Skews: y
//     by 1 per level (delta1_y = 1), x by 4 per level (any integer skew >= delta1_x keeps
//     eq. (14) valid, reading R16) so every x-window this kernel moves is 16-B aligned;
//   * the tile keeps ALL its levels on chip: level a reads a shared-memory buffer holding
//     level a-1 (rows x (NY+2) lines x (NX+5) columns) and writes the other buffer;
//   * tile-granular dependences: the skew makes every dependence point to a tile with
//     component-wise larger-or-equal (S1, S2), so a tile whose predecessors (S1-1, S2) and
//     (S1, S2-1) have COMPLETED finds every value it reads, at every level, in global memory.
//     Persistent CTAs take tiles in anti-diagonal order (S1 + S2, then S0, then S1), wait for
//     the two predecessor flags once, and publish their own flag once (st.release.gpu) --
//     no per-level cross-SM synchronisation;
//   * everything a tile reads from L2/HBM arrives by 3-D TMA tensor copies (SASS UTMALDG)
//     completing on one mbarrier per buffer, one level ahead of the compute: the first level
//     (issued during the previous tile's last level, which writes no shared memory), then
//     per level the hexagon's In rows (its slanted-edge inputs) and the
//     carries the predecessor tiles produced: 2 lines above and 5 columns left, staged into
//     their own dense areas (a TMA box lands densely, so each area matches one box);
//   * a thread owns one line and 4 consecutive x of the tile and sweeps z with a 3-row
//     register window (z neighbours from registers, y neighbours from the level buffer, x
//     edges by shuffle inside 8-lane groups);
//   * results leave from registers: the Out rows (slanted upper edges and top row), every
//     value of level T_steps, and the tile's last 2 lines / last 5 columns of every level
//     (its successors' carries) -- interleaved copy-out.
#include <cuda.h>
#include <cudaTypedefs.h>

#include <cstdint>
#include <type_traits>

#include "../stencil_ops.cuh"
#include "launch.h"
#include "tma.cuh"

namespace hexs {
namespace fast3d {

constexpr int NX = kFast3DNX;  // tile columns (x)
constexpr int NQ = NX / 4;     // column quads: one 8-lane group
constexpr int SIGMA = 4;       // x skew per level
template <typename T> constexpr int NY = sizeof(T) == 4 ? 32 : 16;  // tile lines (y)
template <typename T> constexpr int NT = NY<T> * NQ;                 // threads: one per (line, quad)
constexpr int CC = 8;          // carry-area columns (x = X0 - 4a - 4 .. X0 - 4a + 3)

// Per buffer (level a's input = level a-1 values), Q rows (b = lo_min - 1 + r):
//   main  [Q][NY][NX]     own region: y = Y0 - a + 1 + l, x = X0 - 4a + 4 + m
//   lines [Q][2][NX]      carry lines: y = Y0 - a - 1 + l, x as main
//   carry [Q][NY+2][CC]   carry columns: y = Y0 - a - 1 + l, x = X0 - 4a - 4 + c
template <typename T> struct Lay {
  static constexpr int MAIN = NY<T> * NX, LINES = 2 * NX, CARRY = (NY<T> + 2) * CC;
  static constexpr int ROW = MAIN + LINES + CARRY;  // elements per row (all areas)
};
// one buffer, padded so the second one stays 128-B aligned (TMA destinations)
template <typename T> __host__ __device__ constexpr size_t buf_elems(int Q) {
  return ((size_t)Q * Lay<T>::ROW * sizeof(T) + 127) / 128 * 128 / sizeof(T);
}
template <typename T> constexpr size_t smem_bytes(int Q) { return 2 * buf_elems<T>(Q) * sizeof(T); }

struct Maps {
  CUtensorMap main[2];   // box {NX, NY, Q}
  CUtensorMap lines[2];  // box {NX, 2, Q}
  CUtensorMap carry[2];  // box {CC, NY+2, Q}
  CUtensorMap in2[2];    // box {NX, NY, 2}
  CUtensorMap in1[2];    // box {NX, NY, 1}
};

__device__ __forceinline__ int ld_acquire(const int* p) {
  int v;
  asm volatile("ld.acquire.gpu.global.b32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void st_release(int* p, int v) {
  asm volatile("st.release.gpu.global.b32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}
// order the acquired generic-proxy view of global memory before later async-proxy reads
__device__ __forceinline__ void fence_proxy_async_global() { asm volatile("fence.proxy.async.global;" ::: "memory"); }
__device__ __forceinline__ void tma_3d(void* dst, const CUtensorMap* map, int x, int y, int z, uint64_t* bar) {
  asm volatile(
      "cp.async.bulk.tensor.3d.shared::cluster.global.tile.mbarrier::complete_tx::bytes [%0], [%1, {%2, %3, %4}], [%5];" ::"r"(
          smem_u32(dst)),
      "l"(reinterpret_cast<uint64_t>(map)), "r"(x), "r"(y), "r"(z), "r"(smem_u32(bar))
      : "memory");
}

template <typename T, int KIND>
__device__ __forceinline__ T apply(const T (&x)[3][3][3], const Coef<T>& k) {
  // x[dz][dy][dx], offsets -1..1
  if constexpr (KIND == K_STAR3D7)
    return star3d7<T>(x[1][1][1], x[1][0][1], x[1][2][1], x[1][1][0], x[1][1][2], x[0][1][1], x[2][1][1], k);
  else if constexpr (KIND == K_GRADIENT3D)
    return gradient3d<T>(x[1][1][1], x[1][0][1], x[1][2][1], x[1][1][0], x[1][1][2], x[0][1][1], x[2][1][1], k);
  else {
    T acc = x[0][0][0];
#pragma unroll
    for (int q = 1; q < 27; ++q) acc = acc + x[q / 9][(q / 3) % 3][q % 3];
    return k.k0 * acc;
  }
}

// v = pred ? *p : v as one predicated shared-memory load
__device__ __forceinline__ float lds_if(bool pred, const float* p, float v) {
  asm volatile("{\n.reg .pred q;\nsetp.ne.b32 q, %1, 0;\n@q ld.shared.f32 %0, [%2];\n}\n"
               : "+f"(v)
               : "r"((int)pred), "r"(smem_u32(p)));
  return v;
}
__device__ __forceinline__ double lds_if(bool pred, const double* p, double v) {
  asm volatile("{\n.reg .pred q;\nsetp.ne.b32 q, %1, 0;\n@q ld.shared.f64 %0, [%2];\n}\n"
               : "+d"(v)
               : "r"((int)pred), "r"(smem_u32(p)));
  return v;
}

// A thread's operand window of one row: 3 lines (y-1, y, y+1) x 6 columns (x-1 .. x+4 of its
// 4 outputs).  Centre quads are aligned vector loads; edges come from the neighbouring lanes
// of the 8-lane group by shuffle, the group's outer lanes read theirs (the carry column /
// the column past the tile's quads).  Unused values are dead code.  Warp-uniform calls.
template <typename T> struct Win { T v[3][6]; };

template <typename T, bool ALL_EDGES>  // star / gradient stencils need the centre line's edges only
__device__ __forceinline__ void load_win(Win<T>& w, const T* const (&p)[3], int q) {
#pragma unroll
  for (int l = 0; l < 3; ++l) {
    if constexpr (sizeof(T) == 4) {
      const float4 u = reinterpret_cast<const float4*>(p[l])[0];
      w.v[l][1] = u.x; w.v[l][2] = u.y; w.v[l][3] = u.z; w.v[l][4] = u.w;
    } else {
      const double2 u0 = reinterpret_cast<const double2*>(p[l])[0];
      const double2 u1 = reinterpret_cast<const double2*>(p[l])[1];
      w.v[l][1] = u0.x; w.v[l][2] = u0.y; w.v[l][3] = u1.x; w.v[l][4] = u1.y;
    }
    // interior edges by shuffle; the group's outer lanes load theirs with a predicated
    // LDS (no branch, so the warp never diverges around the shuffles)
    if (ALL_EDGES || l == 1) {
      w.v[l][0] = lds_if(q == 0, p[l] - 1, __shfl_up_sync(0xffffffffu, w.v[l][4], 1, NQ));
      w.v[l][5] = lds_if(q == NQ - 1, p[l] + 4, __shfl_down_sync(0xffffffffu, w.v[l][1], 1, NQ));
    } else {
      w.v[l][0] = w.v[l][5] = T(0);  // never used by this stencil
    }
  }
}

template <typename T, int KIND>
__global__ void __launch_bounds__(NT<T>, 1) fast3d_kernel(const __grid_constant__ Fast3DArgs g,
                                                          const __grid_constant__ Maps mp) {
  constexpr int LNY = NY<T>;
  using LY = Lay<T>;
  extern __shared__ __align__(1024) unsigned char smem_raw[];  // dynamic base: 1024-B aligned
  T* const sbase = reinterpret_cast<T*>(smem_raw);  // stays a shared-space pointer (LDS/STS)
  __shared__ __align__(8) uint64_t full[2];
  __shared__ long long item_s[2][3];  // [current, next] (S0, q1, q2); S0 < 0: none
  const int tid = threadIdx.x;
  const int ly = tid / NQ, q = tid % NQ;  // line, column quad
  const int Q = g.Q;
  const int64_t n1 = g.n1, n2 = g.n2, ns0 = g.S0_hi - g.S0_lo + 1, n_items = ns0 * n1 * n2;
  const int64_t N0 = g.N0, N1 = g.N1, N2 = g.N2, plane = N1 * N2;
  int lo_min = 1 << 30;
  for (int a = 0; a < g.L; ++a) lo_min = min(lo_min, (int)g.lo[a]);
  const int zoff = lo_min - 1;  // b of buffer row 0
  const int BE = (int)buf_elems<T>(Q);
  auto main_of = [&](int b) { return sbase + b * BE; };
  auto lines_of = [&](int b) { return sbase + b * BE + Q * LY::MAIN; };
  auto carry_of = [&](int b) { return sbase + b * BE + Q * (LY::MAIN + LY::LINES); };

  if (tid == 0) {
    mbar_init(&full[0], 1);
    mbar_init(&full[1], 1);
    mbar_fence_init();
  }
  // decode the anti-diagonal order: d = q1 + q2 (outer), then S0, then q1
  auto decode = [&](int64_t it, long long* o) {
    o[0] = -1;
    if (it >= n_items) return;
    int64_t off = 0;
    for (int64_t d = 0; d < n1 + n2 - 1; ++d) {
      const int64_t lo1 = d - (n2 - 1) > 0 ? d - (n2 - 1) : 0;
      const int64_t hi1 = d < n1 - 1 ? d : n1 - 1;
      const int64_t pairs = hi1 - lo1 + 1;
      if (it < off + pairs * ns0) {
        const int64_t r = it - off;
        o[0] = g.S0_lo + r / pairs;
        o[1] = lo1 + r % pairs;
        o[2] = d - o[1];
        return;
      }
      off += pairs * ns0;
    }
  };
  auto tile_origin = [&](const long long* it, int64_t& i0, int& X0, int& Y0) {
    i0 = it[0] * g.W - g.row_off;
    Y0 = (int)((g.S1_lo + it[1]) * LNY);
    X0 = (int)((g.S2_lo + it[2]) * NX);
  };
  // Level a's input buffer a & 1 for a tile: the parts that come from global memory (all of
  // it for the first level, else carry lines / columns + In rows).  Thread 0 only.
  auto issue_level = [&](const long long* it, int a, bool first) {
    int64_t i0;
    int X0, Y0;
    tile_origin(it, i0, X0, Y0);
    const int b = a & 1, par = (int)((g.tau0 + a) & 1);
    const int z0 = (int)(i0 + zoff);
    const int xo = X0 - SIGMA * a, yo = Y0 - a;
    uint32_t elems = (uint32_t)(Q * (LY::LINES + LY::CARRY));
    // In rows of level a: buffer rows level a reads ([lo(a)-1, hi(a)+1]) that level a-1
    // does not compute
    int in_lo[2] = {0, 0}, in_n[2] = {0, 0};
    if (first) {
      elems += (uint32_t)(Q * LY::MAIN);
    } else {
      const int need_lo = g.lo[a] - 1, need_hi = g.hi[a] + 1, clo = g.lo[a - 1], chi = g.hi[a - 1];
      if (need_lo < clo) in_lo[0] = need_lo, in_n[0] = clo - need_lo;
      if (need_hi > chi) in_lo[1] = chi + 1, in_n[1] = need_hi - chi;
      elems += (uint32_t)((in_n[0] + in_n[1]) * LY::MAIN);
    }
    fence_proxy_async_smem();  // earlier generic accesses of this buffer before TMA writes
    mbar_arrive_expect_tx(&full[b], elems * (uint32_t)sizeof(T));
    tma_3d(lines_of(b), &mp.lines[par], xo + 4, yo - 1, z0, &full[b]);
    tma_3d(carry_of(b), &mp.carry[par], xo - 4, yo - 1, z0, &full[b]);
    if (first) {
      tma_3d(main_of(b), &mp.main[par], xo + 4, yo + 1, z0, &full[b]);
    } else {
      for (int s = 0; s < 2; ++s) {
        for (int k = 0; k < in_n[s];) {  // In rows: boxes of 2 rows, then 1
          const int bb = in_lo[s] + k;
          T* dst = main_of(b) + (size_t)(bb - zoff) * LY::MAIN;
          if (in_n[s] - k >= 2) {
            tma_3d(dst, &mp.in2[par], xo + 4, yo + 1, (int)(i0 + bb), &full[b]);
            k += 2;
          } else {
            tma_3d(dst, &mp.in1[par], xo + 4, yo + 1, (int)(i0 + bb), &full[b]);
            k += 1;
          }
        }
      }
    }
  };

  uint32_t ph = 0u;  // parity bit per buffer
  const Coef<T> cf{(T)g.k0, (T)g.k1};
  // the next tile's first level can be staged during this tile's last level (which writes
  // no shared memory) when that buffer is the other one: a_hi - a_lo odd
  const bool early = ((g.a_hi - g.a_lo) & 1) != 0;
  if (tid == 0) {
    decode((int64_t)atomicAdd(g.counter, 1ull), item_s[0]);
    if (item_s[0][0] >= 0) issue_level(item_s[0], g.a_lo, true);
  }
  __syncthreads();
  int cur = 0;
  while (true) {
    const long long* it = item_s[cur];
    if (it[0] < 0) break;
    int64_t i0;
    int X0, Y0;
    tile_origin(it, i0, X0, Y0);
    const int64_t base = (it[0] - g.S0_lo) * n1 * n2;
    int* const my_flag = g.flags + base + it[1] * n2 + it[2];
    bool deps_ok = false;
    for (int a = g.a_lo; a <= g.a_hi; ++a) {
      const int b = a & 1, nb = b ^ 1;
      mbar_wait_parity(&full[b], (ph >> b) & 1u);
      ph ^= 1u << b;
      __syncthreads();  // level a-1's buffer writes visible; buffer nb no longer read
      if (tid == 0) {
        if (a < g.a_hi) {
          if (!deps_ok) {  // predecessors complete: their carries are in global memory
            if (it[1] > 0)
              while (ld_acquire(g.flags + base + (it[1] - 1) * n2 + it[2]) == 0) __nanosleep(32);
            if (it[2] > 0)
              while (ld_acquire(g.flags + base + it[1] * n2 + it[2] - 1) == 0) __nanosleep(32);
            fence_proxy_async_global();
            deps_ok = true;
          }
          issue_level(it, a + 1, false);
        } else {
          decode((int64_t)atomicAdd(g.counter, 1ull), item_s[cur ^ 1]);
          if (early && item_s[cur ^ 1][0] >= 0) issue_level(item_s[cur ^ 1], g.a_lo, true);
        }
      }

      // ---- compute level a: line y = Y0 - a + ly, x = X0 - 4a + 4q + j, rows [lo, hi]
      const int rlo = g.lo[a], rhi = g.hi[a];
      const int y = Y0 - a + ly;
      const int xb = X0 - SIGMA * a + 4 * q;
      const bool to_smem = a < g.a_hi;
      // window line pointers (input-frame line l = ly + k) at buffer row rlo - 1
      const T* P[3];
      int pitch[3];
#pragma unroll
      for (int k = 0; k < 3; ++k) {
        const int l = ly + k, r = rlo - 1 - zoff;
        if (q == 0) {
          P[k] = carry_of(b) + ((size_t)r * (LNY + 2) + l) * CC + 4;
          pitch[k] = (LNY + 2) * CC;
        } else if (l < 2) {
          P[k] = lines_of(b) + ((size_t)r * 2 + l) * NX + 4 * q - 4;
          pitch[k] = 2 * NX;
        } else {
          P[k] = main_of(b) + ((size_t)r * LNY + l - 2) * NX + 4 * q - 4;
          pitch[k] = LY::MAIN;
        }
      }
      T* const Wn = main_of(nb) + ((size_t)(rlo - zoff) * LNY + ly) * NX + 4 * q;  // row rlo of level a
      // per-output masks: interior in (y, x); successors' carries (last 2 lines, last 5 cols)
      uint32_t vmask = 0u;
#pragma unroll
      for (int j = 0; j < 4; ++j)
        vmask |= (y >= 1 && y <= N1 - 2 && xb + j >= 1 && xb + j <= N2 - 2 ? 1u : 0u) << j;
      const uint32_t cstatic = (ly >= LNY - 2) ? 0xFu : (q == NQ - 1 ? 0xFu : (q == NQ - 2 ? 0x8u : 0u));
      const uint32_t cmask = to_smem ? (vmask & cstatic) : 0u;
      int flo = -(1 << 30), fhi = 1 << 30;  // rows stored in full: r <= flo or r >= fhi
      if (a == g.a_final || a == g.L - 1) flo = 1 << 30, fhi = -(1 << 30);
      else if (a == g.H) flo = rlo, fhi = rhi;
      else if (a > g.H) flo = rlo + 1, fhi = rhi - 1;
      T* gp = static_cast<T*>(g.buf[(g.tau0 + a + 1) & 1]) + (i0 + rlo) * plane + (int64_t)y * N2 + xb;
      const bool fast = __all_sync(0xffffffffu, vmask == 0xFu && i0 + rlo >= 1 && i0 + rhi <= N0 - 2);

      auto sweep = [&](auto fast_c) {
        constexpr bool FAST = decltype(fast_c)::value;
        auto step = [&](int r, const Win<T>& Wp, const Win<T>& Wc, const Win<T>& Wx) {
          uint32_t okm = vmask;
          if constexpr (!FAST) {
            const int64_t z = i0 + r;
            if (z < 1 || z > N0 - 2) okm = 0u;
          }
          T out[4];
#pragma unroll
          for (int j = 0; j < 4; ++j) {
            T x[3][3][3];
#pragma unroll
            for (int dy = 0; dy < 3; ++dy)
#pragma unroll
              for (int dx = 0; dx < 3; ++dx) {
                x[0][dy][dx] = Wp.v[dy][j + dx];
                x[1][dy][dx] = Wc.v[dy][j + dx];
                x[2][dy][dx] = Wx.v[dy][j + dx];
              }
            const T v = apply<T, KIND>(x, cf);
            if constexpr (FAST) out[j] = v;
            else out[j] = ((okm >> j) & 1u) ? v : x[1][1][1];
          }
          if (to_smem) {
            T* p = Wn + (size_t)(r - rlo) * LY::MAIN;
            if constexpr (sizeof(T) == 4) {
              reinterpret_cast<float4*>(p)[0] = make_float4(out[0], out[1], out[2], out[3]);
            } else {
              reinterpret_cast<double2*>(p)[0] = make_double2(out[0], out[1]);
              reinterpret_cast<double2*>(p)[1] = make_double2(out[2], out[3]);
            }
          }
          const uint32_t sm_ = (r <= flo || r >= fhi) ? okm : (okm & cmask);
          if (sm_ == 0xFu) {
            if constexpr (sizeof(T) == 4) {
              reinterpret_cast<float4*>(gp)[0] = make_float4(out[0], out[1], out[2], out[3]);
            } else {
              reinterpret_cast<double2*>(gp)[0] = make_double2(out[0], out[1]);
              reinterpret_cast<double2*>(gp)[1] = make_double2(out[2], out[3]);
            }
          } else if (sm_) {
#pragma unroll
            for (int j = 0; j < 4; ++j)
              if ((sm_ >> j) & 1u) gp[j] = out[j];
          }
          gp += plane;
        };
        const T* Pr[3] = {P[0], P[1], P[2]};
        auto adv = [&]() {
#pragma unroll
          for (int k = 0; k < 3; ++k) Pr[k] += pitch[k];
        };
        Win<T> wa, wb, wc;
        load_win<T, KIND == K_BOX3D27>(wa, Pr, q);  // row rlo - 1
        adv();
        load_win<T, KIND == K_BOX3D27>(wb, Pr, q);  // row rlo
        adv();
        int r = rlo;
        while (true) {
          load_win<T, KIND == K_BOX3D27>(wc, Pr, q);
          adv();
          step(r, wa, wb, wc);
          if (++r > rhi) break;
          load_win<T, KIND == K_BOX3D27>(wa, Pr, q);
          adv();
          step(r, wb, wc, wa);
          if (++r > rhi) break;
          load_win<T, KIND == K_BOX3D27>(wb, Pr, q);
          adv();
          step(r, wc, wa, wb);
          if (++r > rhi) break;
        }
      };
      if (fast) sweep(std::true_type{});
      else sweep(std::false_type{});
    }
    __syncthreads();  // the tile's stores are issued by every thread; item_s[cur^1] visible
    if (tid == 0) {
      st_release(my_flag, 1);
      if (!early && item_s[cur ^ 1][0] >= 0) issue_level(item_s[cur ^ 1], g.a_lo, true);
    }
    cur ^= 1;
  }
}

static PFN_cuTensorMapEncodeTiled_v12000 get_encode() {
  static PFN_cuTensorMapEncodeTiled_v12000 fn = nullptr;
  if (!fn) {
    cudaDriverEntryPointQueryResult q;
    void* p = nullptr;
    if (cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &p, cudaEnableDefault, &q) == cudaSuccess &&
        q == cudaDriverEntryPointSuccess)
      fn = reinterpret_cast<PFN_cuTensorMapEncodeTiled_v12000>(p);
  }
  return fn;
}

template <typename T>
static bool encode(CUtensorMap* map, void* base, const Fast3DArgs& a, uint32_t bx, uint32_t by, uint32_t bz) {
  auto fn = get_encode();
  if (!fn) return false;
  cuuint64_t dims[3] = {(cuuint64_t)a.N2, (cuuint64_t)a.N1, (cuuint64_t)a.N0};
  cuuint64_t strides[2] = {(cuuint64_t)a.N2 * sizeof(T), (cuuint64_t)a.N1 * a.N2 * sizeof(T)};
  cuuint32_t box[3] = {bx, by, bz};
  cuuint32_t es[3] = {1, 1, 1};
  const CUtensorMapDataType dt = sizeof(T) == 4 ? CU_TENSOR_MAP_DATA_TYPE_FLOAT32 : CU_TENSOR_MAP_DATA_TYPE_FLOAT64;
  return fn(map, dt, 3, base, dims, strides, box, es, CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE,
            CU_TENSOR_MAP_L2_PROMOTION_L2_128B, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE) == CUDA_SUCCESS;
}

template <typename T, int KIND>
cudaError_t launch_t(const Fast3DArgs& a, cudaStream_t s) {
  static int grid = 0;
  static size_t attr_bytes = 0;
  const size_t smem = smem_bytes<T>(a.Q);
  if (smem > attr_bytes) {
    cudaError_t e = cudaFuncSetAttribute(fast3d_kernel<T, KIND>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    if (e != cudaSuccess) return e;
    attr_bytes = smem;
    grid = 0;
  }
  if (grid == 0) {
    int dev = 0, sms = 0, per_sm = 0;
    cudaGetDevice(&dev);
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
    cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, fast3d_kernel<T, KIND>, NT<T>, smem);
    grid = sms * (per_sm > 0 ? per_sm : 1);
  }
  Maps m;
  const uint32_t Q = (uint32_t)a.Q, ny = (uint32_t)NY<T>;
  for (int b = 0; b < 2; ++b) {
    if (!encode<T>(&m.main[b], a.buf[b], a, NX, ny, Q) || !encode<T>(&m.lines[b], a.buf[b], a, NX, 2, Q) ||
        !encode<T>(&m.carry[b], a.buf[b], a, CC, ny + 2, Q) || !encode<T>(&m.in2[b], a.buf[b], a, NX, ny, 2) ||
        !encode<T>(&m.in1[b], a.buf[b], a, NX, ny, 1))
      return cudaErrorInvalidValue;
  }
  const int64_t items = (a.S0_hi - a.S0_lo + 1) * a.n1 * a.n2;
  const int gsz = (int)(items < grid ? items : grid);
  fast3d_kernel<T, KIND><<<gsz, NT<T>, smem, s>>>(a, m);
  return cudaGetLastError();
}

}  // namespace fast3d

size_t fast3d_smem_bytes(int dtype, int Q) {
  return dtype == 1 ? fast3d::smem_bytes<double>(Q) : fast3d::smem_bytes<float>(Q);
}
int fast3d_tile_lines(int dtype) { return dtype == 1 ? fast3d::NY<double> : fast3d::NY<float>; }

// variant id = kind * 2 + dtype for the 3D classes
cudaError_t launch_fast3d(int variant, const Fast3DArgs& a, int /*grid: persistent*/, cudaStream_t s) {
  switch (variant) {
    case K_STAR3D7 * 2: return fast3d::launch_t<float, K_STAR3D7>(a, s);
    case K_STAR3D7 * 2 + 1: return fast3d::launch_t<double, K_STAR3D7>(a, s);
    case K_GRADIENT3D * 2: return fast3d::launch_t<float, K_GRADIENT3D>(a, s);
    case K_GRADIENT3D * 2 + 1: return fast3d::launch_t<double, K_GRADIENT3D>(a, s);
    case K_BOX3D27 * 2: return fast3d::launch_t<float, K_BOX3D27>(a, s);
    case K_BOX3D27 * 2 + 1: return fast3d::launch_t<double, K_BOX3D27>(a, s);
    default: return cudaErrorInvalidValue;
  }
}

}  // namespace hexs
