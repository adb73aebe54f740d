// hex3d.cu -- the specialised sm_100a phase kernel for 3D single-field stencils of radius 1
// (star3d7, gradient3d, box3d27) under the hybrid schedule: hexagonal over (t, z), classical
// parallelogram tiles over y and x (eq. (14)).  Compiled once per
// (class, dtype, h, w0) of fast3d_variants.h (-DHEXS_F3_VARIANT=id).
//
// Mapping:
//   * work item = one classical tile (S1, S2) of one hexagon S0 of the launch's (T, p): an
//     NY x NX (y, x) parallelogram over the hexagon's 2h+2 levels and its rows z.  Skews: y
//     by 1 per level (delta1_y = 1), x by 4 per level (any integer skew >= delta1_x keeps
//     eq. (14) valid, reading R16) so every x-window this kernel moves is 16-B aligned;
//   * the hexagon shape is a template parameter: every level's row range [lo(a), hi(a)] is a
//     compile-time constant and each level's row sweep is fully unrolled (the paper's
//     constraint-based unrolling); nothing in the sweep depends on the
//     tile's position -- Dirichlet cells are repaired after the sweep in the few tiles that
//     touch the domain edge, and stores carry a per-row predicate from a 32-bit row mask;
//   * the tile keeps ALL its levels on chip: level a reads a shared-memory buffer holding
//     level a-1 (rows x (NY+2) lines x (NX+5) columns) and writes the other buffer;
//   * tile-granular dependences: the skew makes every dependence point to a tile with
//     component-wise larger-or-equal (S1, S2), so a tile whose predecessors (S1-1, S2) and
//     (S1, S2-1) have COMPLETED finds every value it reads, at every level, in global memory.
//     Persistent CTAs take tiles in anti-diagonal order (S1 + S2, then S0, then S1), wait for
//     the two predecessor flags once, and publish their own flag once (st.release.gpu);
//   * everything a tile reads from L2/HBM arrives by 3-D TMA tensor copies (SASS UTMALDG)
//     completing on one mbarrier per buffer: the first level's whole buffer (issued during the
//     previous tile's last level, which writes no shared memory), the In rows of every later
//     level (the hexagon's slanted-edge inputs) two levels ahead, into rows
//     the level in between neither reads nor writes, and per level the carries the
//     predecessor tiles produced: 2 lines above and 5 columns left;
//   * a thread owns one line and 4 consecutive x of the tile and sweeps z with a 3-row
//     register window (z neighbours from registers, y neighbours from the level buffer, x
//     edges by shuffle inside 8-lane groups);
//   * results leave from registers: the Out rows (slanted upper edges and top row), every
//     value of level T_steps, and the tile's last 2 lines / last 2 quads of every level
//     (its successors' carries) -- interleaved copy-out.
#include <cuda.h>
#include <cudaTypedefs.h>

#include <cstdint>
#include <type_traits>
#include <utility>

#include "../stencil_ops.cuh"
#include "fast3d_variants.h"
#include "devcache.h"
#include "launch.h"
#include "tma.cuh"

#ifndef HEXS_F3_UNROLL
#define HEXS_F3_UNROLL 1  // 0: rolled star sweeps (smaller code; measured equal or slower)
#endif
#ifndef HEXS_F3_EARLY_IN
#define HEXS_F3_EARLY_IN 0  // 1: In rows of a tile's levels issued at its start (even) / with level 1 (odd):
                            // measured neutral (heat-3D 592 vs 597, 27-point 367 vs 370), parity green
#endif
#ifndef HEXS_F3_LEAD
#define HEXS_F3_LEAD 1  // window rows loaded ahead of the shuffled row (2, 3 measured 544, 545 vs 551)
#endif
#ifndef HEXS_F3_VARIANT
#error "hex3d.cu is compiled once per fast3d variant: -DHEXS_F3_VARIANT=<id>"
#endif

namespace hexs {
namespace fast3d {

// tile columns (x) of the instantiation this object carries (fast3d_variants.h)
template <int ID> struct VariantNX;
#define HEXS_F3_NXOF(id, dc, T_, KIND_, H_, W0_, NY_, MINB_, ZS_, NX_) \
  template <> struct VariantNX<id> { static constexpr int value = NX_; };
HEXS_FAST3D_VARIANTS(HEXS_F3_NXOF)
#undef HEXS_F3_NXOF
constexpr int NX = VariantNX<HEXS_F3_VARIANT>::value;
constexpr int NXP = NX + 4;    // shared-memory line pitch (spreads the per-line edge loads over banks)
constexpr int NQ = NX / 4;     // column quads: one 8-lane group
constexpr int SIGMA = 4;       // x skew per level
// Carry areas (the predecessor tiles' values): the carry-column quad (main-frame m = -4 .. -1)
// and the edge column (m = -5, element 3 of its quad) in areas of 16-B lines, and 2 carry lines.
// The carry-quad and edge boxes start SC lines early and their rows are padded to 8-chunk multiples, so
// that lane 0's carry quad lands in the one 16-B bank slot its 8-lane group leaves free in the
// same LDS.128 (conflict-free; a TMA destination itself must stay 128-B aligned).
// (fp32 bank geometry; the fp64 variants keep the dense 2-line / NY+2-line areas)
template <typename T> constexpr int SC = sizeof(T) == 4 ? 5 : 0;  // line shift of the carry boxes
template <typename T> constexpr int SL = 0;  // line shift of the carry-line box
template <typename T> constexpr int LR = 2;  // lines per row, carry-line area (its 2 of NY+2 lines may conflict)
template <typename T> constexpr int CLP = sizeof(T) == 4 ? 8 : 2; // extra lines per row, carry areas

// Hexagon of a radius-1 single-statement stencil (delta0 = delta1 = 1): rows b of level a
// (SURVEY §8(a) closed form of eqs. (6)-(13)); buffer rows b = -1 .. 2h + w0 + 1.
template <int H, int W0> struct Hex {
  static constexpr int L = 2 * H + 2, Q = W0 + 2 * H + 3;
  __host__ __device__ static constexpr int lo(int a) { return a <= H ? H - a : a - H - 1; }
  __host__ __device__ static constexpr int hi(int a) { return a <= H ? H + W0 + a : 3 * H + 1 + W0 - a; }
  // rows of level a that tiles of the next phase read (the slanted upper edges of the Out set)
  __host__ __device__ static constexpr bool out_row(int a, int r) {
    return a == H ? (r == lo(a) || r == hi(a)) : (a > H ? (r <= lo(a) + 1 || r >= hi(a) - 1) : false);
  }
};

constexpr int al128(int bytes) { return (bytes + 127) / 128 * 128; }
// One buffer (level a's input = level a-1 values), Q rows (buffer row rr = b + 1), input-frame
// line L' = 0 .. NY+1 (y = Y0 - a - 1 + L'):
//   main  [Q][NY][NXP]   own region: lines L' = 2 + l, x = X0 - 4a + 4 + m
//   lines [Q][LR][NXP]   carry lines: L' = l - SL (l = SL, SL+1), x as main
//   carry [Q][CL][4]     carry quad: L' = l - SC, x = X0 - 4a + c      (m = c - 4)
//   edge  [Q][CL][4]     edge column: L' = l - SC, x = X0 - 4a - 4 + c (c = 3: m = -5)
// Each area starts 128-B aligned (TMA destinations).  Offsets in elements.
template <typename T, int Q, int NY> struct Lay {
  static constexpr int CL = NY + CLP<T>;  // lines per row of the carry / edge areas (>= NY + 2 + SC)
  static constexpr int MAIN = NY * NXP, LINES = LR<T> * NXP, CARRY = CL * 4;
  static constexpr int LINES_OFF = al128(Q * MAIN * (int)sizeof(T)) / (int)sizeof(T);
  static constexpr int CARRY_OFF = al128((LINES_OFF + Q * LINES) * (int)sizeof(T)) / (int)sizeof(T);
  static constexpr int EDGE_OFF = al128((CARRY_OFF + Q * CARRY) * (int)sizeof(T)) / (int)sizeof(T);
  static constexpr int BUF = al128((EDGE_OFF + Q * CARRY) * (int)sizeof(T)) / (int)sizeof(T);
  static constexpr size_t SMEM = 2 * (size_t)BUF * sizeof(T);
  static_assert(SMEM + 1024 <= 227 * 1024, "two level buffers must fit the 227 KB opt-in shared memory");
  static constexpr uint32_t FIRST_BYTES = (uint32_t)(Q * (MAIN + LINES + 2 * CARRY) * sizeof(T));
  static constexpr uint32_t CARRY_BYTES = (uint32_t)(Q * (LINES + 2 * CARRY) * sizeof(T));
  static constexpr uint32_t ROW_BYTES = (uint32_t)(MAIN * sizeof(T));
};

struct Maps {
  CUtensorMap main[2];   // box {NXP, NY, Q}
  CUtensorMap main0[2];  // box {NXP, NY, W0+3}: the rows level 0 reads (full-time tiles)
  CUtensorMap lines[2];  // box {NXP, LR, Q}
  CUtensorMap carry[2];  // box {4, NY+8, Q} (carry quads and edge columns)
  CUtensorMap in2[2];    // box {NXP, NY, 2}
  CUtensorMap in1[2];    // box {NXP, NY, 1}
};

__device__ __forceinline__ int ld_acquire(const int* p) {
  int v;
  asm volatile("ld.acquire.gpu.global.b32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ int ld_relaxed(const int* p) {
  int v;
  asm volatile("ld.relaxed.gpu.global.b32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
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

// fp32 star sweeps evaluate two x columns per instruction (F2: FADD2 / FFMA2,
// stencil_ops.cuh); gradient (sqrt / div) and 27-point (9 shifted lines: more moves and
// spills than FP instructions saved, SASS-checked) stay scalar.  HEXS_F2=0: scalar.
#ifndef HEXS_F2
#define HEXS_F2 0  // 1 measured neutral on heat-3D 512^3 (552 vs 552 GUp/s): the sweep is not FP-issue bound
#endif
template <typename T, int KIND>
constexpr bool kPacked3 = HEXS_F2 && std::is_same<T, float>::value && KIND == K_STAR3D7;

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

// Two phases, so a row's shared-memory latency hides behind the previous rows' arithmetic:
// load_win issues the loads (vector quads; the group's outer lanes also load their edge
// column with a predicated scalar load), edges_win completes the edges by shuffle.
template <typename T, bool ALL_EDGES>  // star / gradient stencils need the centre line's edges only
__device__ __forceinline__ void load_win(Win<T>& w, const T* const (&p)[3], int q, int eo) {
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
    if (ALL_EDGES || l == 1) {
      w.v[l][0] = lds_if(q == 0, p[l] + eo, T(0));  // lane 0: the edge area
      w.v[l][5] = lds_if(q == NQ - 1, p[l] + 4, T(0));
    } else {
      w.v[l][0] = w.v[l][5] = T(0);  // never used by this stencil
    }
  }
}
// star / gradient: the shuffles of a row are issued one row before their selects, so the
// shuffle latency hides behind a row of arithmetic (only the centre row's centre line needs
// x edges: the z neighbours are centre columns)
template <typename T> struct Edge { T l, r; };
template <typename T>
__device__ __forceinline__ Edge<T> edges_shfl(const Win<T>& w) {
  return {__shfl_up_sync(0xffffffffu, w.v[1][4], 1, NQ), __shfl_down_sync(0xffffffffu, w.v[1][1], 1, NQ)};
}
template <typename T>
__device__ __forceinline__ void edges_sel(Win<T>& w, const Edge<T>& e, int q) {
  w.v[1][0] = q != 0 ? e.l : w.v[1][0];
  w.v[1][5] = q != NQ - 1 ? e.r : w.v[1][5];
}
template <typename T, bool ALL_EDGES>
__device__ __forceinline__ void edges_win(Win<T>& w, int q) {
#pragma unroll
  for (int l = 0; l < 3; ++l) {
    if (ALL_EDGES || l == 1) {
      const T lft = __shfl_up_sync(0xffffffffu, w.v[l][4], 1, NQ);
      const T rgt = __shfl_down_sync(0xffffffffu, w.v[l][1], 1, NQ);
      w.v[l][0] = q != 0 ? lft : w.v[l][0];
      w.v[l][5] = q != NQ - 1 ? rgt : w.v[l][5];
    }
  }
}

// Optional per-CTA cycle accounting (debug builds: -DHEXS_F3_TIMING): thread 0 (the TMA
// issuer) and thread 64 (a compute-only warp) add the cycles spent per category.
#ifdef HEXS_F3_TIMING
__device__ unsigned long long g_f3_tm[1024][2][8];
#define F3_TM_DECL long long tm_t = clock64();
#define F3_TM(k)                                                                     \
  do {                                                                               \
    if (threadIdx.x == NC || threadIdx.x == 64) {                                    \
      const long long now = clock64();                                               \
      atomicAdd(&g_f3_tm[blockIdx.x][threadIdx.x == NC ? 0 : 1][k], (unsigned long long)(now - tm_t)); \
      tm_t = now;                                                                    \
    }                                                                                \
  } while (0)
#else
#define F3_TM_DECL
#define F3_TM(k) \
  do {           \
  } while (0)
#endif

__device__ __forceinline__ void named_barrier_sync(int id, int nthreads) {
  asm volatile("bar.sync %0, %1;" ::"r"(id), "r"(nthreads) : "memory");
}

// Optional event trace (debug builds: -DHEXS_F3_TRACE): CTAs 0..7 record (type, tile, level,
// clock64) for the producer lane and compute thread 0; tools/f3_trace.py prints the timeline.
#ifdef HEXS_F3_TRACE
constexpr int kTrCtas = 8, kTrEv = 8192;
__device__ unsigned long long g_f3_tr[kTrCtas][kTrEv];
__device__ int g_f3_trn[kTrCtas];
__device__ __forceinline__ void f3_trace(int type, int tile, int level) {
  if (blockIdx.x < kTrCtas) {
    const int i = atomicAdd(&g_f3_trn[blockIdx.x], 1);
    if (i < kTrEv)
      g_f3_tr[blockIdx.x][i] = ((unsigned long long)type << 60) | ((unsigned long long)(tile & 0xFFFF) << 44) |
                               ((unsigned long long)(level & 0xFF) << 36) | ((unsigned long long)clock64() & 0xFFFFFFFFFull);
  }
}
#define F3_TR(type, tile, level) f3_trace(type, tile, level)
#else
#define F3_TR(type, tile, level) \
  do {                            \
  } while (0)
#endif

template <int... As, typename F>
__device__ __forceinline__ void for_levels(F&& f, std::integer_sequence<int, As...>) {
  (f(std::integral_constant<int, As>{}), ...);
}

// NY tile lines (y); ZS threads per (line, quad), each sweeping 1/ZS of a level's rows;
// MINB CTAs per SM; plus one producer warp
// MIR: the fused halo stores of the multi-GPU slab mode (a separate instantiation, so the
// single-GPU kernel keeps its register budget)
template <typename T, int KIND, int H, int W0, int NY, int MINB, int ZS, bool MIR>
__global__ void __launch_bounds__(ZS * NY * NQ + 32, MINB) fast3d_kernel(const __grid_constant__ Fast3DArgs g,
                                                                   const __grid_constant__ Maps mp) {
  using HX = Hex<H, W0>;
  constexpr int LNY = NY, Q = HX::Q, L = HX::L;
  using LY = Lay<T, Q, NY>;
  extern __shared__ __align__(1024) unsigned char smem_raw[];  // dynamic base: 1024-B aligned
  T* const sbase = reinterpret_cast<T*>(smem_raw);  // stays a shared-space pointer (LDS/STS)
  constexpr int NC = ZS * NY * NQ, NCW = NC / 32;  // compute threads / warps; warp NCW produces
  __shared__ __align__(8) uint64_t full[2];   // buffer filled (producer arrival + TMA bytes)
  __shared__ __align__(8) uint64_t empty[2];  // buffer consumed (one arrival per compute warp)
  __shared__ __align__(8) uint64_t inbar[2 * H + 2];  // early In rows of level a (full-time launches)
  __shared__ long long item_s[2][3];          // tile ring (S0, q1, q2); S0 < 0: no more work
  const int tid = threadIdx.x;
  const int zpart = tid / (NY * NQ);                             // row part (< ZS; producer: ZS)
  const int ly = (tid % (NY * NQ)) / NQ, q = tid % NQ;           // line, column quad
  const int64_t n1 = g.n1, n2 = g.n2, ns0 = g.S0_hi - g.S0_lo + 1, n_items = ns0 * n1 * n2;
  const int64_t N0 = g.N0, N1 = g.N1, N2 = g.N2, plane = N1 * N2;
  const int a_lo = g.a_lo, a_hi = g.a_hi;
  // In rows issued early (full-time launches; HEXS_F3_EARLY_IN=0 at build time: with the carries)
  const bool early_in = HEXS_F3_EARLY_IN && a_lo == 0 && a_hi == 2 * H + 1;

  // per-thread window lines k = 0..2 (input-frame line ly + k): element offset in a buffer
  // at buffer row 0, and the row pitch of the area they live in
  int woff[3], wpitch[3];
#pragma unroll
  for (int k = 0; k < 3; ++k) {
    const int l = ly + k;
    if (q == 0) {
      woff[k] = LY::CARRY_OFF + (l + SC<T>) * 4;
      wpitch[k] = LY::CARRY;
    } else if (l < 2) {
      woff[k] = LY::LINES_OFF + (l + SL<T>) * NXP + 4 * q - 4;
      wpitch[k] = LY::LINES;
    } else {
      woff[k] = (l - 2) * NXP + 4 * q - 4;
      wpitch[k] = LY::MAIN;
    }
  }
  const int eo = q == 0 ? LY::EDGE_OFF - LY::CARRY_OFF + 3 : -1;  // left edge relative to the quad
  const int sts_off = ly * NXP + 4 * q;                  // + row * MAIN in the output buffer
  const bool cthr = (ly >= LNY - 2) || (q >= NQ - 2);   // writes its successors' carries

  // chained launches: the next launch may be scheduled as soon as every CTA of this one runs
  if (g.pdl) asm volatile("griddepcontrol.launch_dependents;" ::: "memory");
  if (tid == 0) {
    mbar_init(&full[0], 1);
    mbar_init(&full[1], 1);
    mbar_init(&empty[0], NCW);
    mbar_init(&empty[1], NCW);
    for (int a = 0; a < 2 * H + 2; ++a) mbar_init(&inbar[a], 1);
    mbar_fence_init();
  }
  __syncthreads();
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
  auto buf_of = [&](int b) { return sbase + b * LY::BUF; };
  // ---- TMA issue (thread 0 only) ----
  // the whole input buffer of level a (first level of a tile): no dependence on predecessors
  auto issue_first = [&](const long long* it, int a) {
    int64_t i0;
    int X0, Y0;
    tile_origin(it, i0, X0, Y0);
    const int b = a & 1, par = (int)((g.tau0 + a) & 1);
    const int z0 = (int)(i0 - 1), xo = X0 - SIGMA * a, yo = Y0 - a;
    T* B = buf_of(b);
    if (a == 0) {  // only the rows level 0 reads: [lo(0)-1, hi(0)+1] (W0+3 of the Q rows)
      constexpr uint32_t FB0 =
          (uint32_t)(((HX::hi(0) - HX::lo(0) + 3) * LY::MAIN + Q * (LY::LINES + 2 * LY::CARRY)) * sizeof(T));
      mbar_arrive_expect_tx(&full[b], FB0);
      tma_3d(B + HX::lo(0) * LY::MAIN, &mp.main0[par], xo + 4, yo + 1, (int)(i0 + HX::lo(0) - 1), &full[b]);
    } else {
      mbar_arrive_expect_tx(&full[b], LY::FIRST_BYTES);
      tma_3d(B, &mp.main[par], xo + 4, yo + 1, z0, &full[b]);
    }
    tma_3d(B + LY::LINES_OFF, &mp.lines[par], xo + 4, yo - 1 - SL<T>, z0, &full[b]);
    tma_3d(B + LY::CARRY_OFF, &mp.carry[par], xo, yo - 1 - SC<T>, z0, &full[b]);
    tma_3d(B + LY::EDGE_OFF, &mp.carry[par], xo - 4, yo - 1 - SC<T>, z0, &full[b]);
  };
  // In rows of level a: buffer rows level a reads ([lo(a)-1, hi(a)+1]) that level a-1 does
  // not compute (0, 1 or 2 per side)
  auto in_rows = [&](int a, int* lo2, int* n2_) {
    const int need_lo = HX::lo(a) - 1, need_hi = HX::hi(a) + 1, clo = HX::lo(a - 1), chi = HX::hi(a - 1);
    lo2[0] = need_lo; n2_[0] = need_lo < clo ? clo - need_lo : 0;
    lo2[1] = chi + 1; n2_[1] = need_hi > chi ? need_hi - chi : 0;
  };
  auto issue_in = [&](const long long* it, int a, uint64_t* bar) {
    int64_t i0;
    int X0, Y0;
    tile_origin(it, i0, X0, Y0);
    const int b = a & 1, par = (int)((g.tau0 + a) & 1);
    const int xo = X0 - SIGMA * a, yo = Y0 - a;
    int lo2[2], nn[2];
    in_rows(a, lo2, nn);
    for (int s = 0; s < 2; ++s)
      for (int k = 0; k < nn[s];) {
        const int bb = lo2[s] + k;
        T* dst = buf_of(b) + (bb + 1) * LY::MAIN;
        if (nn[s] - k >= 2) {
          tma_3d(dst, &mp.in2[par], xo + 4, yo + 1, (int)(i0 + bb), bar);
          k += 2;
        } else {
          tma_3d(dst, &mp.in1[par], xo + 4, yo + 1, (int)(i0 + bb), bar);
          k += 1;
        }
      }
  };
  auto in_bytes = [&](int a) {
    int lo2[2], nn[2];
    in_rows(a, lo2, nn);
    return (uint32_t)(nn[0] + nn[1]) * LY::ROW_BYTES;
  };
  auto issue_carries = [&](const long long* it, int a) {
    int64_t i0;
    int X0, Y0;
    tile_origin(it, i0, X0, Y0);
    const int b = a & 1, par = (int)((g.tau0 + a) & 1);
    const int z0 = (int)(i0 - 1), xo = X0 - SIGMA * a, yo = Y0 - a;
    tma_3d(buf_of(b) + LY::LINES_OFF, &mp.lines[par], xo + 4, yo - 1 - SL<T>, z0, &full[b]);
    tma_3d(buf_of(b) + LY::CARRY_OFF, &mp.carry[par], xo, yo - 1 - SC<T>, z0, &full[b]);
    tma_3d(buf_of(b) + LY::EDGE_OFF, &mp.carry[par], xo - 4, yo - 1 - SC<T>, z0, &full[b]);
  };

  // Chained mode: a tile reads, at every level a, z rows [i0 - 1, i0 + Q - 2], y lines
  // [Y0 - a - 1, Y0 - a + NY] and x [X0 - 4a - 1, X0 - 4a + NX] of time tau0 + a.  A writer
  // launch with base time tau0' computed that time at its level a' = a + D, D = tau0 - tau0' - 1,
  // where its tile (S1', S2') covers y [S1' NY - a', S1' NY - a' + NY - 1] and x
  // [S2' NX - 4a', S2' NX - 4a' + NX - 1]; intersecting gives a range of S1' / S2' that does not
  // depend on a, and hexagon S0' covers rows [S0' W - row_off', S0' W - row_off' + Q - 3].
  // Every such writer tile that exists is acquired (a superset of the true producers).
  auto fdiv = [](int64_t x, int64_t y) { return x >= 0 ? x / y : -((-x + y - 1) / y); };
  // (producer lane) launches seen complete need no more polls: their completed-tile counter
  // reached their tile count once, and the fence after that observation is the acquire
  bool prev_done[2] = {g.prev[0].flags == nullptr, g.prev[1].flags == nullptr};
  auto wait_prev = [&](const long long* it) {
    if (prev_done[0] && prev_done[1]) return;
    bool fresh = false;
    for (int k = 0; k < 2; ++k) {
      const Fast3DPrev& pv = g.prev[k];
      if (prev_done[k]) continue;
      unsigned long long d;
      asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(d) : "l"(pv.done) : "memory");
      if (d == (unsigned long long)((pv.S0_hi - pv.S0_lo + 1) * pv.n1 * pv.n2)) prev_done[k] = fresh = true;
    }
    if (prev_done[0] && prev_done[1]) {
      if (fresh) __threadfence();
      return;
    }
    int64_t i0;
    int X0, Y0;
    tile_origin(it, i0, X0, Y0);
    const int64_t S1r = Y0 / LNY, S2r = X0 / NX;
    for (int k = 0; k < 2; ++k) {
      const Fast3DPrev& pv = g.prev[k];
      if (prev_done[k]) continue;
      const int64_t D = g.tau0 - pv.tau0 - 1;
      const int64_t zlo = i0 - 1, zhi = i0 + g.Q - 2;
      int64_t s0a = -fdiv(-(zlo - (g.Q - 3) + pv.row_off), g.W), s0b = fdiv(zhi + pv.row_off, g.W);
      int64_t s1a = -fdiv(-(S1r * LNY - LNY + D), LNY), s1b = fdiv(S1r * LNY + LNY + D, LNY);
      int64_t s2a = -fdiv(-(S2r * NX - NX + SIGMA * D), NX), s2b = fdiv(S2r * NX + NX + SIGMA * D, NX);
      s0a = s0a < pv.S0_lo ? pv.S0_lo : s0a;
      s0b = s0b > pv.S0_hi ? pv.S0_hi : s0b;
      s1a = s1a < pv.S1_lo ? pv.S1_lo : s1a;
      s1b = s1b > pv.S1_lo + pv.n1 - 1 ? pv.S1_lo + pv.n1 - 1 : s1b;
      s2a = s2a < pv.S2_lo ? pv.S2_lo : s2a;
      s2b = s2b > pv.S2_lo + pv.n2 - 1 ? pv.S2_lo + pv.n2 - 1 : s2b;
      // relaxed polls, all in flight at once (an acquire load per flag would serialise ~20 L2
      // round trips per tile); one fence after the last flag is seen gives the acquire
      bool all = false;
      while (!all) {
        all = true;
        for (int64_t s0 = s0a; s0 <= s0b; ++s0)
          for (int64_t s1 = s1a; s1 <= s1b; ++s1)
            for (int64_t s2 = s2a; s2 <= s2b; ++s2)
              all &= ld_relaxed(pv.flags + ((s0 - pv.S0_lo) * pv.n1 + (s1 - pv.S1_lo)) * pv.n2 + (s2 - pv.S2_lo)) != 0;
        if (!all) __nanosleep(128);
      }
    }
    __threadfence();  // acquire: the writers' stores (released with their flags) happen before our reads
  };

  F3_TM_DECL
  if (tid >= NC) {
    // ================= producer warp (one lane): tiles, predecessor flags, TMA =================
    // Fill k of a buffer waits for the level that consumed fill k-1 (empty[b] completion
    // k-1); fill(a_lo) = the whole first-level buffer, fill(a) = the In rows of level a and
    // the carries its predecessors produced at level a-1 (they are complete before
    // fill(a_lo + 1) is issued).
    if (tid == NC) {
      uint32_t fills[2] = {0u, 0u};
      int slot = 0, ptile = 0;
      while (true) {
        long long* it = item_s[slot];
        decode((int64_t)atomicAdd(g.counter, 1ull), it);
        if (it[0] < 0) {  // no more tiles: wake the compute warps with an empty fill
          const int b0 = a_lo & 1;
          if (fills[b0] > 0) mbar_wait_parity(&empty[b0], (fills[b0] - 1) & 1u);
          mbar_arrive(&full[b0]);
          break;
        }
        const int64_t base = (it[0] - g.S0_lo) * n1 * n2;
        for (int a = a_lo; a <= a_hi; ++a) {
          const int b = a & 1;
          F3_TR(1, ptile, a);
          if (fills[b] > 0) mbar_wait_parity(&empty[b], (fills[b] - 1) & 1u);
          F3_TM(0);
          fence_proxy_async_smem();
          if (a == a_lo) {
            if (g.prev[0].flags) {  // chained: the previous launches' writers of this tile's inputs
              F3_TR(3, ptile, a);
              wait_prev(it);
              fence_proxy_async_global();
              F3_TR(4, ptile, a);
            }
            issue_first(it, a);
            // early In rows (full-time launches): every even level's In rows land in buffer
            // b(0) rows no level before it reads or writes (the hexagon widens by one row per
            // side per level), so they go out with the first fill, on their own barriers
            if (early_in) {
              for (int a2 = 2; a2 <= H + 1; a2 += 2) {
                mbar_arrive_expect_tx(&inbar[a2], in_bytes(a2));
                issue_in(it, a2, &inbar[a2]);
              }
            }
          } else {
            if (a == a_lo + 1) {  // predecessors complete: their carries are in global memory
              F3_TR(3, ptile, a);
              // both predecessors polled together (relaxed loads in flight at once), then one
              // fence: the acquire of their carries
              const int* f = g.flags + base;
              const int* fy = it[1] > 0 ? f + (it[1] - 1) * n2 + it[2] : nullptr;
              const int* fx = it[2] > 0 ? f + it[1] * n2 + it[2] - 1 : nullptr;
              while (true) {
                const int vy = fy ? ld_relaxed(fy) : 1, vx = fx ? ld_relaxed(fx) : 1;
                if (vy != 0 && vx != 0) break;
                __nanosleep(64);
              }
              if (fy || fx) __threadfence();
              fence_proxy_async_global();
              F3_TR(4, ptile, a);
              F3_TM(2);
            }
            if (early_in) {
              // the odd levels' In rows go out once the previous tile's last level released
              // buffer b(1), i.e. with level 1's carries
              if (a == 1) {
                for (int a2 = 1; a2 <= H + 1; a2 += 2) {
                  mbar_arrive_expect_tx(&inbar[a2], in_bytes(a2));
                  issue_in(it, a2, &inbar[a2]);
                }
              }
              mbar_arrive_expect_tx(&full[b], LY::CARRY_BYTES);
            } else {
              mbar_arrive_expect_tx(&full[b], LY::CARRY_BYTES + (a <= H + 1 ? in_bytes(a) : 0u));
              if (a <= H + 1) issue_in(it, a, &full[b]);
            }
            issue_carries(it, a);
          }
          ++fills[b];
          F3_TR(2, ptile, a);
          F3_TM(4);
        }
        ++ptile;
        slot ^= 1;
      }
    }
    return;
  }

  // ================= compute warps =================
  uint32_t ph = 0u;  // parity bit per buffer
  const Coef<T> cf{(T)g.k0, (T)g.k1};
  [[maybe_unused]] Coef<F2> cf2;
  if constexpr (kPacked3<T, KIND>) cf2 = Coef<F2>{f2_pack((float)g.k0, (float)g.k0), f2_pack((float)g.k1, (float)g.k1)};
  const int lane = tid & 31;
  int slot = 0, ctile = 0;
  while (true) {
    {
      const int b0 = a_lo & 1;  // the tile's first fill publishes its item
      mbar_wait_parity(&full[b0], (ph >> b0) & 1u);
    }
    const long long* it = item_s[slot];
    if (it[0] < 0) break;
    int64_t i0;
    int X0, Y0;
    tile_origin(it, i0, X0, Y0);
    const int64_t base = (it[0] - g.S0_lo) * n1 * n2;
    int* const my_flag = g.flags + base + it[1] * n2 + it[2];
    // rows b of the hexagon whose z is an interior point (bit b); Dirichlet rows excluded
    uint32_t zmask = 0u;
#pragma unroll
    for (int b = 0; b <= 2 * H + W0; ++b) zmask |= (i0 + b >= 1 && i0 + b <= N0 - 2 ? 1u : 0u) << b;
    // a tile that never touches a domain edge needs no repair pass
    const bool edge = zmask != (2u << (2 * H + W0)) - 1u || Y0 - a_hi < 1 || Y0 - a_lo + LNY - 1 > N1 - 2 ||
                      X0 - SIGMA * a_hi < 1 || X0 - SIGMA * a_lo + NX - 1 > N2 - 2;
    F3_TM(3);

    bool mir_used = false;  // this thread stored into a neighbour's mirror during the tile
    for_levels(
        [&](auto ac) {
          constexpr int A = decltype(ac)::value;
          if (A < a_lo || A > a_hi) return;
          constexpr int b = A & 1, nb = b ^ 1;
          constexpr int LO = HX::lo(A), HI = HX::hi(A);
          // this thread's rows: N consecutive rows from R0 (the parts of an odd row count
          // share one row, computed twice with identical results)
          constexpr int N = (HI - LO + 1 + ZS - 1) / ZS;
          const int R0 = zpart == 0 ? LO : HI - N + 1;
          const int dR = R0 - LO;
          if (tid == 0) F3_TR(5, ctile, A);
          if (A != a_lo) mbar_wait_parity(&full[b], (ph >> b) & 1u);
          if (early_in && A >= 1 && A <= H + 1) mbar_wait_parity(&inbar[A], (uint32_t)(ctile & 1));
          ph ^= 1u << b;
          F3_TM(0);
          named_barrier_sync(1, NC);  // level A-1's buffer writes visible to every compute warp
          if (tid == 0) F3_TR(6, ctile, A);
          F3_TM(1);

          // ---- compute level A: line y = Y0 - A + ly, x = X0 - 4A + 4q + j, rows [LO, HI]
          const T* const B = buf_of(b);
          const T* P[3];
#pragma unroll
          for (int k = 0; k < 3; ++k) P[k] = B + woff[k] + R0 * wpitch[k];  // window row R0 - 1
          T* const Wn = buf_of(nb) + (R0 + 1) * LY::MAIN + sts_off;          // output row R0
          const int y = Y0 - A + ly;
          const int xb = X0 - SIGMA * A + 4 * q;
          const bool to_smem = A < a_hi;
          // whole-quad store validity (y interior, quad inside [0, N2)); the Dirichlet columns
          // x = 0 and x = N2-1 inside a valid quad keep their value by a select
          const bool vq = y >= 1 && y <= N1 - 2 && xb >= 0 && xb + 3 <= N2 - 1;
          const bool xl = xb == 0, xr = xb + 3 == N2 - 1;
          const bool st_all = A == g.a_final || A == L - 1;
          const uint32_t zm_out = vq ? zmask : 0u;
          const uint32_t zm_non = (vq && (st_all || (cthr && to_smem))) ? zmask : 0u;
          // per-row store predicate, bit i = row R0 + i (Out rows: slanted upper edges)
          constexpr uint32_t OMASK = [] {
            uint32_t m = 0u;
            for (int r = 0; r < 32; ++r) m |= (HX::out_row(A, r) ? 1u : 0u) << r;
            return m;
          }();
          const uint32_t zsel = ((OMASK & zm_out) | (~OMASK & zm_non)) >> R0;
          // store pointer of row LO, advanced one plane per row (a predicated store per row)
          T* gp = static_cast<T*>(g.buf[(g.tau0 + A + 1) & 1]) + (i0 + R0) * plane + (int64_t)y * N2 + xb;
          // fused halo stores (slab mode): a line of a neighbour's send zone is also stored into
          // that neighbour's mirror [parity][z][y - zone start][x] (peer memory); the zones are
          // disjoint (slabs of >= 2G lines), so a line has at most one mirror
          T* mpp = nullptr;
          int64_t mplane = 0;
          if constexpr (MIR) {
            mplane = (int64_t)g.mir_G * N2;
            const int side = (g.mir[0] && y >= g.mir_y0[0] && y < g.mir_y0[0] + g.mir_G)   ? 0
                             : (g.mir[1] && y >= g.mir_y0[1] && y < g.mir_y0[1] + g.mir_G) ? 1
                                                                                            : -1;
            if (side >= 0)
              mpp = static_cast<T*>(g.mir[side]) + ((int64_t)((g.tau0 + A + 1) & 1) * N0 + (i0 + R0)) * mplane +
                    (int64_t)(y - g.mir_y0[side]) * N2 + xb;
          }
          const bool mon = MIR && mpp != nullptr;  // (the pointer advances per row; the flag does not)
          if constexpr (MIR) mir_used |= mon;

          const T* Pr[3] = {P[0], P[1], P[2]};
          auto adv = [&]() {
#pragma unroll
            for (int k = 0; k < 3; ++k) Pr[k] += wpitch[k];
          };
          constexpr bool E27 = KIND == K_BOX3D27;
          // one output row i from the windows of rows i-1, i, i+1 (registers)
          auto step = [&](int i, const Win<T>& wm, const Win<T>& wc, const Win<T>& wp) {
            T out[4];
            if constexpr (kPacked3<T, KIND>) {
              // x columns (2p, 2p+1) as one F2 pair: the centre-column operands are the
              // LDS.128 quad's own register pairs, the x-shifted ones one move each
#pragma unroll
              for (int p = 0; p < 2; ++p) {
                F2 x[3][3][3];
#pragma unroll
                for (int dy = 0; dy < 3; ++dy)
#pragma unroll
                  for (int dx = 0; dx < 3; ++dx) {
                    x[0][dy][dx] = f2_pack(wm.v[dy][2 * p + dx], wm.v[dy][2 * p + dx + 1]);
                    x[1][dy][dx] = f2_pack(wc.v[dy][2 * p + dx], wc.v[dy][2 * p + dx + 1]);
                    x[2][dy][dx] = f2_pack(wp.v[dy][2 * p + dx], wp.v[dy][2 * p + dx + 1]);
                  }
                float o0, o1;
                f2_unpack(apply<F2, KIND>(x, cf2), o0, o1);
                out[2 * p] = o0;
                out[2 * p + 1] = o1;
              }
            } else {
#pragma unroll
            for (int j = 0; j < 4; ++j) {
              T x[3][3][3];
#pragma unroll
              for (int dy = 0; dy < 3; ++dy)
#pragma unroll
                for (int dx = 0; dx < 3; ++dx) {
                  x[0][dy][dx] = wm.v[dy][j + dx];
                  x[1][dy][dx] = wc.v[dy][j + dx];
                  x[2][dy][dx] = wp.v[dy][j + dx];
                }
              out[j] = apply<T, KIND>(x, cf);
            }
            }
            out[0] = xl ? wc.v[1][1] : out[0];
            out[3] = xr ? wc.v[1][4] : out[3];
            if (to_smem) {
              T* p = Wn + i * LY::MAIN;
              if constexpr (sizeof(T) == 4) {
                reinterpret_cast<float4*>(p)[0] = make_float4(out[0], out[1], out[2], out[3]);
              } else {
                reinterpret_cast<double2*>(p)[0] = make_double2(out[0], out[1]);
                reinterpret_cast<double2*>(p)[1] = make_double2(out[2], out[3]);
              }
            }
            if ((zsel >> i) & 1u) {
              auto st4 = [&](T* d) {
                if constexpr (sizeof(T) == 4) {
                  reinterpret_cast<float4*>(d)[0] = make_float4(out[0], out[1], out[2], out[3]);
                } else {
                  reinterpret_cast<double2*>(d)[0] = make_double2(out[0], out[1]);
                  reinterpret_cast<double2*>(d)[1] = make_double2(out[2], out[3]);
                }
              };
              st4(gp);
              if constexpr (MIR) {
                // the mirror is never read by this kernel: an asm store the compiler schedules
                // freely (no ordering against the level buffers' shared loads)
                if (mon) {
                  if constexpr (sizeof(T) == 4) {
                    asm volatile("st.global.v4.f32 [%0], {%1, %2, %3, %4};" ::"l"(mpp), "f"(out[0]), "f"(out[1]),
                                 "f"(out[2]), "f"(out[3]));
                  } else {
                    asm volatile("st.global.v2.f64 [%0], {%1, %2};" ::"l"(mpp), "d"(out[0]), "d"(out[1]));
                    asm volatile("st.global.v2.f64 [%0], {%1, %2};" ::"l"(mpp + 2), "d"(out[2]), "d"(out[3]));
                  }
                }
              }
            }
            gp += plane;
            if constexpr (MIR) mpp += mplane;
          };
          if constexpr (KIND == K_STAR3D7 && HEXS_F3_UNROLL && ZS == 1) {
            // short per-point expression: the whole sweep unrolled and software-pipelined
            // (loads of row i+3, edges of row i+2, arithmetic of row i+1)
            // row i+1 needs its edges before step(i); rows' shuffles run one row earlier
            // HEXS_F3_LEAD rows of loads in flight ahead of the row being shuffled
            constexpr int LD = HEXS_F3_LEAD;
            Win<T> w[N + 2];
#pragma unroll
            for (int r = 0; r < 3 + LD - 1 && r < N + 2; ++r) {
              load_win<T, E27>(w[r], Pr, q, eo);
              adv();
            }
            Edge<T> e1 = edges_shfl(w[1]);
            Edge<T> e2 = edges_shfl(w[2]);
#pragma unroll
            for (int i = 0; i < N; ++i) {
              if (i + 3 + LD - 1 < N + 2) {
                load_win<T, E27>(w[i + 3 + LD - 1], Pr, q, eo);
                adv();
              }
              edges_sel(w[i + 1], e1, q);
              e1 = e2;
              if (i + 3 < N + 2) e2 = edges_shfl(w[i + 3]);
              step(i, w[i], w[i + 1], w[i + 2]);
            }
          } else {
            // long per-point expressions (IEEE sqrt / div, 27 operands): a rolled sweep with a
            // 3-row register window keeps the level's code small enough for the i-cache
            Win<T> wa, wb, wc;
            auto ld = [&](Win<T>& w) {
              load_win<T, E27>(w, Pr, q, eo);
              adv();
              edges_win<T, E27>(w, q);
            };
            ld(wa);
            ld(wb);
#pragma unroll 1
            for (int i = 0; i < N; i += 3) {
              ld(wc);
              step(i, wa, wb, wc);
              if (i + 1 >= N) break;
              ld(wa);
              step(i + 1, wb, wc, wa);
              if (i + 2 >= N) break;
              ld(wb);
              step(i + 2, wc, wa, wb);
            }
          }
          // ---- Dirichlet repair (domain-edge tiles): cells on the boundary lines / rows keep
          // their value in the level buffer; it is the centre of their own stencil window
          if (edge && to_smem) {
            const bool yb = y == 0 || y == N1 - 1;
            for (int r = R0; r < R0 + N; ++r) {
              if (yb || !((zmask >> r) & 1u)) {
                const T* c = P[1] + (r - R0 + 1) * wpitch[1];
                T* o = Wn + (r - R0) * LY::MAIN;
#pragma unroll
                for (int j = 0; j < 4; ++j) o[j] = c[j];
              }
            }
          }
          // buffer b consumed (and this warp's generic writes of nb ordered before later TMA)
          fence_proxy_async_smem();
          __syncwarp();
          if (lane == 0) mbar_arrive(&empty[b]);
          if (tid == 0) F3_TR(7, ctile, A);
          F3_TM(3);
        },
        std::make_integer_sequence<int, L>{});
    if constexpr (MIR) {
      // fused halo stores: the threads that wrote into a mirror fence at system scope before the
      // barrier, so the tile's peer stores are ordered before its flag and a successor's later
      // store to the same mirror place lands last
      if (g.mir_fence && mir_used) __threadfence_system();
    }
    named_barrier_sync(1, NC);  // every compute thread's stores of the tile are issued
    F3_TM(1);
    if (tid == 0) {
      st_release(my_flag, 1);
      // chained mode: count the launch's completed tiles (release: after the tile's stores)
      if (g.done) asm volatile("red.release.gpu.global.add.u64 [%0], 1;" ::"l"(g.done) : "memory");
    }
    if (tid == 0) F3_TR(8, ctile, 0);
    ++ctile;
    slot ^= 1;
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

template <typename T, int KIND, int H, int W0, int NY, int MINB, int ZS, bool MIR>
cudaError_t launch_t(const Fast3DArgs& a, cudaStream_t s) {
  using LY = Lay<T, Hex<H, W0>::Q, NY>;
  constexpr int NT = ZS * NY * NQ + 32;  // compute threads + the producer warp
  static DeviceMemo<int> memo;  // per device: smem opt-in + persistent grid size
  constexpr size_t smem = LY::SMEM;
  auto kern = fast3d_kernel<T, KIND, H, W0, NY, MINB, ZS, MIR>;
  int grid = 0;
  cudaError_t e0 = memo.get(&grid, [&](int dev, int* gsz) {
    cudaError_t e = cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    if (e != cudaSuccess) return e;
    int sms = 0, per_sm = 0;
    e = cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
    if (e == cudaSuccess) e = cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, kern, NT, smem);
    *gsz = sms * (per_sm > 0 ? per_sm : 1);
    return e;
  });
  if (e0 != cudaSuccess) return e0;
  if (a.Q != Hex<H, W0>::Q || a.L != Hex<H, W0>::L) return cudaErrorInvalidValue;
  Maps m;
  const uint32_t Q = (uint32_t)a.Q, ny = (uint32_t)NY;
  for (int b = 0; b < 2; ++b) {
    if (!encode<T>(&m.main[b], a.buf[b], a, NXP, ny, Q) ||
        !encode<T>(&m.main0[b], a.buf[b], a, NXP, ny, (uint32_t)(W0 + 3)) || !encode<T>(&m.lines[b], a.buf[b], a, NXP, LR<T>, Q) ||
        !encode<T>(&m.carry[b], a.buf[b], a, 4, ny + CLP<T>, Q) || !encode<T>(&m.in2[b], a.buf[b], a, NXP, ny, 2) ||
        !encode<T>(&m.in1[b], a.buf[b], a, NXP, ny, 1))
      return cudaErrorInvalidValue;
  }
  const int64_t items = (a.S0_hi - a.S0_lo + 1) * a.n1 * a.n2;
  const int gsz = (int)(items < grid ? items : grid);
  if (a.pdl && a.prev[0].flags) {
    // chained launch: may start while the previous launch drains (its tiles wait on flags); the
    // run's first launch follows the flag reset (a memset) strictly
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = dim3((unsigned)gsz);
    cfg.blockDim = dim3((unsigned)NT);
    cfg.dynamicSmemBytes = smem;
    cfg.stream = s;
    cudaLaunchAttribute at[1];
    at[0].id = cudaLaunchAttributeProgrammaticStreamSerialization;
    at[0].val.programmaticStreamSerializationAllowed = 1;
    cfg.attrs = at;
    cfg.numAttrs = 1;
    return cudaLaunchKernelEx(&cfg, kern, a, m);
  }
  kern<<<gsz, NT, smem, s>>>(a, m);
  return cudaGetLastError();
}

}  // namespace fast3d

// the instantiation this object carries (fast3d_variants.h, -DHEXS_F3_VARIANT=<id>)
template <int ID> struct Sel3;
#define HEXS_F3_SEL(id, dc, T_, KIND_, H_, W0_, NY_, MINB_, ZS_, NX_)                         \
  template <> struct Sel3<id> {                                                          \
    using T = T_;                                                                        \
    static constexpr int KIND = KIND_, H = H_, W0 = W0_, NY = NY_, MINB = MINB_, ZS = ZS_; \
  };
HEXS_FAST3D_VARIANTS(HEXS_F3_SEL)
#undef HEXS_F3_SEL
#define HEXS_F3_CAT2(a, b) a##b
#define HEXS_F3_CAT(a, b) HEXS_F3_CAT2(a, b)
using S3 = Sel3<HEXS_F3_VARIANT>;

cudaError_t HEXS_F3_CAT(launch_fast3d_v, HEXS_F3_VARIANT)(const Fast3DArgs& a, cudaStream_t s) {
  if (a.mir[0] || a.mir[1])
    return fast3d::launch_t<S3::T, S3::KIND, S3::H, S3::W0, S3::NY, S3::MINB, S3::ZS, true>(a, s);
  return fast3d::launch_t<S3::T, S3::KIND, S3::H, S3::W0, S3::NY, S3::MINB, S3::ZS, false>(a, s);
}
#ifdef HEXS_F3_TRACE
extern "C" int HEXS_F3_CAT(hexs_f3_trace_v, HEXS_F3_VARIANT)(unsigned long long* host, int* counts, int reset) {
  if (cudaMemcpyFromSymbol(host, fast3d::g_f3_tr, sizeof(fast3d::g_f3_tr)) != cudaSuccess) return -1;
  if (cudaMemcpyFromSymbol(counts, fast3d::g_f3_trn, sizeof(fast3d::g_f3_trn)) != cudaSuccess) return -1;
  if (reset) {
    static int zero[fast3d::kTrCtas];
    cudaMemcpyToSymbol(fast3d::g_f3_trn, zero, sizeof(zero));
  }
  return 0;
}
#endif
#ifdef HEXS_F3_TIMING
extern "C" int HEXS_F3_CAT(hexs_f3_timing_v, HEXS_F3_VARIANT)(unsigned long long* host, int reset) {
  if (cudaMemcpyFromSymbol(host, fast3d::g_f3_tm, sizeof(fast3d::g_f3_tm)) != cudaSuccess) return -1;
  if (reset) {
    static unsigned long long zero[1024 * 2 * 8];
    cudaMemcpyToSymbol(fast3d::g_f3_tm, zero, sizeof(zero));
  }
  return 0;
}
#endif
size_t HEXS_F3_CAT(fast3d_smem_v, HEXS_F3_VARIANT)() {
  return fast3d::Lay<S3::T, fast3d::Hex<S3::H, S3::W0>::Q, S3::NY>::SMEM;
}

}  // namespace hexs
