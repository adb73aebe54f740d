// stream3d.cu -- the streaming sm_100a phase kernel for 3D star stencils of radius 1
// (star3d7 = heat/laplacian 3D, gradient3d) under the hybrid schedule of Sec. 3.6
// (PAPER.md:592-632): hexagonal tiles over (t, y), classical tiles over z and x.
// Compiled once per (class, h, w0) of stream3d_variants.h (-DHEXS_S3_VARIANT=id).
//
// Schedule (planner: plan.cpp, EXEC_STREAM3D):
//   * hexagonal dimension y (dim 1; any non-innermost dimension may be hexagonal,
//     PAPER.md:633-641).  A launch (T, p) runs every hexagon S0 of the phase concurrently.
//   * classical tiling of z (dim 0) with width w_z = 1 and skew 1: tile S_z at local level a
//     is the single plane z = S_z - a (eq. (14)).  Tiles are executed in
//     ascending S_z by one CTA -- "streaming": step s of the CTA is tile S_z = s, and computes
//     plane s - a of every level a of the hexagon.  Every dependence of level a (planes
//     z-1, z, z+1 of level a-1) points to steps s-2, s-1, s, so the hexagon's time wavefront
//     lives in registers (a 3-plane ring per level and thread) -- the register tiling the
//     paper names as its next step -- and no tile waits on another CTA
//     for its z-neighbours.
//   * classical tiling of x (dim 2) with width NX = 64 and skew 4 per level (any integer skew
//     >= delta1_x = 1 keeps eq. (14) valid, reading R16; 4 keeps every quad 16-B
//     aligned).  The strips of one hexagon are separate CTAs; strip j depends on strip j-1
//     (S_x - 1) only, through the 2 quads per (row, level, plane) that leave strip j-1 at
//     its right edge.  Those travel through a small L2-resident ring (`scratch`) with
//     per-strip progress counters (st.release / ld.acquire), so strips form a pipeline.
//
// Thread mapping: compute warp w owns hexagon rows r = w (lanes 0-15) and its mirror
// r' = 2h+w0-w (lanes 16-31): mirror rows have identical level ranges, so a warp never
// diverges.  A lane owns one x-quad per level; lanes are ring-mapped over the skewed strip
// (lane q holds quad (q + a) mod 16 of level a), so a lane's quad stays put from level to
// level except for one "designated" lane per level, whose next quad enters from strip j-1
// (the carry).
// Per step and level a (plane v = s - a) a lane either
//   COMPUTEs: centre, z-1, z+1 from its register ring, y-1 / y+1 (rows r-1, r+1 of level a-1,
//             plane v) and the x-edges from the shared-memory exchange ring X, or
//   LOADs:    In values of the hexagon (its slanted lower edges), Dirichlet
//             planes/rows, the launch's input level -- brought into X by a producer warp with
//             1-D bulk TMA copies (cp.async.bulk, SASS UBLKCP) two steps ahead.
// Results go to the register ring, to X (for the neighbour rows at the next step) and, when
// the hexagon's Out set (slanted upper edges, top level, level T) contains them, straight to
// HBM with 128-bit stores (interleaved copy-out).
#include <cstdint>
#include <utility>

#include "../stencil_ops.cuh"
#include "devcache.h"
#include "launch.h"
#include "stream3d_variants.h"
#include "tma.cuh"

#ifndef HEXS_S3_VARIANT
#error "stream3d.cu is compiled once per variant: -DHEXS_S3_VARIANT=<id>"
#endif

namespace hexs {
namespace s3d {

constexpr int NQ = kStream3DNX / 4;  // quads per row and strip (a half-warp)
constexpr int NX = kStream3DNX;      // strip width (x)
constexpr int XP = NX + 8;           // X row segment: quads p = -1 .. NQ of the next level's frame
constexpr int NCS = 4;               // carry staging depth (steps)
constexpr int RS = kStream3DRS;      // scratch carry ring depth (steps)
constexpr int kPubEvery = 4;         // steps between progress publications (one gpu-scope release each)

// Hexagon of a radius-1 single-statement stencil (delta0 = delta1 = 1), rows b of level a
// (SURVEY §8(a) closed form of constraints (6)-(13)).
template <int H, int W0>
struct Hx {
  static_assert(W0 % 2 == 1, "rows pair into mirror warps: 2h+w0+1 must be even");
  static constexpr int L = 2 * H + 2;        // levels
  static constexpr int RN = 2 * H + W0 + 1;  // computed rows 0 .. RN-1
  static constexpr int NW = RN / 2;          // compute warps
  static_assert(L <= 15, "ring-mapped lanes: 2h+1 < NQ");
  __host__ __device__ static constexpr int lo(int a) { return a <= H ? H - a : a - H - 1; }
  __host__ __device__ static constexpr int hi(int a) { return a <= H ? H + W0 + a : 3 * H + 1 + W0 - a; }
  // rows of level a read by level a + 1, a in [-1, L-2]
  __host__ __device__ static constexpr int rlo(int a) { return lo(a + 1) - 1; }
  __host__ __device__ static constexpr int rhi(int a) { return hi(a + 1) + 1; }
  // X pair index of (level a, row r), r in [rlo(a), rhi(a)]
  __host__ __device__ static constexpr int pair_base(int a) {
    int n = 0;
    for (int b = -1; b < a; ++b) n += rhi(b) - rlo(b) + 1;
    return n;
  }
  static constexpr int NPAIR = pair_base(L - 1);
  // Out set of a full hexagon: the slanted upper edges and the top level (read by tiles of
  // the next phase; w0+4h+3 values per column)
  __host__ __device__ static constexpr bool out_row(int a, int r) {
    return a == L - 1 || (a == H ? (r == lo(a) || r == hi(a)) : (a > H ? (r <= lo(a) + 1 || r >= hi(a) - 1) : false));
  }
  // scratch carry block of one step: levels 0 .. L-2 x rows 0 .. RN-1 x 8 floats
  static constexpr int CBLK = (L - 1) * RN * 8;
};

template <typename T, int H, int W0, int NXS>
struct Lay {
  using HX = Hx<H, W0>;
  static constexpr int XSLOT = HX::NPAIR * XP;                     // elements per X slot
  static constexpr int C_OFF = NXS * XSLOT;                        // carry staging
  static constexpr int CSLOT = HX::CBLK;
  static constexpr int END = C_OFF + NCS * CSLOT;
  static constexpr size_t SMEM = (size_t)END * sizeof(T) + 1024;   // + barriers, 1 KB aligned
};

__device__ __forceinline__ int ld_acquire(const int* p) {
  int v;
  asm volatile("ld.acquire.gpu.global.b32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void st_release(int* p, int v) {
  asm volatile("st.release.gpu.global.b32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}
__device__ __forceinline__ int ld_relaxed_gpu(const int* p) {
  int v;
  asm volatile("ld.relaxed.gpu.global.b32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ int ld_acquire_cta(const int* p) {
  int v;
  asm volatile("ld.acquire.cta.shared.b32 %0, [%1];" : "=r"(v) : "r"(smem_u32(p)) : "memory");
  return v;
}
__device__ __forceinline__ void st_release_cta(int* p, int v) {
  asm volatile("st.release.cta.shared.b32 [%0], %1;" ::"r"(smem_u32(p)), "r"(v) : "memory");
}
__device__ __forceinline__ void fence_acq_rel_gpu() { asm volatile("fence.acq_rel.gpu;" ::: "memory"); }
// non-blocking probe of an mbarrier phase
__device__ __forceinline__ bool mbar_test_parity(uint64_t* bar, uint32_t parity) {
  uint32_t ok;
  asm volatile(
      "{\n.reg .pred P1;\nmbarrier.test_wait.parity.shared::cta.b64 P1, [%1], %2;\nselp.u32 %0, 1, 0, P1;\n}\n"
      : "=r"(ok)
      : "r"(smem_u32(bar)), "r"(parity)
      : "memory");
  return ok != 0;
}
__device__ __forceinline__ void fence_proxy_async_global() { asm volatile("fence.proxy.async.global;" ::: "memory"); }
__device__ __forceinline__ void named_barrier_sync(int id, int nthreads) {
  asm volatile("bar.sync %0, %1;" ::"r"(id), "r"(nthreads) : "memory");
}
__device__ __forceinline__ float4 lds4(const float* p) { return *reinterpret_cast<const float4*>(p); }
__device__ __forceinline__ void sts4(float* p, float4 v) { *reinterpret_cast<float4*>(p) = v; }

template <int... As, typename F>
__device__ __forceinline__ void for_levels(F&& f, std::integer_sequence<int, As...>) {
  (f(std::integral_constant<int, As>{}), ...);
}

template <int KIND>
__device__ __forceinline__ float point(float c, float n, float s, float w, float e, float u, float d,
                                       const Coef<float>& k) {
  if constexpr (KIND == K_STAR3D7) return star3d7<float>(c, n, s, w, e, u, d, k);
  else return gradient3d<float>(c, n, s, w, e, u, d, k);
}

#ifdef HEXS_S3_TRACE
// Debug builds (-DHEXS_S3_TRACE): globaltimer stamps per CTA ticket and step:
// [0] compute step done, [1] progress published, [2] loader saw the predecessor's step,
// [3] carry copy issued, [4] tid 0 step start, [5] after full_x, [6] after full_c,
// [7] before the barrier, [8 + w] compute warp w ready for the barrier.
constexpr int kS3TrCtas = 512, kS3TrSteps = 1200;
__device__ unsigned long long g_s3_tr[kS3TrCtas][16][kS3TrSteps];
__device__ __forceinline__ unsigned long long gtimer() {
  unsigned long long t;
  asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
  return t;
}
#define S3_TR(kind, step) \
  do { if (item < kS3TrCtas && (step) < kS3TrSteps) g_s3_tr[item][kind][step] = gtimer(); } while (0)
#else
#define S3_TR(kind, step) do { } while (0)
#endif

// Bit A of the returned mask is set for A in [lo, hi] (clamped to [0, 31]).
__device__ __forceinline__ uint32_t bit_range(int lo, int hi) {
  lo = lo < 0 ? 0 : lo;
  hi = hi > 31 ? 31 : hi;
  if (hi < lo) return 0u;
  return (0xffffffffu >> (31 - hi)) & (0xffffffffu << lo);
}

template <int KIND, int H, int W0, int NXS>
__global__ void __launch_bounds__(32 * (Hx<H, W0>::NW + 2), 2)
    stream3d_kernel(const __grid_constant__ Stream3DArgs g) {
  using HX = Hx<H, W0>;
  using LY = Lay<float, H, W0, NXS>;
  constexpr int L = HX::L, RN = HX::RN, NW = HX::NW, NC = 32 * NW;
  extern __shared__ __align__(1024) unsigned char smem_raw[];
  float* const X = reinterpret_cast<float*>(smem_raw);
  float* const Cst = X + LY::C_OFF;
  uint64_t* const bars = reinterpret_cast<uint64_t*>(smem_raw + (size_t)LY::END * sizeof(float));
  uint64_t* const full_x = bars;              // [NXS]: loads of a step landed (TMA bytes)
  uint64_t* const empty_x = bars + NXS;       // [NXS]: slot read by its step (1 arrival)
  uint64_t* const full_c = bars + 2 * NXS;    // [NCS]: carries of a step landed
  uint64_t* const empty_c = bars + 2 * NXS + NCS;
  int* const item_s = reinterpret_cast<int*>(bars + 2 * NXS + 2 * NCS);

  const int tid = threadIdx.x, warp = tid >> 5, lane = tid & 31;
  if (tid == 0) {
    for (int k = 0; k < NXS; ++k) {
      mbar_init(&full_x[k], 1);
      mbar_init(&empty_x[k], 1);
    }
    for (int k = 0; k < NCS; ++k) {
      mbar_init(&full_c[k], 1);
      mbar_init(&empty_c[k], 1);
    }
    mbar_fence_init();
    // strips of one hexagon take consecutive tickets: a CTA's predecessor strip has been
    // scheduled before it (no deadlock on the progress counters)
    item_s[0] = (int)atomicAdd(g.ticket, 1u);
  }
  // zero the exchange ring: garbage never reaches a stored value, but keep the arithmetic on
  // out-of-domain lanes finite and deterministic
  for (int k = tid; k < LY::END; k += blockDim.x) X[k] = 0.f;
  fence_proxy_async_smem();  // the zeroing before any TMA write into X
  __syncthreads();

  const int item = item_s[0];
  const int jstr = item % g.n_str;                     // x strip
  const int64_t S0 = g.S0_lo + item / g.n_str;         // hexagon
  const int i0 = (int)(S0 * g.W - g.row_off);          // y of local row 0 (extents < 2^30)
  const int N0 = (int)g.N0, N1 = (int)g.N1, N2 = (int)g.N2;
  const int64_t plane = (int64_t)N1 * N2;
  const int X0 = jstr * NX;                            // strip origin (level 0)
  const int a_lo = g.a_lo, a_hi = g.a_hi;
  // steps: level a produces plane v = s - a; s in [a_lo - 1, N0 - 2 + a_hi]
  const int s_first = a_lo - 1;
  const int n_steps = N0 - 2 + a_hi - s_first + 1;
  int* const progress = g.progress;
  float* const scratch = g.scratch;
  const bool has_pred = jstr > 0, has_succ = jstr < g.n_str - 1;
  const int par0 = (int)(g.tau0 & 1);  // level a's values live in buffer (par0 + a + 1) & 1

  // Static (per-CTA) classification of (level a, row r), bit A = a + 1, a in [-1, L-1]:
  //   comp:  a in [a_lo, a_hi], r in [lo(a), hi(a)], y interior      -> COMPUTE when v interior
  //   load:  a in [a_lo-1, a_hi-1] (read by level a + 1 in this launch), r in [lo(a+1)-1,
  //          hi(a+1)+1], y in the domain                              -> LOAD unless COMPUTE
  auto classify = [&](int r, uint32_t& comp, uint32_t& load) {
    const int y = i0 + r;
    comp = load = 0u;
#pragma unroll
    for (int A = 0; A <= L; ++A) {
      const int a = A - 1;
      if (a >= 0 && a >= a_lo && a <= a_hi && r >= HX::lo(a) && r <= HX::hi(a) && y >= 1 && y <= N1 - 2)
        comp |= 1u << A;
      if (a <= L - 2 && a <= a_hi - 1 && a >= a_lo - 1 && r >= HX::rlo(a) && r <= HX::rhi(a) && y >= 0 &&
          y <= N1 - 1)
        load |= 1u << A;
    }
  };

  if (warp == NW) {
    // ================= X filler: In / Dirichlet / input-level rows, NXS-2 steps ahead =================
    // lane k owns pairs k, k+32, ... of the X slot (at most 4); their static class is fixed
    constexpr int PPL = (HX::NPAIR + 31) / 32;
    int pa[PPL], py[PPL];
    uint32_t pc = 0u, pl = 0u;  // bit t: pair t of this lane computes / may load
#pragma unroll
    for (int t = 0; t < PPL; ++t) {
      const int k = lane + 32 * t;
      int a = -1;
#pragma unroll
      for (int b = 0; b < L - 1; ++b)
        if (k >= HX::pair_base(b)) a = b;
      const int r = HX::rlo(a) + (k - HX::pair_base(a));
      uint32_t cm, lm;
      classify(r, cm, lm);
      pa[t] = a;
      py[t] = i0 + r;
      if (k < HX::NPAIR && ((cm >> (a + 1)) & 1u)) pc |= 1u << t;
      if (k < HX::NPAIR && ((lm >> (a + 1)) & 1u)) pl |= 1u << t;
    }
    for (int i = 0; i < n_steps; ++i) {
      const int s = s_first + i, slot = i % NXS;  // read by step i + 1
      if (i >= NXS) mbar_wait_parity(&empty_x[slot], (uint32_t)(((i - NXS) / NXS) & 1));
      float* const Xs = X + slot * LY::XSLOT;
      uint32_t nb[PPL], bytes = 0;
#pragma unroll
      for (int t = 0; t < PPL; ++t) {
        nb[t] = 0;
        const int a = pa[t], v = s - a;
        const bool vint = v >= 1 && v <= N0 - 2, vdom = v >= 0 && v <= N0 - 1;
        if (((pl >> t) & 1u) && vdom && !(((pc >> t) & 1u) && vint)) {
          const int xs0 = X0 - 4 * a - 8;  // level-a row segment in level a+1's frame
          const int xs = xs0 < 0 ? 0 : xs0, xe = xs0 + XP > N2 ? N2 : xs0 + XP;
          if (xe > xs) nb[t] = (uint32_t)(xe - xs) * 4u;
        }
        bytes += nb[t];
      }
      const uint32_t total = __reduce_add_sync(0xffffffffu, bytes);
      if (lane == 0) mbar_arrive_expect_tx(&full_x[slot], total);
      __syncwarp();
#pragma unroll
      for (int t = 0; t < PPL; ++t) {
        if (nb[t] == 0) continue;
        const int a = pa[t], xs0 = X0 - 4 * a - 8, xs = xs0 < 0 ? 0 : xs0;
        const float* src = static_cast<const float*>(g.buf[(par0 + a + 1) & 1]) + (int64_t)(s - a) * plane +
                           (int64_t)py[t] * N2 + xs;
        tma_load_1d(Xs + (lane + 32 * t) * XP + (xs - xs0), src, nb[t], &full_x[slot]);
      }
    }
    return;
  }
  if (warp == NW + 1) {
    // ================= carry copier (lane 0): strip j-1's right-edge quads of each step =================
    // into staging slot i % NCS once the compute warps freed it and j-1 has published step i;
    // one acquire fence per observation of j-1's counter (it publishes every few steps)
    if (lane == 0 && has_pred) {
      const int* pp = progress + item - 1;
      const float* src0 = scratch + (size_t)(item - 1) * RS * HX::CBLK;
      int pred_seen = 0;
      for (int ci = 0; ci < n_steps; ++ci) {
        const int slot = ci % NCS;
        if (ci >= NCS) mbar_wait_parity(&empty_c[slot], (uint32_t)(((ci - NCS) / NCS) & 1));
        if (pred_seen < ci + 1) {
          while ((pred_seen = ld_relaxed_gpu(pp)) < ci + 1) __nanosleep(100);
          fence_acq_rel_gpu();         // acquire strip j-1's stores up to step pred_seen - 1 ...
          fence_proxy_async_global();  // ... and order them before these async-proxy reads
          S3_TR(2, ci);
        }
        mbar_arrive_expect_tx(&full_c[slot], (uint32_t)(HX::CBLK * sizeof(float)));
        tma_load_1d(Cst + slot * LY::CSLOT, src0 + (size_t)(ci % RS) * HX::CBLK, HX::CBLK * sizeof(float),
                    &full_c[slot]);
        S3_TR(3, ci);
      }
    }
    return;
  }

  // ================= compute warps =================
  const int half = lane >> 4, q = lane & 15;
  const int r = half ? RN - 1 - warp : warp;  // this lane's hexagon row
  const int y = i0 + r;
  const Coef<float> cf{(float)g.k0, (float)g.k1};
  float* const my_scratch = scratch + (size_t)item * RS * HX::CBLK;
  uint32_t m_comp, m_load;
  classify(r, m_comp, m_load);
  // per level (bit A): Out-set stores, quad fully in the domain, Dirichlet x = 0 / x = N2-1
  uint32_t m_out = 0u, m_xin = 0u, m_xl = 0u, m_xr = 0u;
#pragma unroll
  for (int A = 1; A <= L; ++A) {
    const int a = A - 1;
    const int x = X0 - 4 * a + 4 * ((q + a) & (NQ - 1));
    if (HX::out_row(a, r) || a == g.a_final) m_out |= 1u << A;
    if (x >= 0 && x + 3 <= N2 - 1) m_xin |= 1u << A;
    if (x == 0) m_xl |= 1u << A;
    if (x + 3 == N2 - 1) m_xr |= 1u << A;
  }
  m_out &= m_xin;
  float* const gb0 = static_cast<float*>(g.buf[0]);
  float* const gb1 = static_cast<float*>(g.buf[1]);
  const int rXP = r * XP;       // this row's offset inside a level block of X
  const int64_t yN2 = (int64_t)y * N2;
  float4 ring[L][3];  // [level a + 1][step mod 3]: level a's plane produced at that step
#pragma unroll
  for (int A = 0; A < L; ++A)
#pragma unroll
    for (int k = 0; k < 3; ++k) ring[A][k] = make_float4(0.f, 0.f, 0.f, 0.f);
  int succ_seen = 0;  // tid 0: strip j+1's published progress (back-pressure cache)

  // end of a step (all compute warps): back-pressure for the next step's scratch writes, the
  // step barrier, then tid 0 releases the consumed slots and publishes progress every
  // kPubEvery steps (one gpu-scope release; warp 0 carries the lightest rows)
  auto end_step = [&](int i) {
    if (tid == 0 && has_succ && i + 1 < n_steps && succ_seen < i + 2 - RS) {
      // step i+1 rewrites scratch slot (i+1) % RS: strip j+1 must have finished step i+1-RS
      while ((succ_seen = ld_relaxed_gpu(progress + item + 1)) < i + 2 - RS) __nanosleep(64);
      fence_acq_rel_gpu();
    }
    if (tid == 0) S3_TR(7, i);
    named_barrier_sync(1, NC);  // step i done: X[i % NXS] complete, X[(i-1) % NXS] free
    if (tid == 0) {
      S3_TR(0, i);
      if (i >= 1) mbar_arrive(&empty_x[(i - 1) % NXS]);
      if (has_pred) mbar_arrive(&empty_c[i % NCS]);
      if ((i + 1) % kPubEvery == 0 || i + 1 == n_steps) {
        st_release(progress + item, i + 1);  // cumulative over the CTA's stores (bar.sync above)
        S3_TR(1, i);
      }
    }
  };

  // ---------------- general step (stream ends, t-cut launches, hexagons cut by y) ----------------
  auto step = [&](int i, auto slc) {
    constexpr int SL = decltype(slc)::value;  // i % 3
    constexpr int SLm1 = (SL + 2) % 3, SLm2 = (SL + 1) % 3;
    const int s = s_first + i;
    const float* const Xc = X + ((i + NXS - 1) % NXS) * LY::XSLOT + rXP;  // values produced at step i-1
    float* const Xn = X + (i % NXS) * LY::XSLOT + rXP;                   // values produced now
    const float* const Cc = Cst + (i % NCS) * LY::CSLOT + r * 8;         // strip j-1's carries
    float* const Sc = my_scratch + (size_t)(i % RS) * HX::CBLK + r * 8;  // strip j+1's carries
    // levels whose plane v = s - a is interior (COMPUTE) / in the domain (LOAD)
    const uint32_t vint = bit_range(s - N0 + 3, s), vdom = bit_range(s - N0 + 2, s + 1);
    const uint32_t doc = m_comp & vint, dol = m_load & vdom & ~doc;
    mbar_wait_parity(&full_x[i % NXS], (uint32_t)((i / NXS) & 1));
    if (has_pred) mbar_wait_parity(&full_c[i % NCS], (uint32_t)((i / NCS) & 1));
    for_levels(
        [&](auto ac) {
          constexpr int A = decltype(ac)::value;  // 0 .. L: level a = A - 1
          constexpr int a = A - 1;
          const int pr = (q + a) & (NQ - 1);     // quad in this level's frame (reading frame)
          const int colr = 4 * pr + 4;           // X column of that quad; its next-level slot is colr + 4
          if constexpr (a >= 0) {
            if ((doc >> A) & 1u) {
              // ---- COMPUTE level a at (v, y, quad): inputs of level a-1 ----
              constexpr int RB = (HX::pair_base(a - 1) - HX::rlo(a - 1)) * XP;  // level a-1 block
              const float4 c = ring[A - 1][SLm1], u = ring[A - 1][SLm2], d = ring[A - 1][SL];
              const float* rowc = Xc + RB + colr;
              const float4 n = lds4(rowc - XP);
              const float4 so = lds4(rowc + XP);
              const float we = rowc[-1], ee = rowc[4];
              float4 o;
              o.x = point<KIND>(c.x, n.x, so.x, we, c.y, u.x, d.x, cf);
              o.y = point<KIND>(c.y, n.y, so.y, c.x, c.z, u.y, d.y, cf);
              o.z = point<KIND>(c.z, n.z, so.z, c.y, c.w, u.z, d.z, cf);
              o.w = point<KIND>(c.w, n.w, so.w, c.z, ee, u.w, d.w, cf);
              if ((m_xl >> A) & 1u) o.x = c.x;  // Dirichlet columns keep their value
              if ((m_xr >> A) & 1u) o.w = c.w;
              // ---- copy-out: Out set of the hexagon, every value of level T_steps ----
              if ((m_out >> A) & 1u) {
                const int x = X0 - 4 * a + 4 * pr;
                float* gp = (((par0 + a + 1) & 1) ? gb1 : gb0) + (int64_t)(s - a) * plane + yN2 + x;
                *reinterpret_cast<float4*>(gp) = o;
              }
              if constexpr (a <= L - 2) {
                if (a <= a_hi - 1) {
                  constexpr int WB = (HX::pair_base(a) - HX::rlo(a)) * XP;  // level a block
                  sts4(Xn + WB + colr + 4, o);
                  // strip j+1's carries: this level's last two quads
                  if (has_succ && pr >= NQ - 2)
                    *reinterpret_cast<float4*>(Sc + a * RN * 8 + (pr - (NQ - 2)) * 4) = o;
                  // the designated lane's next quad (p = 0) and the edge quad (p = -1) come from
                  // strip j-1
                  if (has_pred && pr == NQ - 1) {
                    const float4 c0 = lds4(Cc + a * RN * 8), c1 = lds4(Cc + a * RN * 8 + 4);
                    sts4(Xn + WB, c0);
                    sts4(Xn + WB + 4, c1);
                    o = c1;
                  }
                  ring[A][SL] = o;
                }
              }
              return;
            }
          }
          if constexpr (a <= L - 2) {
            // ---- LOAD: values the X filler brought into Xn (In rows, Dirichlet, input level) ----
            if ((dol >> A) & 1u) {
              constexpr int WB = (HX::pair_base(a) - HX::rlo(a)) * XP;
              ring[A][SL] = lds4(Xn + WB + (pr == NQ - 1 ? 4 : colr + 4));
            }
          }
        },
        std::make_integer_sequence<int, L + 1>{});
    fence_proxy_async_smem();  // this thread's X writes before later TMA writes to the slot
    end_step(i);
  };

  // ---------------- fast path: interior steps of a full hexagon inside the domain ----------------
  // Every level of every row runs the same straight-line body (levels a row does not compute
  // produce ignored values): no per-level branches, so the compiler interleaves the levels'
  // loads and arithmetic, and one copy of the code serves every warp (instruction cache).  The
  // row's static modes only predicate the side effects.  Stream ends, t-cut launches and
  // hexagons cut by the y boundary take `step` above.
  const bool fast_cta = a_lo == 0 && a_hi == L - 1 && i0 - 1 >= 0 && i0 + RN <= N1 - 1;
  const uint32_t f_comp = m_comp, f_load = m_load & ~m_comp;
  auto fast = [&](int i, auto slc) {
    constexpr int SL = decltype(slc)::value;
    constexpr int SLm1 = (SL + 2) % 3, SLm2 = (SL + 1) % 3;
    const int s = s_first + i;
    const float* const Xc = X + ((i + NXS - 1) % NXS) * LY::XSLOT + rXP;
    float* const Xn = X + (i % NXS) * LY::XSLOT + rXP;
    const float* const Cc = Cst + (i % NCS) * LY::CSLOT + r * 8;
    float* const Sc = my_scratch + (size_t)(i % RS) * HX::CBLK + r * 8;
    float* const gpe = (((par0 + 1) & 1) ? gb1 : gb0) + (int64_t)s * plane + yN2 + X0;  // even levels
    float* const gpo = (((par0 + 1) & 1) ? gb0 : gb1) + (int64_t)s * plane + yN2 + X0;  // odd levels
    mbar_wait_parity(&full_x[i % NXS], (uint32_t)((i / NXS) & 1));
    if (has_pred) mbar_wait_parity(&full_c[i % NCS], (uint32_t)((i / NCS) & 1));
    for_levels(
        [&](auto ac) {
          constexpr int A = decltype(ac)::value;
          constexpr int a = A - 1;
          constexpr bool NEED = a <= L - 2;
          const int pr = (q + a) & (NQ - 1);
          const int colr = 4 * pr + 4;
          const bool lo_ = (f_load >> A) & 1u;
          if constexpr (a >= 0) {
            const bool co = (f_comp >> A) & 1u;
            constexpr int RB = (HX::pair_base(a - 1) - HX::rlo(a - 1)) * XP;
            const float4 c = ring[A - 1][SLm1], u = ring[A - 1][SLm2], d = ring[A - 1][SL];
            const float* rowc = Xc + RB + colr;
            const float4 n = lds4(rowc - XP);
            const float4 so = lds4(rowc + XP);
            const float we = rowc[-1], ee = rowc[4];
            float4 o;
            o.x = point<KIND>(c.x, n.x, so.x, we, c.y, u.x, d.x, cf);
            o.y = point<KIND>(c.y, n.y, so.y, c.x, c.z, u.y, d.y, cf);
            o.z = point<KIND>(c.z, n.z, so.z, c.y, c.w, u.z, d.z, cf);
            o.w = point<KIND>(c.w, n.w, so.w, c.z, ee, u.w, d.w, cf);
            o.x = ((m_xl >> A) & 1u) ? c.x : o.x;  // Dirichlet columns keep their value
            o.w = ((m_xr >> A) & 1u) ? c.w : o.w;
            if ((m_out >> A) & (f_comp >> A) & 1u) {
              float* gp = ((a & 1) ? gpo : gpe) - (int64_t)a * plane - 4 * a + 4 * pr;
              *reinterpret_cast<float4*>(gp) = o;
            }
            if constexpr (NEED) {
              constexpr int WB = (HX::pair_base(a) - HX::rlo(a)) * XP;
              if (co) {
                sts4(Xn + WB + colr + 4, o);
                if (has_succ && pr >= NQ - 2)
                  *reinterpret_cast<float4*>(Sc + a * RN * 8 + (pr - (NQ - 2)) * 4) = o;
                if (has_pred && pr == NQ - 1) {
                  const float4 c0 = lds4(Cc + a * RN * 8), c1 = lds4(Cc + a * RN * 8 + 4);
                  sts4(Xn + WB, c0);
                  sts4(Xn + WB + 4, c1);
                  o = c1;
                }
              }
              if (lo_) o = lds4(Xn + WB + (pr == NQ - 1 ? 4 : colr + 4));
              ring[A][SL] = o;
            }
          } else {
            constexpr int WB = (HX::pair_base(a) - HX::rlo(a)) * XP;
            if (lo_) ring[A][SL] = lds4(Xn + WB + (pr == NQ - 1 ? 4 : colr + 4));
          }
        },
        std::make_integer_sequence<int, L + 1>{});
    end_step(i);
  };
  // interior steps: every level's plane v = s - a in [1, N0-2]; and no TMA rewrite (Dirichlet
  // planes at the stream's end) of a slot the lanes wrote (X ring depth NXS), so no proxy fence
  const int i_fast_lo = fast_cta ? L - s_first : n_steps;
  const int i_fast_hi = fast_cta ? N0 - 3 - NXS - s_first : -1;
  int i = 0;
  for (; i + 3 <= n_steps; i += 3) {
    if (i >= i_fast_lo && i + 2 <= i_fast_hi) {
      fast(i, std::integral_constant<int, 0>{});
      fast(i + 1, std::integral_constant<int, 1>{});
      fast(i + 2, std::integral_constant<int, 2>{});
    } else {
      step(i, std::integral_constant<int, 0>{});
      step(i + 1, std::integral_constant<int, 1>{});
      step(i + 2, std::integral_constant<int, 2>{});
    }
  }
  if (i < n_steps) step(i, std::integral_constant<int, 0>{});
  if (i + 1 < n_steps) step(i + 1, std::integral_constant<int, 1>{});
}

template <int KIND, int H, int W0, int NXS>
cudaError_t launch_t(const Stream3DArgs& a, cudaStream_t s) {
  using HX = Hx<H, W0>;
  constexpr size_t smem = Lay<float, H, W0, NXS>::SMEM;
  constexpr int NT = 32 * (HX::NW + 2);
  auto kern = stream3d_kernel<KIND, H, W0, NXS>;
  static DeviceMemo<int> memo;
  int ok = 0;
  cudaError_t e = memo.get(&ok, [&](int, int* v) {
    *v = 1;
    return cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  });
  if (e != cudaSuccess) return e;
  if (a.L != HX::L || a.RN != HX::RN) return cudaErrorInvalidValue;
  kern<<<(unsigned)a.n_items, NT, smem, s>>>(a);
  return cudaGetLastError();
}

}  // namespace s3d

template <int ID> struct SelS3;
#define HEXS_S3_SEL(id, dc, T_, KIND_, H_, W0_, NXS_)                   \
  template <> struct SelS3<id> {                                        \
    static constexpr int KIND = KIND_, H = H_, W0 = W0_, NXS = NXS_;    \
  };
HEXS_STREAM3D_VARIANTS(HEXS_S3_SEL)
#undef HEXS_S3_SEL
#define HEXS_S3_CAT2(a, b) a##b
#define HEXS_S3_CAT(a, b) HEXS_S3_CAT2(a, b)
using SS3 = SelS3<HEXS_S3_VARIANT>;

cudaError_t HEXS_S3_CAT(launch_stream3d_v, HEXS_S3_VARIANT)(const Stream3DArgs& a, cudaStream_t s) {
  return s3d::launch_t<SS3::KIND, SS3::H, SS3::W0, SS3::NXS>(a, s);
}
int HEXS_S3_CAT(stream3d_carry_block_v, HEXS_S3_VARIANT)() { return s3d::Hx<SS3::H, SS3::W0>::CBLK; }

#ifdef HEXS_S3_TRACE
extern "C" int HEXS_S3_CAT(hexs_s3_trace_v, HEXS_S3_VARIANT)(unsigned long long* host) {
  return cudaMemcpyFromSymbol(host, s3d::g_s3_tr, sizeof(s3d::g_s3_tr)) == cudaSuccess ? 0 : -1;
}
#endif

}  // namespace hexs
