// hex3d.cu -- the specialised sm_100a phase kernel for 3D single-field stencils of radius 1
// (star3d7, gradient3d, box3d27) under the hybrid schedule: hexagonal over (t, z), classical
// parallelogram tiles over y and x (eq. (14)).
//
// Mapping:
//   * work item = one classical tile (S1, S2) of one hexagon S0 of the launch's (T, p): a
//     NY x NX (y, x) parallelogram over the hexagon's 2h+2 levels and rows z.  Skews: y by 1
//     per level (delta1_y = 1), x by 4 per level with a +1 tile translation (Sec. 4.2.3,
//     PAPER.md:755-763) so that every x-window this kernel moves starts on a 16-B boundary
//     (the TMA unit requires it; any skew >= delta1_x keeps eq. (14) valid -- reading R16);
//   * work item = one ROW of tiles (S0, S1): the CTA streams its tiles S2 = 0, 1, ...
//     sequentially, as the paper's blocks do with their classical loops,
//     so the x-predecessor of every tile is the CTA's own previous tile (complete before the
//     next starts).  Rows are pipelined across CTAs at LEVEL granularity: level a of tile
//     (S1, S2) needs row S1-1 to have finished level a-1 of its tile S2.  Each row publishes
//     one monotonic progress counter (tiles x levels done, st.release after the level's
//     carries are in global memory); persistent CTAs fetch rows S1-major from an atomic
//     counter, so the ~23-51 hexagons x 65 rows of a 512^3 phase keep all 148 SMs busy;
//   * the tile's current level lives in shared memory (two level buffers: planes z x 18
//     lines x 40 columns); a thread owns 2 lines x 4 columns of one half of the rows and
//     sweeps z with a 3-plane register window (z-neighbours from registers, y/x neighbours
//     from LDS.128 + LDS.64);
//   * everything a tile reads from L2/HBM arrives by 3-D TMA tensor copies
//     (cp.async.bulk.tensor.3d, SASS UTMALDG) completing on one mbarrier per level buffer:
//     the In planes of level a+1 (the hexagon's slanted-edge inputs) one
//     level ahead, the carries (2 lines above / 5 columns left, produced by the predecessor
//     tiles in this launch) when their flags allow; out-of-grid box elements are zero-filled
//     by the TMA unit and never used;
//   * results leave from registers: the Out planes, the tile's last 2 lines and 5 columns
//     (its successors' carries) and the final level -- interleaved copy-out.
#include <cuda.h>
#include <cudaTypedefs.h>

#include <cstdint>
#include <type_traits>

#include "../stencil_ops.cuh"
#include "launch.h"
#include "tma.cuh"

namespace hexs {
namespace fast3d {

constexpr int NY = kFast3DNY, NX = kFast3DNX;  // classical tile (y lines, x columns)
constexpr int NLP = NY / 2;                    // line pairs per tile
#ifndef HEXS_3D_NRG
#define HEXS_3D_NRG 4
#endif
constexpr int NRG = HEXS_3D_NRG;               // row groups (one compute warp each for NY = 8)
constexpr int NCT = NRG * NLP * 8;             // compute threads: row groups x NLP line pairs x 8 column quads
constexpr int NT = NCT + 32;                   // + one producer warp (loads, flags)
// resident CTAs per SM the register budget is cut for (fp32 tiles fit 4 per SM in shared
// memory; the 27-point box needs more registers, fp64 doubles every buffer)
template <typename T, int KIND> constexpr int MINB = sizeof(T) == 8 ? 2 : (KIND == K_BOX3D27 ? 3 : 4);
constexpr int SIGMA = 4;                       // x skew per level
constexpr int CL = SIGMA + 1;                  // left carry columns (skew + stencil radius)
constexpr int LY = NY + 2;                     // buffer lines: 2 carry lines + NY
constexpr int SX = 40;                         // buffer columns: CL carry + NX window (+3), TMA box
// plane pitch (elements), padded so every TMA destination is 128-B aligned
template <typename T> constexpr int PP = ((LY * SX * (int)sizeof(T) + 127) / 128 * 128) / (int)sizeof(T);
template <typename T> constexpr size_t smem_bytes(int Q) {
  return (size_t)2 * Q * PP<T> * sizeof(T) + 128;
}

struct Maps {
  CUtensorMap plane[2];  // box {SX, LY, 1}   per ping-pong buffer
};

__device__ __forceinline__ int ld_relaxed(const int* p) {
  int v;
  asm volatile("ld.relaxed.gpu.global.b32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
// relaxed polls + one fence = acquire (no per-poll L1 invalidation)
__device__ __forceinline__ void fence_acq_rel_gpu() { asm volatile("fence.acq_rel.gpu;" ::: "memory"); }
// order the acquired generic-proxy view before later async-proxy (TMA) reads of global memory
__device__ __forceinline__ void fence_proxy_async_global() { asm volatile("fence.proxy.async.global;" ::: "memory"); }
__device__ __forceinline__ bool mbar_test_parity(uint64_t* bar, uint32_t parity) {
  uint32_t ok;
  asm volatile(
      "{\n.reg .pred P1;\nmbarrier.test_wait.parity.shared::cta.b64 P1, [%1], %2;\nselp.u32 %0, 1, 0, P1;\n}\n"
      : "=r"(ok)
      : "r"(smem_u32(bar)), "r"(parity)
      : "memory");
  return ok != 0;
}
__device__ __forceinline__ void mbar_arrive(uint64_t* bar) {
  asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(smem_u32(bar)) : "memory");
}
// parity wait that suspends the warp (up to the hint, in ns) instead of spinning
__device__ __forceinline__ void mbar_wait_sleep(uint64_t* bar, uint32_t parity) {
  asm volatile(
      "{\n"
      ".reg .pred P1;\n"
      "HEXS_WS_%=:\n"
      "mbarrier.try_wait.parity.shared::cta.b64 P1, [%0], %1, %2;\n"
      "@!P1 bra.uni HEXS_WS_%=;\n"
      "}\n" ::"r"(smem_u32(bar)),
      "r"(parity), "n"(1000000)
      : "memory");
}
// 16-/8-/4-B asynchronous global -> shared copies (LDGSTS); src_size 0 zero-fills
__device__ __forceinline__ void cp_async16(void* dst, const void* src, bool valid) {
  asm volatile("cp.async.cg.shared.global [%0], [%1], 16, %2;" ::"r"(smem_u32(dst)), "l"(src), "r"(valid ? 16 : 0)
               : "memory");
}
template <int N>
__device__ __forceinline__ void cp_async_small(void* dst, const void* src, bool valid) {
  asm volatile("cp.async.ca.shared.global [%0], [%1], %2, %3;" ::"r"(smem_u32(dst)), "l"(src), "n"(N),
               "r"(valid ? N : 0)
               : "memory");
}
// the mbarrier tracks this thread's earlier cp.async (pending count +1, arrival on completion)
__device__ __forceinline__ void cp_async_mbar_arrive(uint64_t* bar) {
  asm volatile("cp.async.mbarrier.arrive.shared::cta.b64 [%0];" ::"r"(smem_u32(bar)) : "memory");
}
// named barrier 1 over the compute warps only (the producer warp never joins it)
__device__ __forceinline__ void bar_compute() { asm volatile("bar.sync 1, %0;" ::"n"(NCT) : "memory"); }
__device__ __forceinline__ void st_release(int* p, int v) {
  asm volatile("st.release.gpu.global.b32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}
__device__ __forceinline__ long long gtimer() {
  long long t;
  asm volatile("mov.u64 %0, %globaltimer;" : "=l"(t));
  return t;
}
constexpr int kTraceStride = 32;  // per item: [sm, start, prologue, (flag, data, done) per level]

__device__ __forceinline__ void mbar_expect_tx(uint64_t* bar, uint32_t bytes) {
  asm volatile("mbarrier.expect_tx.relaxed.cta.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(bar)), "r"(bytes)
               : "memory");
}
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

// Buffer conventions.  The input buffer of level a (level a-1 values) has its column 0 at
// x = X0 - 4a (16-B aligned) and its line 0 at y = Y0 - a - 1: columns [0, CL) and lines
// {0, 1} are carries, the tile's own level-(a-1) window sits at columns [CL, CL + NX) and
// lines [2, LY).  Level a's output window (x in [X0-4a+1, X0-4a+NX], y in [Y0-a, Y0-a+NY))
// is written into the other buffer in ITS convention (column = x - (X0 - 4(a+1)),
// line = y - (Y0 - a - 2)).  A thread (lp, xq) computes outputs x = X0-4a+1+4xq+j,
// y = Y0-a+2lp+i, whose inputs sit at input columns [4xq, 4xq+5] and lines [2lp, 2lp+3].
//
// Warp roles.  Warps 0..1 compute; warp 2 (the producer) runs one level ahead of them:
// while level a is computed it publishes level a-1 (st.release once the compute warps have
// signalled it done), issues the In planes of level a+1, polls the predecessors' flags for
// level a, issues the carries of level a+1, moves the carry columns into place and arms the
// `ready` barrier of level a+1.  Compute warps only ever wait on `ready`.
//
// Shared-memory hazards (all buffer regions named in the convention above):
//   * In planes of level a+1 land in planes level a does not write -- issued after level
//     a-1 (their previous reader) is done;
//   * carries of level a+1 land in lines {0,1} / columns [0, CL) of ob(a), which level a
//     (writing lines >= 2, columns >= CL) does not touch;
//   * level a+1 reads rows of both compute warps: a named barrier of the compute warps
//     closes every level before either passes `ready` of the next.
template <typename T, int KIND>
__global__ void __launch_bounds__(NT, (MINB<T, KIND>)) fast3d_kernel(const __grid_constant__ Fast3DArgs g,
                                                       const __grid_constant__ Maps m) {
  extern __shared__ __align__(1024) unsigned char smem_raw[];  // dynamic base is 1024-B aligned
  __shared__ __align__(8) uint64_t full[2], ready[2], done[2];
  __shared__ int64_t item_s[3];
  T* buf = reinterpret_cast<T*>(smem_raw);  // stays a shared-space pointer (LDS/STS, not generic LD/ST)
  auto B = [&](int which, int q, int ly, int lx) -> T* {
    return buf + ((size_t)which * g.Q + q) * PP<T> + ly * SX + lx;
  };
  const int tid = threadIdx.x;
  const int64_t n1 = g.n1, n2 = g.n2;
  const int64_t plane = g.N1 * g.N2;
  if (tid == 0) {
    for (int b = 0; b < 2; ++b) {
      mbar_init(&full[b], 1);
      mbar_init(&ready[b], 1);
      mbar_init(&done[b], 1);
    }
    mbar_fence_init();
  }
  __syncthreads();

  if (tid >= NCT) {
    // ------------------------------------------------------------------ producer warp
    const int lane = tid - NCT;
    const int64_t ns0 = g.S0_hi - g.S0_lo + 1;
    const uint32_t plane_bytes = LY * SX * sizeof(T);
    const int Lp = g.a_hi - g.a_lo + 1;  // levels per tile in this launch
    // The next tile's first level can be staged during this tile's last level when that
    // level neither reads nor writes buffer a_lo & 1 (the compute warps skip the smem
    // writes of the last level): true iff a_hi - a_lo is odd.
    const bool early = ((g.a_hi - g.a_lo) & 1) != 0;
    const bool no_carry = (g.dbg & 1) != 0, no_in = (g.dbg & 2) != 0;  // timing experiments only
    const bool no_fence = (g.dbg & 4) != 0;
    uint32_t ph_full = 0u;  // phase parity bit per buffer (all lanes)
    uint32_t ph_done = 0u;  // lane 0 only: `done` is consumed by lane 0
    struct Tile {
      int64_t S0, q1, q2;
    };
    // next tile in stream order: the row's next S2, else a freshly fetched row (S1-major,
    // so a row's predecessor is always fetched first)
    auto next_tile = [&](const Tile& t) -> Tile {
      if (t.S0 >= 0 && t.q2 + 1 < n2) return Tile{t.S0, t.q1, t.q2 + 1};
      int64_t it = 0;
      if (lane == 0) it = (int64_t)atomicAdd(g.counter, 1ull);
      it = __shfl_sync(0xffffffffu, it, 0);
      if (it >= ns0 * n1) return Tile{-1, 0, 0};
      return Tile{g.S0_lo + it % ns0, it / ns0, 0};
    };
    // stage level a_lo of tile t (every input plane comes from earlier launches)
    auto stage_first = [&](const Tile& t) {
      if (lane == 0 && t.S0 >= 0) {
        const int a = g.a_lo, ib = a & 1;
        const int64_t i0 = t.S0 * g.W - g.row_off;
        const int64_t Y0 = (g.S1_lo + t.q1) * NY, X0 = (g.S2_lo + t.q2) * NX;
        if (no_in) {
          mbar_arrive(&full[ib]);
          return;
        }
        fence_proxy_async_smem();
        const int qlo = g.lo[a], qhi = g.hi[a] + 2;
        mbar_arrive_expect_tx(&full[ib], plane_bytes * (qhi - qlo + 1));
        const CUtensorMap* mp = &m.plane[(g.tau0 + a) & 1];
        for (int q = qlo; q <= qhi; ++q)
          tma_3d(B(ib, q, 0, 0), mp, (int)(X0 - SIGMA * a), (int)(Y0 - a - 1), (int)(i0 + q - 1), &full[ib]);
      }
    };
    bool have_prev = false, staged = false;
    long long* prev_tr = nullptr;
    Tile cur = next_tile(Tile{-1, 0, 0});
    while (true) {
      const int64_t S0 = cur.S0, q1 = cur.q1, q2 = cur.q2;
      long long* tr = nullptr;
      if (g.trace && lane == 0 && S0 >= 0) {
        tr = g.trace + ((S0 - g.S0_lo) * n1 * n2 + q1 * n2 + q2) * kTraceStride;
        unsigned smid;
        asm volatile("mov.u32 %0, %smid;" : "=r"(smid));
        tr[0] = ((long long)smid << 32) | (long long)(q1 * 65536 + q2);
        tr[1] = gtimer();
      }
      if (lane == 0) {
        // the previous tile's last level must be done before item_s / its buffers are reused
        if (have_prev) {
          const int b = g.a_hi & 1;
          mbar_wait_parity(&done[b], (ph_done >> b) & 1u);
          ph_done ^= 1u << b;
          if (prev_tr) prev_tr[5 + 3 * (g.a_hi - g.a_lo)] = gtimer();
        }
        item_s[0] = S0;
        item_s[1] = q1;
        item_s[2] = q2;
      }
      prev_tr = tr;
      if (S0 < 0) {
        if (lane == 0) mbar_arrive(&ready[g.a_lo & 1]);  // releases the compute warps
        break;
      }
      if (!staged) stage_first(cur);
      {
        const int ib = g.a_lo & 1;
        if (lane == 0) {
          mbar_wait_parity(&full[ib], (ph_full >> ib) & 1u);
          if (tr) tr[2] = gtimer();
          mbar_arrive(&ready[ib]);  // also publishes item_s (release.cta)
        }
        ph_full ^= 1u << ib;
      }
      have_prev = true;
      staged = false;
      int* row_flag = g.flags + (S0 - g.S0_lo) * n1 + q1;
      const int base = (int)q2 * Lp;  // progress value of this tile's start
      const int64_t i0 = S0 * g.W - g.row_off;  // z of local row b = 0 (buffer plane q = b + 1)
      const int64_t Y0 = (g.S1_lo + q1) * NY, X0 = (g.S2_lo + q2) * NX;
      // Level publication (lane 0).  `cons` levels of this tile have been seen done; each is
      // published (st.release.gpu, cumulative over the compute warps' stores ordered before
      // their `done` arrival) as soon as it is seen -- also while polling, so a row never
      // holds back its successor while it waits for its own predecessor.
      int cons = 0;
      auto consume = [&](bool block) -> bool {  // lane 0: try to see level a_lo + cons done
        const int lvl = g.a_lo + cons, b = lvl & 1;
        const uint32_t par = (ph_done >> b) & 1u;
        if (block) mbar_wait_parity(&done[b], par);
        else if (!mbar_test_parity(&done[b], par)) return false;
        ph_done ^= 1u << b;
        ++cons;
        if (tr) tr[5 + 3 * (lvl - g.a_lo)] = gtimer();
        if (lvl < g.a_hi && !no_fence) st_release(row_flag, base + cons);
        return true;
      };

      for (int a = g.a_lo; a < g.a_hi; ++a) {  // prepare level a+1 while level a is computed
        const int nb = (a + 1) & 1;
        const int tk = 3 + 3 * (a + 1 - g.a_lo);
        const int plo = g.lo[a], phi = g.hi[a];  // rows computed at level a
        const int xo = (int)(X0 - SIGMA * (a + 1)), yo = (int)(Y0 - a - 2);
        if (lane == 0) {
          // level a-1 (the last reader of buffer nb) done and published
          while (cons < a - g.a_lo) consume(true);
          // (1) In planes of level a+1 (the planes level a does not write): TMA
          const int qlo = g.lo[a + 1], qhi = g.hi[a + 1] + 2;
          int n_in = 0;
          for (int q = qlo; q <= qhi; ++q)
            if (q - 1 < plo || q - 1 > phi) ++n_in;
          fence_proxy_async_smem();
          if (n_in && !no_in) {
            mbar_expect_tx(&full[nb], plane_bytes * n_in);
            const CUtensorMap* mp = &m.plane[(g.tau0 + a + 1) & 1];
            for (int q = qlo; q <= qhi; ++q)
              if (q - 1 < plo || q - 1 > phi) tma_3d(B(nb, q, 0, 0), mp, xo, yo, (int)(i0 + q - 1), &full[nb]);
          }
          // (2) the row predecessor's level a (relaxed polls, one fence); the x-predecessor
          // is this CTA's previous tile, complete before this one began.  Our own level a is
          // published the moment it is done.
          const int need = base + a - g.a_lo + 1;
          const int* f_y = row_flag - 1;
          while (!no_carry && q1 > 0 && ld_relaxed(f_y) < need) {
            if (cons == a - g.a_lo) consume(false);
            __nanosleep(32);
          }
          if (!no_fence) fence_acq_rel_gpu();
          if (tr) tr[tk] = gtimer();
        }
        __syncwarp();
        // (3) carries of level a+1 straight into place with 16-B cp.async (all lanes):
        // lines {0,1} x SX columns and lines [2, LY) x columns [0, CL) of every plane that
        // level a computes; out-of-grid chunks are zero-filled (never used).  Each lane owns
        // fixed chunks of a plane (job k = lane, lane + 32), so a plane costs a few adds.
        {
          const T* src = static_cast<const T*>(g.buf[(g.tau0 + a + 1) & 1]);
          constexpr int CH = 16 / sizeof(T);   // elements per 16-B chunk
          constexpr int NLC = 2 * (SX / CH);   // line-carry chunks per plane
          constexpr int NCC = NY * (CL / CH);  // column-carry 16-B chunks per plane
          constexpr int NPP = NLC + NCC + NY;  // + one small copy per line for the last column(s)
          static_assert(NPP <= 64, "two jobs per lane");
          int64_t goff[2];
          int soff[2];
          bool jok[2], big[2];
#pragma unroll
          for (int u = 0; u < 2; ++u) {
            const int k = lane + 32 * u;
            int ly, cx;
            if (k < NLC) ly = k / (SX / CH), cx = (k % (SX / CH)) * CH;
            else if (k < NLC + NCC) ly = 2 + (k - NLC) / (CL / CH), cx = ((k - NLC) % (CL / CH)) * CH;
            else ly = 2 + (k - NLC - NCC), cx = (CL / CH) * CH;
            const int64_t y = yo + ly, x = xo + cx;
            jok[u] = k < NPP && y >= 0 && y < g.N1 && x >= 0 && x < g.N2;
            big[u] = k < NLC + NCC;
            goff[u] = jok[u] ? y * g.N2 + x : 0;
            soff[u] = ly * SX + cx;
          }
          const bool has2 = lane + 32 < NPP;
          const int qe = no_carry ? plo : phi + 1;
          for (int q = plo + 1; q <= qe; ++q) {
            const int64_t z = i0 + q - 1;
            const bool zok = z >= 0 && z < g.N0;
            const T* zp = src + (zok ? z : 0) * plane;
            T* bq = B(nb, q, 0, 0);
#pragma unroll
            for (int u = 0; u < 2; ++u) {
              if (u == 1 && !has2) break;
              const bool ok = zok && jok[u];
              const T* gp = ok ? zp + goff[u] : src;
              if (big[u]) cp_async16(bq + soff[u], gp, ok);
              else cp_async_small<(CL % CH) * (int)sizeof(T)>(bq + soff[u], gp, ok);
            }
          }
          cp_async_mbar_arrive(&full[nb]);
        }
        __syncwarp();
        if (lane == 0) {
          mbar_arrive(&full[nb]);
          while (!mbar_test_parity(&full[nb], (ph_full >> nb) & 1u))
            if (cons == a - g.a_lo) consume(false);
          if (tr) tr[tk + 1] = gtimer();
          mbar_arrive(&ready[nb]);
        }
        ph_full ^= 1u << nb;
      }
      // publish level a_hi-1 (the last level successors need); a_hi itself is consumed at
      // the next tile's start
      if (lane == 0)
        while (cons < g.a_hi - g.a_lo) consume(true);
      __syncwarp();
      cur = next_tile(cur);
      if (early) {  // buffer a_lo & 1 is idle during level a_hi: stage the next tile now
        stage_first(cur);
        staged = true;
      }
    }
    return;
  }

  // -------------------------------------------------------------------- compute warps
  const Coef<T> cf{(T)g.k0, (T)g.k1};
  const int zg = tid / (NLP * 8), lp = (tid >> 3) % NLP, xq = tid & 7;  // row group (= warp), line pair, col quad
  uint32_t ph_ready = 0u;  // phase parity bit per buffer
  // the successors' carry cells among a thread's outputs: the tile's last 2 lines, last CL columns
  uint32_t cstatic = 0u;
#pragma unroll
  for (int i = 0; i < 2; ++i)
#pragma unroll
    for (int j = 0; j < 4; ++j)
      if ((lp == NLP - 1) || (4 * xq + j >= NX - CL)) cstatic |= 1u << (i * 4 + j);
  while (true) {
    {
      const int b = g.a_lo & 1;
      mbar_wait_sleep(&ready[b], (ph_ready >> b) & 1u);
      ph_ready ^= 1u << b;
    }
    const int64_t S0 = item_s[0];
    if (S0 < 0) break;
    const int64_t q1 = item_s[1], q2 = item_s[2];
    const int64_t i0 = S0 * g.W - g.row_off;
    const int64_t Y0 = (g.S1_lo + q1) * NY, X0 = (g.S2_lo + q2) * NX;
    // every output of every level inside the grid in (y, x)?  (the common case: no masks)
    const bool yx_interior = Y0 - g.a_hi >= 1 && Y0 - g.a_lo + NY - 1 <= g.N1 - 2 &&
                             X0 - SIGMA * g.a_hi + 1 >= 1 && X0 - SIGMA * g.a_lo + NX <= g.N2 - 2;

    for (int a = g.a_lo; a <= g.a_hi; ++a) {
      const int ib = a & 1, ob = (a + 1) & 1;
      if (a > g.a_lo) {
        mbar_wait_sleep(&ready[ib], (ph_ready >> ib) & 1u);
        ph_ready ^= 1u << ib;
      }
      const int rlo = g.lo[a], rhi = g.hi[a];
      const int nr = rhi - rlo + 1;  // rows split into NRG contiguous groups
      const int r0 = rlo + (nr * zg) / NRG, r1 = rlo + (nr * (zg + 1)) / NRG - 1;
      const bool to_smem = a < g.a_hi;  // the last level's values are not read again
      const int64_t yb = Y0 - a + 2 * lp, xb = X0 - SIGMA * a + 1 + 4 * xq;  // output (0, 0)
      // per-output masks (bit i*4+j): interior in (y, x); successors' carry cells
      uint32_t vmask = 0xFFu, cmask = cstatic;
      if (!yx_interior) {
        vmask = 0u;
        cmask = 0u;
#pragma unroll
        for (int i = 0; i < 2; ++i)
#pragma unroll
          for (int j = 0; j < 4; ++j) {
            const bool ok = (yb + i >= 1) && (yb + i <= g.N1 - 2) && (xb + j >= 1) && (xb + j <= g.N2 - 2);
            vmask |= (ok ? 1u : 0u) << (i * 4 + j);
            cmask |= (ok ? 1u : 0u) << (i * 4 + j);
          }
        cmask &= cstatic;
      }
      // rows whose outputs leave in full: r <= flo or r >= fhi (Out planes, final level)
      int flo = -(1 << 30), fhi = 1 << 30;
      if (a == g.a_final || a == g.L - 1) flo = 1 << 30, fhi = -(1 << 30);
      else if (a == g.H) flo = rlo, fhi = rhi;
      else if (a > g.H) flo = rlo + 1, fhi = rhi - 1;
      T* dst = static_cast<T*>(g.buf[(g.tau0 + a + 1) & 1]);
      const bool fast = vmask == 0xFFu && i0 + r0 >= 1 && i0 + r1 <= g.N0 - 2;

      auto load_plane = [&](int q, T (&w)[4][6]) {
#pragma unroll
        for (int l = 0; l < 4; ++l) {
          const T* p = B(ib, q, 2 * lp + l, 4 * xq);
          if constexpr (sizeof(T) == 4) {
            const float4 u = reinterpret_cast<const float4*>(p)[0];
            const float2 v = reinterpret_cast<const float2*>(p)[2];
            w[l][0] = u.x; w[l][1] = u.y; w[l][2] = u.z; w[l][3] = u.w; w[l][4] = v.x; w[l][5] = v.y;
          } else {
#pragma unroll
            for (int i = 0; i < 3; ++i) {
              const double2 u = reinterpret_cast<const double2*>(p)[i];
              w[l][2 * i] = u.x; w[l][2 * i + 1] = u.y;
            }
          }
        }
      };
      auto sweep = [&](auto fast_c) {
        constexpr bool FAST = decltype(fast_c)::value;
        if (r0 > r1) return;
        T* rp = dst + (i0 + r0) * plane + yb * g.N2 + xb;  // global output (0, 0) of row r0
        auto step = [&](int r, const T (&P)[4][6], const T (&C)[4][6], const T (&N)[4][6]) {
          uint32_t okm = vmask;
          if constexpr (!FAST) {
            const int64_t z = i0 + r;
            if (z < 1 || z > g.N0 - 2) okm = 0u;
          }
          T out[2][4];
#pragma unroll
          for (int i = 0; i < 2; ++i)
#pragma unroll
            for (int j = 0; j < 4; ++j) {
              T x[3][3][3];
#pragma unroll
              for (int dy = 0; dy < 3; ++dy)
#pragma unroll
                for (int dx = 0; dx < 3; ++dx) {
                  x[0][dy][dx] = P[i + dy][j + dx];
                  x[1][dy][dx] = C[i + dy][j + dx];
                  x[2][dy][dx] = N[i + dy][j + dx];
                }
              const T v = apply<T, KIND>(x, cf);
              if constexpr (FAST) out[i][j] = v;
              else out[i][j] = ((okm >> (i * 4 + j)) & 1u) ? v : x[1][1][1];
            }
          // into the output buffer: columns CL + 4xq + j (one scalar, one pair, one scalar)
          if (to_smem) {
#pragma unroll
            for (int i = 0; i < 2; ++i) {
              T* p = B(ob, r + 1, 2 + 2 * lp + i, CL + 4 * xq);
              p[0] = out[i][0];
              if constexpr (sizeof(T) == 4) reinterpret_cast<float2*>(p + 1)[0] = make_float2(out[i][1], out[i][2]);
              else { p[1] = out[i][1]; p[2] = out[i][2]; }
              p[3] = out[i][3];
            }
          }
          // copy-out from registers: Out planes / final level in full, else the successors'
          // carries (the window's last 2 lines and last CL columns)
          const bool fullrow = r <= flo || r >= fhi;
          const uint32_t sm_ = fullrow ? okm : (okm & cmask);
          if (FAST && sm_ == 0xFFu && sizeof(T) == 4) {
#pragma unroll
            for (int i = 0; i < 2; ++i) {
              T* q = rp + i * g.N2;
              q[0] = out[i][0];
              reinterpret_cast<float2*>(q + 1)[0] = make_float2(out[i][1], out[i][2]);
              q[3] = out[i][3];
            }
          } else if (sm_) {
#pragma unroll
            for (int i = 0; i < 2; ++i)
#pragma unroll
              for (int j = 0; j < 4; ++j)
                if ((sm_ >> (i * 4 + j)) & 1u) rp[i * g.N2 + j] = out[i][j];
          }
          rp += plane;
        };
        T wa[4][6], wb[4][6], wc[4][6];
        load_plane(r0, wa);      // plane of row r0 - 1
        load_plane(r0 + 1, wb);  // plane of row r0
        int r = r0;
        while (true) {
          load_plane(r + 2, wc);
          step(r, wa, wb, wc);
          if (++r > r1) break;
          load_plane(r + 2, wa);
          step(r, wb, wc, wa);
          if (++r > r1) break;
          load_plane(r + 2, wb);
          step(r, wc, wa, wb);
          if (++r > r1) break;
        }
      };
      if (fast) sweep(std::true_type{});
      else sweep(std::false_type{});
      bar_compute();  // level a complete in ob for both compute warps; their stores issued
      if (tid == 0) mbar_arrive(&done[a & 1]);
    }
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
static bool encode(CUtensorMap* map, void* base, const Fast3DArgs& a, uint32_t bx, uint32_t by) {
  auto fn = get_encode();
  if (!fn) return false;
  cuuint64_t dims[3] = {(cuuint64_t)a.N2, (cuuint64_t)a.N1, (cuuint64_t)a.N0};
  cuuint64_t strides[2] = {(cuuint64_t)a.N2 * sizeof(T), (cuuint64_t)a.N1 * a.N2 * sizeof(T)};
  cuuint32_t box[3] = {bx, by, 1};
  cuuint32_t es[3] = {1, 1, 1};
  const CUtensorMapDataType dt = sizeof(T) == 4 ? CU_TENSOR_MAP_DATA_TYPE_FLOAT32 : CU_TENSOR_MAP_DATA_TYPE_FLOAT64;
  return fn(map, dt, 3, base, dims, strides, box, es, CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE,
            CU_TENSOR_MAP_L2_PROMOTION_L2_128B, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE) == CUDA_SUCCESS;
}

static long long* g_trace = nullptr;
static int64_t g_trace_launch = -1, g_launch_count = 0;
static int g_dbg = 0;  // timing experiments: 1 = skip carries, 2 = skip In planes (wrong results)

template <typename T, int KIND>
cudaError_t launch_t(const Fast3DArgs& a_in, cudaStream_t s) {
  Fast3DArgs a = a_in;
  a.trace = (g_trace && g_launch_count++ == g_trace_launch) ? g_trace : nullptr;
  a.dbg = g_dbg;
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
    cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, fast3d_kernel<T, KIND>, NT, smem);
    grid = sms * (per_sm > 0 ? per_sm : 1);
  }
  Maps m;
  for (int b = 0; b < 2; ++b) {
    if (!encode<T>(&m.plane[b], a.buf[b], a, SX, LY))
      return cudaErrorInvalidValue;
  }
  fast3d_kernel<T, KIND><<<grid, NT, smem, s>>>(a, m);
  return cudaGetLastError();
}

}  // namespace fast3d

void fast3d_set_trace(long long* dev_buf, int64_t launch_index) {
  fast3d::g_trace = dev_buf;
  fast3d::g_trace_launch = launch_index;
  fast3d::g_launch_count = 0;
}

size_t fast3d_smem_bytes(int dtype, int Q) {
  return dtype == 1 ? fast3d::smem_bytes<double>(Q) : fast3d::smem_bytes<float>(Q);
}

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

// Debug hooks (not part of include/stencil.h): trace one 3D launch's per-item timeline;
// timing-experiment modes that skip loads (results are wrong while set).
extern "C" void hexs_debug_fast3d_mode(int mode) { hexs::fast3d::g_dbg = mode; }
extern "C" void hexs_debug_fast3d_trace(void* dev_buf, int64_t launch_index) {
  hexs::fast3d_set_trace(static_cast<long long*>(dev_buf), launch_index);
}
