// ablation.cu -- B200 replay of the paper's optimisation ablation (Sec. 6.2, Table 4 / Table 5,
// PAPER.md:986-1067): ONE hybrid-tiled 3D phase kernel, six memory strategies selected at
// compile time, everything else (schedule, tile sizes, thread mapping, work order) identical.
//
//   (a) no shared memory: every operand from global memory, every result to global memory
//       (PAPER.md:1003-1004);
//   (b) shared memory: "for each tile we first copy all required values into shared memory,
//       we then perform the computation within shared memory and finally we copy the results
//       back";
//   (c) (b) + interleaved copy-out: results are stored as soon as they are computed
//       (PAPER.md:1007-1009);
//   (d) (c) + aligned loads: the tiles are translated in the data space so the copy-in box
//       starts on a 128-B line (Sec. 4.2.3's translation offset);
//   (e) (d) + static reuse: every global value has a fixed shared-memory home (x modulo 64), so
//       the next classical tile finds the overlap where the previous one left it and loads only
//       its new 32 columns;
//   (f) (d) + dynamic reuse: tile-relative shared memory plus an explicit copy phase between two
//       tiles that moves the overlap to where the next tile expects it.
//
// Setup of Table 4: CTA of 1 x 10 x 32 threads, classical tiles w1 = 10
// (y) x w2 = 32 (x), hexagons over z (default h = 2, w0 = 7).  One thread owns one (y, x)
// column of a classical tile and walks the hexagon's rows of each level (dimension 0 maps to
// one thread, "iteration i is mapped to thread i mod Ti").
//
// Work mapping (B200): the paper runs all classical tiles of a hexagon sequentially in one
// CTA.  Reuse (e, f) needs consecutive x tiles in the same CTA, so a work item is one
// (hexagon S0, y tile S1) row whose x tiles S2 run in order; rows of the same hexagon form a
// pipeline -- tile (S1, S2) starts once row S1-1 has completed tile S2+1 (its y-halo, i.e. the
// part of the copy-in box produced by row S1-1, is final; eq. (14)'s skew makes every other
// dependence point to an earlier tile of the same row).  Persistent CTAs take rows in
// (S1, S0) order, so every wait is on an earlier ticket and the resident grid cannot deadlock.
//
// Shared memory holds both ping-pong parities of the tile's box in global coordinates:
// rows [-1, W] of the hexagon, y in [B1 - a_hi - 1, B1 + 11 - a_lo), x in [B2 - a_hi - 1,
// B2 + 33 - a_lo) -- the union over the tile's levels of the skewed tile plus its radius-1
// halo (the "over-approximated box").  Reading the In values of all levels
// at the tile's start is valid: the schedule produced them before the tile, and no tile
// overwrites one of them before this tile has read it in the canonical order (ping-pong WAR,
// PAPER.md:146-148).  A point's value is stored to global memory iff the tile does not
// recompute the same point two levels later (then that later value is the one other tiles read).
#include "../stencil_ops.cuh"
#include "devcache.h"
#include "launch.h"

namespace hexs {

namespace {

constexpr int kAblThreads = kAblW1 * kAblW2;  // 1 x 10 x 32 (Table 4)

__device__ __forceinline__ int abl_ld_acquire(const int* p) {
  int v;
  asm volatile("ld.acquire.gpu.global.b32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void abl_st_release(int* p, int v) {
  asm volatile("st.release.gpu.global.b32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}

// One point from an accessor at(dz, dy, dx): the operand order of point_from_memory (and of
// the oracle), so every configuration is bit-identical to the others.
template <int KIND, typename At>
__device__ __forceinline__ float abl_point(At at, const Coef<float>& k) {
  if constexpr (KIND == K_STAR3D7) {
    return star3d7<float>(at(0, 0, 0), at(0, -1, 0), at(0, 1, 0), at(0, 0, -1), at(0, 0, 1), at(-1, 0, 0),
                          at(1, 0, 0), k);
  } else if constexpr (KIND == K_GRADIENT3D) {
    return gradient3d<float>(at(0, 0, 0), at(0, -1, 0), at(0, 1, 0), at(0, 0, -1), at(0, 0, 1), at(-1, 0, 0),
                             at(1, 0, 0), k);
  } else {
    float acc = at(-1, -1, -1);
#pragma unroll
    for (int q = 1; q < 27; ++q) acc = acc + at(q / 9 - 1, (q / 3) % 3 - 1, q % 3 - 1);
    return k.k0 * acc;
  }
}

template <int CFG, int KIND>
__global__ void __launch_bounds__(kAblThreads, 1) ablation_kernel(const __grid_constant__ AblArgs g) {
  extern __shared__ float smem[];
  __shared__ int item_s;
  constexpr bool kSmem = CFG != ABL_A;
  constexpr bool kCircular = CFG == ABL_E;
  const int tid = threadIdx.x, ty = tid / kAblW2, tx = tid % kAblW2;
  const int warp = tid / 32, lane = tid % 32;
  const Coef<float> k{(float)g.k0, (float)g.k1};
  const int64_t N0 = g.N0, N1 = g.N1, N2 = g.N2, s0 = N1 * N2, s1 = N2;
  float* const gb0 = static_cast<float*>(g.buf[0]);
  float* const gb1 = static_cast<float*>(g.buf[1]);
  auto gbuf = [&](int par) { return par ? gb1 : gb0; };  // selects, not a local array
  const int RB = g.W + 2, YB = g.YB, XB = g.XB, XP = g.XP;
  const int plane = YB * XP;
  float* const sm0 = smem;
  float* const sm1 = smem + (size_t)RB * plane;
  auto sb = [&](int par) { return par ? sm1 : sm0; };
  const int nS0 = (int)(g.S0_hi - g.S0_lo + 1);
  const int n_items = nS0 * g.n1;

  while (true) {
    if (tid == 0) item_s = (int)atomicAdd(g.counter, 1u);
    __syncthreads();
    const int it = item_s;
    __syncthreads();
    if (it >= n_items) break;
    const int q1 = it / nS0;
    const int64_t S0 = g.S0_lo + it % nS0;
    const int64_t i0 = S0 * g.W - g.row_off;  // z of hexagon row b = 0
    const int64_t B1 = (g.S1_lo + q1) * kAblW1 + g.ctrans1;  // y base of level a: B1 - a (eq. (14))
    const int64_t Y0 = B1 - g.a_hi - 1;
    int* prog = g.progress + it;  // progress[q1][S0]: completed x tiles of this row
    const int* prev = q1 > 0 ? g.progress + it - nS0 : nullptr;
    for (int q2 = 0; q2 < g.n2; ++q2) {
      const int64_t B2 = (g.S2_lo + q2) * kAblW2 + g.ctrans2;
      const int64_t X0 = B2 - g.a_hi - 1;
      auto xs = [&](int64_t gx) -> int { return kCircular ? (int)(gx & 63) : (int)(gx - X0); };
      if (tid == 0 && prev) {
        const int need = q2 + 2 < g.n2 ? q2 + 2 : g.n2;
        while (abl_ld_acquire(prev) < need) __nanosleep(32);
        __threadfence();
      }
      __syncthreads();
      if constexpr (kSmem) {
        int c_lo = 0;  // first box column to load from global memory
        if constexpr (CFG == ABL_F) {
          if (q2 > 0) {  // explicit copy phase: columns [32, XB) -> [0, XB - 32)
            const int nc = XB - kAblW2;
            for (int par = 0; par < 2; ++par)
              for (int line = warp; line < RB * YB; line += kAblThreads / 32)
                if (lane < nc) {
                  float* L = sb(par) + (line / YB) * plane + (line % YB) * XP;
                  L[lane] = L[lane + kAblW2];
                }
            __syncthreads();
            c_lo = nc;
          }
        } else if constexpr (CFG == ABL_E) {
          if (q2 > 0) c_lo = XB - kAblW2;  // the overlap stays at its static home
        }
        // copy-in: one warp per box line, lanes along x (coalesced)
        for (int par = 0; par < 2; ++par) {
          const float* G = gbuf(par);
          for (int line = warp; line < RB * YB; line += kAblThreads / 32) {
            const int rb = line / YB, yb = line % YB;
            const int64_t gz = i0 + rb - 1, gy = Y0 + yb;
            if (gz < 0 || gz >= N0 || gy < 0 || gy >= N1) continue;
            float* L = sb(par) + rb * plane + yb * XP;
            const float* GL = G + gz * s0 + gy * s1;
            for (int c = c_lo + lane; c < XB; c += 32) {
              const int64_t gx = X0 + c;
              if (gx >= 0 && gx < N2) L[xs(gx)] = GL[gx];
            }
          }
        }
        __syncthreads();
      }
      // the 2h+2 levels of the tile (tile-local time, sequential)
      for (int a = g.a_lo; a <= g.a_hi; ++a) {
        const int src = (int)((g.tau0 + a) & 1), dst = src ^ 1;
        const int64_t y = B1 - a + ty, x = B2 - a + tx;
        const bool col_in = y >= 1 && y <= N1 - 2 && x >= 1 && x <= N2 - 2;
        // same (y, x) column again two levels later (same parity): the later value is the one
        // other tiles read, this one is not stored
        const bool col_again = a + 2 <= g.a_hi && ty < kAblW1 - 2 && tx < kAblW2 - 2;
        const int lo2 = col_again ? g.lo[a + 2] : 1, hi2 = col_again ? g.hi[a + 2] : 0;
        if (col_in) {
          for (int b = g.lo[a]; b <= g.hi[a]; ++b) {
            const int64_t z = i0 + b;
            if (z < 1 || z > N0 - 2) continue;
            const int64_t gp = z * s0 + y * s1 + x;
            if constexpr (!kSmem) {
              const float* A = gbuf(src);
              const float v =
                  abl_point<KIND>([&](int dz, int dy, int dx) { return A[gp + dz * s0 + dy * s1 + dx]; }, k);
              gbuf(dst)[gp] = v;
            } else {
              const float* A = sb(src);
              const int rb = b + 1, yb = (int)(y - Y0);
              const float v = abl_point<KIND>(
                  [&](int dz, int dy, int dx) { return A[(rb + dz) * plane + (yb + dy) * XP + xs(x + dx)]; }, k);
              sb(dst)[rb * plane + yb * XP + xs(x)] = v;
              if constexpr (CFG != ABL_B)
                if (b < lo2 || b > hi2) gbuf(dst)[gp] = v;  // interleaved copy-out
            }
          }
        }
        __syncthreads();
      }
      if constexpr (CFG == ABL_B) {  // separate copy-out phase: the same values, after compute
        for (int a = g.a_lo; a <= g.a_hi; ++a) {
          const int dst = (int)((g.tau0 + a + 1) & 1);
          const int64_t y = B1 - a + ty, x = B2 - a + tx;
          if (!(y >= 1 && y <= N1 - 2 && x >= 1 && x <= N2 - 2)) continue;
          const bool col_again = a + 2 <= g.a_hi && ty < kAblW1 - 2 && tx < kAblW2 - 2;
          const int lo2 = col_again ? g.lo[a + 2] : 1, hi2 = col_again ? g.hi[a + 2] : 0;
          for (int b = g.lo[a]; b <= g.hi[a]; ++b) {
            const int64_t z = i0 + b;
            if (z < 1 || z > N0 - 2 || (b >= lo2 && b <= hi2)) continue;
            gbuf(dst)[z * s0 + y * s1 + x] = sb(dst)[(b + 1) * plane + (int)(y - Y0) * XP + xs(x)];
          }
        }
        __syncthreads();
      }
      if (tid == 0) {
        __threadfence();
        abl_st_release(prog, q2 + 1);
      }
    }
  }
}

template <int CFG, int KIND>
cudaError_t launch_cfg(const AblArgs& a, cudaStream_t s) {
  auto kern = ablation_kernel<CFG, KIND>;
  const size_t smem = ablation_smem_bytes(CFG, a.W, a.YB, a.XP);
  static DeviceMemo<int> attr_memo;  // dynamic shared memory opt-in, once per device
  int sms = 0;
  cudaError_t e = attr_memo.get(&sms, [&](int dev, int* v) {
    int optin = 0;
    cudaFuncAttributes fa{};
    cudaError_t r = cudaDeviceGetAttribute(&optin, cudaDevAttrMaxSharedMemoryPerBlockOptin, dev);
    if (r == cudaSuccess) r = cudaFuncGetAttributes(&fa, kern);
    if (r == cudaSuccess)
      r = cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, optin - (int)fa.sharedSizeBytes);
    if (r != cudaSuccess) return r;
    return cudaDeviceGetAttribute(v, cudaDevAttrMultiProcessorCount, dev);
  });
  if (e != cudaSuccess) return e;
  // persistent grid: every CTA resident (the row pipeline's waits need it)
  int per_sm = 0;
  if ((e = cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, kern, kAblThreads, smem)) != cudaSuccess) return e;
  if (per_sm < 1) return cudaErrorInvalidConfiguration;
  const int64_t items = (a.S0_hi - a.S0_lo + 1) * (int64_t)a.n1;
  const int64_t slots = (int64_t)per_sm * sms;
  kern<<<(int)(items < slots ? items : slots), kAblThreads, smem, s>>>(a);
  return cudaGetLastError();
}

template <int KIND>
cudaError_t launch_kind(int cfg, const AblArgs& a, cudaStream_t s) {
  switch (cfg) {
    case ABL_A: return launch_cfg<ABL_A, KIND>(a, s);
    case ABL_B: return launch_cfg<ABL_B, KIND>(a, s);
    case ABL_C: return launch_cfg<ABL_C, KIND>(a, s);
    case ABL_D: return launch_cfg<ABL_D, KIND>(a, s);
    case ABL_E: return launch_cfg<ABL_E, KIND>(a, s);
    case ABL_F: return launch_cfg<ABL_F, KIND>(a, s);
    default: return cudaErrorInvalidValue;
  }
}

}  // namespace

size_t ablation_smem_bytes(int cfg, int W, int YB, int XP) {
  if (cfg == ABL_A) return 0;
  return 2 * (size_t)(W + 2) * YB * XP * sizeof(float);
}

cudaError_t launch_ablation(int cfg, int kind, const AblArgs& a, cudaStream_t s) {
  switch (kind) {
    case K_STAR3D7: return launch_kind<K_STAR3D7>(cfg, a, s);
    case K_BOX3D27: return launch_kind<K_BOX3D27>(cfg, a, s);
    case K_GRADIENT3D: return launch_kind<K_GRADIENT3D>(cfg, a, s);
    default: return cudaErrorInvalidValue;
  }
}

}  // namespace hexs
