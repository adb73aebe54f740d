// fdtd.cu -- the specialised sm_100a phase kernel for FDTD-2D (three coupled in-place fields
// ex, ey, hz; statements ey -> ex -> hz per step, tau = 3t + k, Sec. 3.2)
// under the hybrid schedule: hexagonal over (tau, i) with delta0 = 1, delta1 = 1/2 (eqs.
// (10), (12)), classical over j with skew delta1_j = 1 per tau level (eq. (14), reading R14).
//
// Mapping:
//   * one CTA per hexagon S0 of the launch's (T, p) (Sec. 4.1);
//   * j is streamed in chunks of C columns: chunk k at local level a covers
//     j in [kC - a, kC - a + C - 1] -- the classical tile of eq. (14) with w1 = C, u = a --
//     and the chunks run sequentially inside the CTA, as the paper's S1 loop does;
//   * all three fields of the hexagon's rows (plus the halo rows -1 and W the statements
//     read) live in a shared-memory RING of NB blocks of C columns (column j at ring index
//     (j + C) mod NB*C), so the columns a chunk shares with its predecessor (the skewed
//     overlap) are reused on chip -- the inter-tile reuse of Sec. 4.2.2;
//   * the block a chunk will need next is prefetched one chunk ahead with 16-B cp.async
//     (LDGSTS, every address 16-B aligned -- the aligned loads of Sec. 4.2.3), so no warp
//     waits on HBM latency; out-of-grid chunks are zero-filled and never used;
//   * a level is a pure map over its cells (each statement reads only the other fields and
//     its own old value), so one CTA barrier separates levels; four threads per column split
//     the rows (interleaved, so a warp is 32 consecutive columns of one row: conflict-free);
//     the fields are disjoint ring regions (__restrict__), so a thread's row loads are
//     batched ahead of its stores;
//   * a column is final once no later chunk touches it (j < (k+1)C - a_hi): after each chunk
//     its C final columns of every row the hexagon modifies are written back with coalesced
//     stores -- the interleaved copy-out of Sec. 4.2.1.
#include <cstdint>
#include <type_traits>

#include "../stencil_ops.cuh"
#include "devcache.h"
#include "launch.h"
#include "tma.cuh"

namespace hexs {
namespace fdtd {

#ifndef HEXS_FDTD_C
#define HEXS_FDTD_C 64
#endif
constexpr int C = HEXS_FDTD_C;  // columns per chunk (= ring block)
#ifndef HEXS_FDTD_BLOCKROWS
#define HEXS_FDTD_BLOCKROWS 1  // ey / hz levels: contiguous row blocks per thread (register reuse)
#endif
#ifndef HEXS_FDTD_PAIR
#define HEXS_FDTD_PAIR 1  // ey and ex of a time step in one barrier interval (unrolled kernel)
#endif
#ifndef HEXS_FDTD_UNROLL
#define HEXS_FDTD_UNROLL 1  // 0: the run-time-row kernel for every tile
#endif
#ifndef HEXS_FDTD_RING
#define HEXS_FDTD_RING 4  // 3 (3 CTAs/SM, one-chunk prefetch) measured 226 -> 192 GUp/s
#endif
// Ring of NB blocks of C columns: 4 (prefetch two chunks ahead, 2 CTAs/SM) or 3 (one chunk
// ahead; 3 CTAs/SM fit the shared memory).  Ring column of grid column j: (j + C) mod RC.
constexpr int NB = HEXS_FDTD_RING;
constexpr int RC = NB * C;    // ring columns
__device__ __forceinline__ int ring_col(int j) { return (j + C) % RC; }  // j >= -C
#ifndef HEXS_FDTD_RP
#define HEXS_FDTD_RP 4  // 2 (3 CTAs/SM) measured 228 -> 197 GUp/s
#endif
constexpr int RP = HEXS_FDTD_RP;  // threads per column (row parts, rows interleaved)
#ifndef HEXS_FDTD_MINB
#define HEXS_FDTD_MINB ((RP == 2 || NB == 3) ? 3 : 2)
#endif
constexpr int MINB = HEXS_FDTD_MINB;  // resident CTAs per SM (shared memory: 3 fields x ring)
constexpr int NT = RP * C;

template <typename T>
size_t smem_bytes(int W) {
  // three fields' ring rows, plus (unrolled kernel) RP + 2 padding rows that the row slots past a
  // level's last row may read (their stores are predicated off)
  return ((size_t)3 * (W + 2) * RC + (size_t)(RP + 2) * RC) * sizeof(T);
}

__device__ __forceinline__ void cp_async16(void* dst, const void* src, bool valid) {
  asm volatile("cp.async.cg.shared.global [%0], [%1], 16, %2;" ::"r"((uint32_t)__cvta_generic_to_shared(dst)),
               "l"(src), "r"(valid ? 16 : 0)
               : "memory");
}
__device__ __forceinline__ void cp_async_commit() { asm volatile("cp.async.commit_group;" ::: "memory"); }
template <int N>
__device__ __forceinline__ void cp_async_wait() {
  asm volatile("cp.async.wait_group %0;" ::"n"(N) : "memory");
}

__device__ __forceinline__ int64_t max64(int64_t a, int64_t b) { return a > b ? a : b; }
__device__ __forceinline__ int64_t min64(int64_t a, int64_t b) { return a < b ? a : b; }

// Compile-time hexagon of the FDTD schedule (delta0 = 1, delta1 = 1/2, reading R15): the row
// range of level a, SURVEY 8(a)'s closed form of eqs. (6)-(13) with F0 = h, F1 = floor(h/2),
// e1 = 1/2, e0 = 0.  The host checks it against the plan's rows before choosing the unrolled
// kernel (fdtd_unrolled_ok).
template <int H, int W0> struct FHex {
  static constexpr int L = 2 * H + 2, F0 = H, F1 = H / 2, W = 2 * W0 + 2 + F0 + F1;
  __host__ __device__ static constexpr int cdiv2(int x) { return x >= 0 ? (x + 1) / 2 : -((-x) / 2); }  // ceil(x / 2)
  __host__ __device__ static constexpr int fdiv2(int x) { return x >= 0 ? x / 2 : -((-x + 1) / 2); }   // floor(x / 2)
  __host__ __device__ static constexpr int lo(int a) {
    const int l1 = a - (2 * H + 1) + F0, l2 = cdiv2(H - 1 - a);
    return l1 > l2 ? l1 : l2;
  }
  __host__ __device__ static constexpr int hi(int a) {
    const int h1 = fdiv2(2 * H + 1 - a) + F0 + W0, h2 = a - H + F0 + F1 + W0;
    return h1 < h2 ? h1 : h2;
  }
};
// predicated shared store (no select, no branch): the unrolled kernel's masked row slots
__device__ __forceinline__ void sts_if(bool p, float* a, float v) {
  asm volatile("{\n.reg .pred q;\nsetp.ne.b32 q, %0, 0;\n@q st.shared.f32 [%1], %2;\n}\n" ::"r"((int)p), "r"(smem_u32(a)),
               "f"(v));
}
__device__ __forceinline__ void sts_if(bool p, double* a, double v) {
  asm volatile("{\n.reg .pred q;\nsetp.ne.b32 q, %0, 0;\n@q st.shared.f64 [%1], %2;\n}\n" ::"r"((int)p), "r"(smem_u32(a)),
               "d"(v));
}
template <int A, int N, class F>
__device__ __forceinline__ void static_for(F&& f) {
  if constexpr (A < N) {
    f(std::integral_constant<int, A>{});
    static_for<A + 1, N>(f);
  }
}

// fields: 0 = ex, 1 = ey, 2 = hz (the order of FdtdArgs::f); statement k: 0 ey, 1 ex, 2 hz
// UH > 0: the levels and their row ranges are compile-time (hexagon (UH, UW0), launches start
// at tau0 = 0 mod 3): every level is unrolled with its rows spread over the RP row parts as
// immediate shared-memory offsets -- no per-level table reads, no run-time trip counts.
// UH = 0: any (h, w0), rows from the kernel arguments.
template <typename T, int UH, int UW0>
__global__ void __launch_bounds__(NT, MINB) fdtd_kernel(const __grid_constant__ FdtdArgs g) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  T* ring = reinterpret_cast<T*>(smem_raw);
  const int W = g.W, R = W + 2;  // smem rows: b in [-1, W] at b + 1
  T* const F[3] = {static_cast<T*>(g.f[0]), static_cast<T*>(g.f[1]), static_cast<T*>(g.f[2])};  // ex ey hz
  const Coef<T> cf{(T)g.k0, (T)g.k1};
  const int tid = threadIdx.x;
  const int64_t N0 = g.N0, N1 = g.N1;
  const int64_t S0 = g.S0_lo + blockIdx.x;
  const int64_t i0 = S0 * W - g.row_off;  // i of local row b = 0

  // rows each field is modified at (write-back range), clipped to the grid
  int mlo[3] = {1 << 30, 1 << 30, 1 << 30}, mhi[3] = {-1, -1, -1};
  for (int a = g.a_lo; a <= g.a_hi; ++a) {
    const int k = (int)((g.tau0 + a) % 3), f = k == 0 ? 1 : (k == 1 ? 0 : 2);
    mlo[0] = f == 0 ? min(mlo[0], g.lo[a]) : mlo[0];
    mhi[0] = f == 0 ? max(mhi[0], g.hi[a]) : mhi[0];
    mlo[1] = f == 1 ? min(mlo[1], g.lo[a]) : mlo[1];
    mhi[1] = f == 1 ? max(mhi[1], g.hi[a]) : mhi[1];
    mlo[2] = f == 2 ? min(mlo[2], g.lo[a]) : mlo[2];
    mhi[2] = f == 2 ? max(mhi[2], g.hi[a]) : mhi[2];
  }
  const int bmin = (int)max64(0, -i0), bmax = (int)min64(W - 1, N0 - 1 - i0);
#pragma unroll
  for (int f = 0; f < 3; ++f) {
    mlo[f] = max(mlo[f], bmin);
    mhi[f] = min(mhi[f], bmax);
  }

  // Stage ring block `blk` (columns [(blk-1)C, blk C)) of all fields and rows.  Element
  // e = tid + NT*u: 16-B chunk c = e % NCH is fixed per thread (NT % NCH == 0), the
  // (field, row) index advances by NT / NCH per step.
  constexpr int CH = 16 / sizeof(T);  // elements per 16-B chunk
  constexpr int NCH = C / CH;         // chunks per row block
  constexpr int RSTEP = NT / NCH;
  static_assert(NT % NCH == 0, "staging walk");
  const int sc = tid % NCH;
  // A thread stages the same (field, row) pairs for every block: fr = tid/NCH + u*RSTEP.
  // Their row base pointers (NULL outside the grid) are computed once.
  constexpr int MAXU = (3 * 42 + RSTEP - 1) / RSTEP;  // ceil(3 (W+2) / RSTEP) for W <= 40 (fdtd_variant)
  const T* rowp[MAXU];
  int soff[MAXU];
#pragma unroll
  for (int u = 0; u < MAXU; ++u) {
    const int fr = tid / NCH + u * RSTEP;
    const int f = fr / R, rb = fr - f * R;
    const int64_t i = i0 + rb - 1;
    const bool ok = fr < 3 * R && i >= 0 && i < N0;
    T* const fb = f == 0 ? F[0] : (f == 1 ? F[1] : F[2]);
    rowp[u] = ok ? fb + i * N1 : nullptr;
    soff[u] = fr < 3 * R ? (f * R + rb) * RC : -1;
  }
  auto stage = [&](int blk) {
    const int j = (blk - 1) * C + sc * CH;
    const bool jok = j >= 0 && j < N1;
    const int cj = ring_col(j);
#pragma unroll
    for (int u = 0; u < MAXU; ++u) {
      if (soff[u] < 0) continue;
      const bool ok = jok && rowp[u] != nullptr;
      cp_async16(ring + soff[u] + cj, ok ? rowp[u] + j : F[0], ok);
    }
    cp_async_commit();
  };

  const int nlev = g.a_hi - g.a_lo + 1;
  const int k_last = (int)((N1 - 1 + g.a_hi) / C);
  for (int blk = 0; blk < NB - 1; ++blk) stage(blk);
  const int col = tid & (C - 1), rpar = tid / C;  // column, row part
  const int zrr = (int)(-i0) - rpar, nrr = (int)(N0 - 1 - i0) - rpar;  // (unrolled kernel) edge rows
  T* const rex = ring + (size_t)(0 * R + 1) * RC;  // row b of a field at r.. + b * RC + ring column
  T* const rey = ring + (size_t)(1 * R + 1) * RC;
  T* const rhz = ring + (size_t)(2 * R + 1) * RC;
  for (int k = 0; k <= k_last; ++k) {
    stage(k + NB - 1);     // a later chunk's new block (ring slot of block k-1, written back)
    cp_async_wait<1>();    // every block but the newest has landed
    __syncthreads();
    if constexpr (UH > 0) {
      using HX = FHex<UH, UW0>;
      // all rows of the three fields hold (b + 1) * RC + ring column offsets from a per-level base
      static_for<0, HX::L>([&](auto a_c) {
        constexpr int a = decltype(a_c)::value;
        constexpr int st = a % 3, LO = HX::lo(a), HI = HX::hi(a);
        constexpr int M = (HI - LO + RP) / RP;  // row slots per thread (the last one predicated)
        if (a < g.a_lo || a > g.a_hi) return;   // time-cut launches (CTA-uniform)
        // Which slots store: cells outside the grid may compute anything -- they are never
        // written back, and no in-grid cell reads one (ey[i] reads hz[i-1] for i >= 1, ex[j]
        // hz[j-1] for j >= 1, hz[i][j] ex[j+1] / ey[i+1] inside the grid; staging zero-fills
        // them) -- so only the in-grid cells a statement never updates (ey row 0, ex column 0,
        // hz row N0-1 and column N1-1, the oracle's loop bounds) and the row slots past the
        // level's last row are masked: one compare per slot and a predicated store.
        const int j = k * C - a + col;
        const int cj = (int)((unsigned)(j + C) % (unsigned)RC);
        bool lvok = true;  // column / last-slot conditions of this level
        if constexpr (st == 1) lvok = j != 0;
        if constexpr (st == 2) lvok = j != (int)N1 - 1;
        constexpr int RR = HX::W + 2;  // ring rows per field (compile-time: immediate offsets)
        T* const fb = ring + (LO + 1 + rpar) * RC + cj;  // field 0 (ex), row LO + rpar
        constexpr int LASTLIM = HI - LO - RP * (M - 1);  // the last slot exists for rpar <= LASTLIM
        const bool lastok = rpar <= LASTLIM;
        // row b = LO + RP m + rpar is global row 0 (ey) / N0-1 (hz) iff LO + RP m == zrr / nrr:
        // one compare with an immediate per slot
        auto slot_ok = [&](int m) {
          bool ok = lvok && (m < M - 1 || lastok);
          if (st == 0) ok = ok && (LO + RP * m != zrr);
          if (st == 2) ok = ok && (LO + RP * m != nrr);
          return ok;
        };
        // Block rows (HEXS_FDTD_BLOCKROWS): thread rpar takes rows LO + rpar M + m, so the
        // row neighbours a statement reads (hz[i-1] for ey, ey[i+1] for hz) are the previous /
        // next slot's own loads -- one shared load per slot fewer for ey and hz
        const int nrow = HI - LO + 1 - rpar * M;  // valid slots m < nrow
        T* const fbb = ring + (LO + 1 + rpar * M) * RC + cj;
        const int zb = zrr + rpar - rpar * M, nb = nrr + rpar - rpar * M;  // edge rows as LO + m
        if constexpr (HEXS_FDTD_BLOCKROWS && st == 0) {
          T hprev = fbb[(2 * RR - 1) * RC];  // hz[b-1] of slot 0
#pragma unroll
          for (int m = 0; m < M; ++m) {
            T* pe = fbb + (RR + m) * RC;
            const T hb = fbb[(2 * RR + m) * RC];
            const T v = fdtd_ey<T>(*pe, hb, hprev, cf);
            hprev = hb;
            sts_if(lvok && m < nrow && LO + m != zb, pe, v);
          }
        } else if constexpr (HEXS_FDTD_BLOCKROWS && st == 2) {
          const int dp = cj == RC - 1 ? 1 - RC : 1;  // column j+1 in the ring
          T enext = fbb[RR * RC];  // ey[b] of slot 0
#pragma unroll
          for (int m = 0; m < M; ++m) {
            T* ph = fbb + (2 * RR + m) * RC;
            const T* px = fbb + m * RC;
            const T eb = enext;
            enext = fbb[(RR + m + 1) * RC];  // ey[b+1] = the next slot's ey[b]
            const T v = fdtd_hz<T>(*ph, px[dp], px[0], enext, eb, cf);
            sts_if(lvok && m < nrow && LO + m != nb, ph, v);
          }
        } else if constexpr (st == 0) {  // ey[i][j] -= ce * (hz[i][j] - hz[i-1][j])
#pragma unroll
          for (int m = 0; m < M; ++m) {
            T* pe = fb + (RR + RP * m) * RC;
            const T* ph = fb + (2 * RR + RP * m) * RC;
            const T v = fdtd_ey<T>(*pe, ph[0], ph[-RC], cf);
            sts_if(slot_ok(m), pe, v);
          }
        } else if constexpr (st == 1) {  // ex[i][j] -= ce * (hz[i][j] - hz[i][j-1])
          const int dm = cj == 0 ? RC - 1 : -1;  // column j-1 in the ring
#pragma unroll
          for (int m = 0; m < M; ++m) {
            T* px = fb + (RP * m) * RC;
            const T* ph = fb + (2 * RR + RP * m) * RC;
            const T v = fdtd_ex<T>(*px, ph[0], ph[dm], cf);
            sts_if(slot_ok(m), px, v);
          }
        } else {  // hz[i][j] -= ch * (((ex[i][j+1] - ex[i][j]) + ey[i+1][j]) - ey[i][j])
          const int dp = cj == RC - 1 ? 1 - RC : 1;  // column j+1 in the ring
#pragma unroll
          for (int m = 0; m < M; ++m) {
            T* ph = fb + (2 * RR + RP * m) * RC;
            const T* px = fb + (RP * m) * RC;
            const T* pe = fb + (RR + RP * m) * RC;
            const T v = fdtd_hz<T>(*ph, px[dp], px[0], pe[RC], pe[0], cf);
            sts_if(slot_ok(m), ph, v);
          }
        }
        // ey (tau = 3t) and ex (3t + 1) read only hz of step t-1 and write different fields:
        // one barrier interval holds both (2 barriers per time step instead of 3)
        if constexpr (st != 0 || !HEXS_FDTD_PAIR) {
          __syncthreads();
        } else {
          if (a == g.a_hi) __syncthreads();  // a launch's last level: before the write-back
        }
      });
    } else {
    int st = (int)((g.tau0 + g.a_lo) % 3);
    for (int l = 0; l < nlev; ++l, st = st == 2 ? 0 : st + 1) {
      // level parameters from the kernel arguments (constant bank), clipped to the grid and the
      // statement's domain (oracle/oracle.c: ey i >= 1; ex j >= 1; hz i < N0-1, j < N1-1)
      const int a = g.a_lo + l;
      const int blo = max(g.lo[a], st == 0 ? (int)(1 - i0) : (int)(-i0));
      const int bhi = min(g.hi[a], st == 2 ? (int)(N0 - 2 - i0) : (int)(N0 - 1 - i0));
      const int j = k * C - a + col;
      if (j >= (st == 1 ? 1 : 0) && j <= (st == 2 ? (int)N1 - 2 : (int)N1 - 1)) {
        // 32-bit shared-memory element offsets (one IADD per row step instead of 64-bit
        // pointer arithmetic); row b of field f at (f*R + b + 1) * RC + ring column
        const int cj = ring_col(j);
        const int b0 = blo + rpar;
        int o = (b0 + 1) * RC + cj;  // row b0 of a field, relative to its first row
        constexpr int STEP = RP * RC;
        if (st == 0) {  // ey[i][j] -= ce * (hz[i][j] - hz[i-1][j])
#pragma unroll 4
          for (int b = b0; b <= bhi; b += RP, o += STEP) {
            T* pe = ring + R * RC + o;
            const T* ph = ring + 2 * R * RC + o;
            *pe = fdtd_ey<T>(*pe, ph[0], ph[-RC], cf);
          }
        } else if (st == 1) {  // ex[i][j] -= ce * (hz[i][j] - hz[i][j-1])
          const int dm = ring_col(j - 1) - cj;  // column j-1 relative to j in the ring
#pragma unroll 4
          for (int b = b0; b <= bhi; b += RP, o += STEP) {
            T* px = ring + o;
            const T* ph = ring + 2 * R * RC + o;
            *px = fdtd_ex<T>(*px, ph[0], ph[dm], cf);
          }
        } else {  // hz[i][j] -= ch * (((ex[i][j+1] - ex[i][j]) + ey[i+1][j]) - ey[i][j])
          const int dp = ring_col(j + 1) - cj;  // column j+1 relative to j in the ring
#pragma unroll 4
          for (int b = b0; b <= bhi; b += RP, o += STEP) {
            T* ph = ring + 2 * R * RC + o;
            const T* px = ring + o;
            const T* pe = ring + R * RC + o;
            *ph = fdtd_hz<T>(*ph, px[dp], px[0], pe[RC], pe[0], cf);
          }
        }
      }
      __syncthreads();
    }
    }
    // write back the columns no later chunk touches: [kC - a_hi, (k+1)C - a_hi), or all
    // remaining columns after the last chunk
    const int wlo = max(0, k * C - g.a_hi);
    const int whi = (k == k_last) ? (int)N1 - 1 : (k + 1) * C - g.a_hi - 1;
    for (int j = k * C - g.a_hi + col; j <= whi; j += C) {
      if (j < wlo) continue;
      const int cj = ring_col(j);
#pragma unroll
      for (int f = 0; f < 3; ++f) {
        const int b0 = mlo[f] + rpar;
        const T* sp = (f == 0 ? rex : (f == 1 ? rey : rhz)) + cj + b0 * RC;
        T* gp = F[f] + ((i0 + b0) * N1 + j);
        const int64_t gstep = RP * N1;
        for (int b = b0; b <= mhi[f]; b += RP, sp += RP * RC, gp += gstep) *gp = *sp;
      }
    }
    __syncthreads();  // the write-back reads ring slots the next stage() overwrites
  }
  cp_async_wait<0>();
}

// the compiled unrolled hexagon (the default FDTD tile, plan.cpp) applies when the plan's
// rows are exactly its rows and the launch starts a time step (statement order ey, ex, hz)
constexpr int kUH = 11, kUW0 = 5;
bool unrolled_ok(const FdtdArgs& a) {
  using HX = FHex<kUH, kUW0>;
  if (a.W != HX::W || a.tau0 % 3 != 0) return false;
  for (int q = 0; q < HX::L; ++q)
    if (a.lo[q] != HX::lo(q) || a.hi[q] != HX::hi(q)) return false;
  return true;
}

template <typename T>
cudaError_t launch_t(const FdtdArgs& a, int grid, cudaStream_t s) {
  // per device: opt in once to the largest ring any plan can ask for (fdtd_variant caps it)
  static DeviceMemo<int> attr;
  const size_t smem = smem_bytes<T>(a.W);
  if (smem > 200 * 1024) return cudaErrorInvalidValue;
  int done = 0;
  cudaError_t e = attr.get(&done, [](int, int* v) {
    *v = 1;
    cudaError_t r = cudaFuncSetAttribute(fdtd_kernel<T, 0, 0>, cudaFuncAttributeMaxDynamicSharedMemorySize, 200 * 1024);
    if (r == cudaSuccess)
      r = cudaFuncSetAttribute(fdtd_kernel<T, kUH, kUW0>, cudaFuncAttributeMaxDynamicSharedMemorySize, 200 * 1024);
    return r;
  });
  if (e != cudaSuccess) return e;
  if (HEXS_FDTD_UNROLL && unrolled_ok(a))
    fdtd_kernel<T, kUH, kUW0><<<grid, NT, smem, s>>>(a);
  else
    fdtd_kernel<T, 0, 0><<<grid, NT, smem, s>>>(a);
  return cudaGetLastError();
}

}  // namespace fdtd

size_t fdtd_smem_bytes(int dtype, int W) {
  return dtype == 1 ? fdtd::smem_bytes<double>(W) : fdtd::smem_bytes<float>(W);
}

int fdtd_ctas_per_sm() { return fdtd::MINB; }

cudaError_t launch_fdtd(int variant, const FdtdArgs& a, int grid, cudaStream_t s) {
  switch (variant) {
    case 0: return fdtd::launch_t<float>(a, grid, s);
    case 1: return fdtd::launch_t<double>(a, grid, s);
    default: return cudaErrorInvalidValue;
  }
}

}  // namespace hexs
