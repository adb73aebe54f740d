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
//     read) live in a shared-memory RING of 4 blocks of C columns (column j at ring index
//     (j + C) mod 4C), so the columns a chunk shares with its predecessor (the skewed
//     overlap) are reused on chip -- the inter-tile reuse of Sec. 4.2.2;
//   * the block a chunk will need next is prefetched one chunk ahead with 16-B cp.async
//     (LDGSTS, every address 16-B aligned -- the aligned loads of Sec. 4.2.3), so no warp
//     waits on HBM latency; out-of-grid chunks are zero-filled and never used;
//   * a level is a pure map over its cells (each statement reads only the other fields and
//     its own old value), so one CTA barrier separates levels; two threads per column split
//     the rows;
//   * a column is final once no later chunk touches it (j < (k+1)C - a_hi): after each chunk
//     its C final columns of every row the hexagon modifies are written back with coalesced
//     stores -- the interleaved copy-out of Sec. 4.2.1.
#include <cstdint>

#include "../stencil_ops.cuh"
#include "launch.h"

namespace hexs {
namespace fdtd {

constexpr int C = 64;        // columns per chunk (= ring block)
constexpr int RC = 4 * C;    // ring columns
constexpr int NT = 2 * C;    // two threads per column

template <typename T>
size_t smem_bytes(int W) {
  return (size_t)3 * (W + 2) * RC * sizeof(T);
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

// fields: 0 = ex, 1 = ey, 2 = hz (the order of FdtdArgs::f); statement k: 0 ey, 1 ex, 2 hz
template <typename T>
__global__ void __launch_bounds__(NT) fdtd_kernel(const __grid_constant__ FdtdArgs g) {
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
  auto stage = [&](int64_t blk) {
    const int64_t j = (blk - 1) * C + sc * CH;
    const bool jok = j >= 0 && j < N1;
    const int cj = (int)((j + C) & (RC - 1));
    int f = 0, rb = tid / NCH;  // smem row index (b + 1) within field f
    for (int fr = tid / NCH; fr < 3 * R; fr += RSTEP) {
      while (rb >= R) rb -= R, ++f;
      const int64_t i = i0 + rb - 1;
      const bool ok = jok && i >= 0 && i < N0;
      const T* base = f == 0 ? F[0] : (f == 1 ? F[1] : F[2]);
      const T* src = ok ? base + i * N1 + j : base;
      cp_async16(ring + ((size_t)f * R + rb) * RC + cj, src, ok);
      rb += RSTEP;
    }
    cp_async_commit();
  };

  const int64_t k_last = (N1 - 1 + g.a_hi) / C;
  stage(0);
  stage(1);
  stage(2);
  const int col = tid & (C - 1), rpar = tid / C;
  T* const rex = ring + (size_t)(0 * R + 1) * RC;  // row b of a field at r.. + b * RC + ring column
  T* const rey = ring + (size_t)(1 * R + 1) * RC;
  T* const rhz = ring + (size_t)(2 * R + 1) * RC;
  for (int64_t k = 0; k <= k_last; ++k) {
    stage(k + 3);          // next chunk's new block (ring slot of block k-1, written back)
    cp_async_wait<1>();    // every block but the newest has landed
    __syncthreads();
    for (int a = g.a_lo; a <= g.a_hi; ++a) {
      const int st = (int)((g.tau0 + a) % 3);
      const int64_t j = k * C - a + col;
      const int cj = (int)((j + C) & (RC - 1));
      // statement domains (oracle/oracle.c): ey i >= 1; ex j >= 1; hz i < N0-1, j < N1-1
      const int64_t ilo = st == 0 ? 1 : 0, ihi = st == 2 ? N0 - 2 : N0 - 1;
      const bool jok = st == 1 ? (j >= 1 && j < N1) : (st == 2 ? (j >= 0 && j < N1 - 1) : (j >= 0 && j < N1));
      const int blo = (int)max64(g.lo[a], ilo - i0), bhi = (int)min64(g.hi[a], ihi - i0);
      if (jok) {
        int b = blo + rpar;
        if (st == 0) {  // ey[i][j] -= ce * (hz[i][j] - hz[i-1][j])
          T* pe = rey + b * RC + cj;
          const T* ph = rhz + b * RC + cj;
#pragma unroll 2
          for (; b <= bhi; b += 2, pe += 2 * RC, ph += 2 * RC) *pe = fdtd_ey<T>(*pe, ph[0], ph[-RC], cf);
        } else if (st == 1) {  // ex[i][j] -= ce * (hz[i][j] - hz[i][j-1])
          const int cjm = (int)((j - 1 + C) & (RC - 1));
          T* px = rex + b * RC + cj;
          const T* ph = rhz + b * RC + cj;
          const T* phm = rhz + b * RC + cjm;
#pragma unroll 2
          for (; b <= bhi; b += 2, px += 2 * RC, ph += 2 * RC, phm += 2 * RC) *px = fdtd_ex<T>(*px, *ph, *phm, cf);
        } else {  // hz[i][j] -= ch * (((ex[i][j+1] - ex[i][j]) + ey[i+1][j]) - ey[i][j])
          const int cjp = (int)((j + 1 + C) & (RC - 1));
          T* ph = rhz + b * RC + cj;
          const T* px = rex + b * RC + cj;
          const T* pxp = rex + b * RC + cjp;
          const T* pe = rey + b * RC + cj;
#pragma unroll 2
          for (; b <= bhi; b += 2, ph += 2 * RC, px += 2 * RC, pxp += 2 * RC, pe += 2 * RC)
            *ph = fdtd_hz<T>(*ph, *pxp, *px, pe[RC], pe[0], cf);
        }
      }
      __syncthreads();
    }
    // write back the columns no later chunk touches: [kC - a_hi, (k+1)C - a_hi), or all
    // remaining columns after the last chunk
    const int64_t wlo = max64(0, k * C - g.a_hi);
    const int64_t whi = (k == k_last) ? N1 - 1 : (k + 1) * C - g.a_hi - 1;
    for (int64_t j = k * C - g.a_hi + col; j <= whi; j += C) {
      if (j < wlo) continue;
      const int cj = (int)((j + C) & (RC - 1));
#pragma unroll
      for (int f = 0; f < 3; ++f) {
        const T* sp = (f == 0 ? rex : (f == 1 ? rey : rhz)) + cj;
        T* gp = F[f] + j;
        for (int b = mlo[f] + rpar; b <= mhi[f]; b += 2) gp[(i0 + b) * N1] = sp[b * RC];
      }
    }
    __syncthreads();  // the write-back reads ring slots the next stage() overwrites
  }
  cp_async_wait<0>();
}

template <typename T>
cudaError_t launch_t(const FdtdArgs& a, int grid, cudaStream_t s) {
  static size_t attr = 0;
  const size_t smem = smem_bytes<T>(a.W);
  if (smem > attr) {
    cudaError_t e = cudaFuncSetAttribute(fdtd_kernel<T>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    if (e != cudaSuccess) return e;
    attr = smem;
  }
  fdtd_kernel<T><<<grid, NT, smem, s>>>(a);
  return cudaGetLastError();
}

}  // namespace fdtd

size_t fdtd_smem_bytes(int dtype, int W) {
  return dtype == 1 ? fdtd::smem_bytes<double>(W) : fdtd::smem_bytes<float>(W);
}

cudaError_t launch_fdtd(int variant, const FdtdArgs& a, int grid, cudaStream_t s) {
  switch (variant) {
    case 0: return fdtd::launch_t<float>(a, grid, s);
    case 1: return fdtd::launch_t<double>(a, grid, s);
    default: return cudaErrorInvalidValue;
  }
}

}  // namespace hexs
