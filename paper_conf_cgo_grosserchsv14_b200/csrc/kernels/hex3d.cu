// hex3d.cu -- the specialised sm_100a phase kernel for 3D single-field stencils of radius 1
// (star3d7, gradient3d, box3d27) under the hybrid schedule: hexagonal over (t, z), classical
// parallelogram tiles over y and x (eq. (14)).
//
// Mapping:
//   * work item = one classical tile (S1, S2) of one hexagon S0 of the launch's (T, p): a
//     NY x NX (y, x) parallelogram over all 2h+2 levels and all hexagon rows z;
//   * items run as a dependence WAVEFRONT: (S1, S2) needs (S1-1, S2) and (S1, S2-1) of the
//     same hexagon (the skew of eq. (14) makes every dependence point to a lower tile index);
//     persistent CTAs fetch items in anti-diagonal order from an atomic counter and wait on
//     the predecessors' release flags, so the ~26-51 hexagons per phase of a 512^3 grid keep
//     all 148 SMs busy (the paper's mapping runs S1..Sn sequentially inside one block,
//     PAPER.md:683-689);
//   * the tile's current level lives in shared memory (two level buffers, planes z x lines y
//     x columns x); a thread owns 2 lines x 4 columns of one half of the rows and sweeps z
//     with a 3-plane register window, so z-neighbours come from registers and y/x
//     neighbours from vectorised LDS.128/LDS.64;
//   * per level only the In planes (the hexagon's slanted-edge inputs) and
//     the two carry lines/columns produced by the predecessor tiles are fetched from L2/HBM,
//     asynchronously with cp.async one level ahead (into buffer areas the current level does
//     not write); only the Out planes, the tile's last two lines/columns (the successors'
//     carries) and the final level are stored -- interleaved copy-out.
#include <cstdint>

#include "../stencil_ops.cuh"
#include "launch.h"

namespace hexs {
namespace fast3d {

constexpr int NY = 16, NX = 32;   // classical tile (y lines, x columns)
constexpr int NT = 128;           // 2 row groups x 8 line pairs x 8 column quads
constexpr int LY = NY + 2;        // buffer lines (2 carry lines)
constexpr int OFF = 4;            // buffer column of x-coordinate lx = 0 (16-B alignment shift)
constexpr int SX = NX + 8;        // buffer row pitch (elements): lx in [0, NX+3] at OFF..OFF+NX+3

using Args = Fast3DArgs;
static_assert(NY == kFast3DNY && NX == kFast3DNX, "tile geometry");

__device__ __forceinline__ int ld_acquire(const int* p) {
  int v;
  asm volatile("ld.acquire.gpu.global.b32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void st_release(int* p, int v) {
  asm volatile("st.release.gpu.global.b32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}
template <typename T>
__device__ __forceinline__ void cp_async(T* dst_smem, const T* src) {
  const uint32_t d = static_cast<uint32_t>(__cvta_generic_to_shared(dst_smem));
  if constexpr (sizeof(T) == 4)
    asm volatile("cp.async.ca.shared.global [%0], [%1], 4;" ::"r"(d), "l"(src) : "memory");
  else
    asm volatile("cp.async.ca.shared.global [%0], [%1], 8;" ::"r"(d), "l"(src) : "memory");
}
__device__ __forceinline__ void cp_async_commit_wait() {
  asm volatile("cp.async.commit_group;\ncp.async.wait_group 0;" ::: "memory");
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

template <typename T>
struct Tile {
  const Args& g;
  T* sm;              // [2][Q][LY][SX]
  int64_t i0, Y0, X0; // z of local row b = 0; tile origin (window at level a: Y0-a.., X0-a..)
  int64_t plane;      // N1*N2

  __device__ __forceinline__ T* bufp(int which, int q, int ly, int lx) const {
    return sm + (((size_t)which * g.Q + q) * LY + ly) * SX + OFF + lx;
  }
  // Global position of buffer cell (q, ly, lx) holding level-ell values (ell = level whose
  // outputs the buffer holds; inputs of level a are level a-1).
  __device__ __forceinline__ void pos(int ell, int q, int ly, int lx, int64_t& z, int64_t& y, int64_t& x) const {
    z = i0 + (q - 1);
    y = Y0 - ell - 2 + ly;
    x = X0 - ell - 2 + lx;
  }

  // cp.async the cells of plane q, lines [ly0, ly1), cols [lx0, lx1) of the input buffer of
  // level a (level a-1 values, global buffer parity (tau0 + a) & 1), clamped into the grid.
  __device__ __forceinline__ void fetch(int a, int which, int q, int ly0, int ly1, int lx0, int lx1) const {
    const T* src = static_cast<const T*>(g.buf[(g.tau0 + a) & 1]);
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    int64_t z, y, x;
    pos(a - 1, q, 0, 0, z, y, x);
    z = z < 0 ? 0 : (z >= g.N0 ? g.N0 - 1 : z);
    const T* zp = src + z * plane;
    for (int ly = ly0 + warp; ly < ly1; ly += NT / 32) {
      int64_t yy = y + ly;
      yy = yy < 0 ? 0 : (yy >= g.N1 ? g.N1 - 1 : yy);
      const T* yp = zp + yy * g.N2;
      for (int lx = lx0 + lane; lx < lx1; lx += 32) {
        int64_t xx = x + lx;
        xx = xx < 0 ? 0 : (xx >= g.N2 ? g.N2 - 1 : xx);
        cp_async(bufp(which, q, ly, lx), yp + xx);
      }
    }
  }

  __device__ __forceinline__ int lo(int a) const { return g.lo[a]; }
  __device__ __forceinline__ int hi(int a) const { return g.hi[a]; }

  // The In planes of level a (planes not computed at level a-1; every input plane if
  // `all`) in full, into the input buffer of level a.  No dependence inside the launch:
  // they were produced by earlier launches.
  __device__ __forceinline__ void fetch_in_planes(int a, bool all) const {
    const int which = a & 1;
    for (int q = lo(a); q <= hi(a) + 2; ++q) {
      const int b = q - 1;
      if (all || b < lo(a - 1) || b > hi(a - 1)) fetch(a, which, q, 0, LY, 0, NX + 2);
    }
  }
  // The carries of level a: for every plane computed at level a-1, the two lines above the
  // window (from tiles (S1-1, S2) and (S1-1, S2-1)) and the two columns left of it (from
  // (S1, S2-1)), produced by those tiles at level a-1 in this launch.
  __device__ __forceinline__ void fetch_carries(int a) const {
    const int which = a & 1;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const T* src = static_cast<const T*>(g.buf[(g.tau0 + a) & 1]);
    for (int q = lo(a - 1) + 1; q <= hi(a - 1) + 1; ++q) {
      fetch(a, which, q, 0, 2, 0, NX + 2);
      // two columns x NY lines: one pass of one warp (lane = 2 * line + column)
      if (warp == (q & 3)) {
        const int ly = 2 + (lane >> 1), lx = lane & 1;
        int64_t z, y, x;
        pos(a - 1, q, ly, lx, z, y, x);
        z = z < 0 ? 0 : (z >= g.N0 ? g.N0 - 1 : z);
        y = y < 0 ? 0 : (y >= g.N1 ? g.N1 - 1 : y);
        x = x < 0 ? 0 : (x >= g.N2 ? g.N2 - 1 : x);
        cp_async(bufp(which, q, ly, lx), src + z * plane + y * g.N2 + x);
      }
    }
  }
};

template <typename T, int KIND>
__global__ void __launch_bounds__(NT, 3) fast3d_kernel(const __grid_constant__ Args g) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  __shared__ int64_t item_s[3];
  T* sm = reinterpret_cast<T*>(smem_raw);
  const Coef<T> cf{(T)g.k0, (T)g.k1};
  const int tid = threadIdx.x;
  const int zg = tid >> 6, lp = (tid >> 3) & 7, xq = tid & 7;  // row group, line pair, col quad
  const int64_t ns0 = g.S0_hi - g.S0_lo + 1;
  const int64_t n1 = g.n1, n2 = g.n2, n_items = ns0 * n1 * n2;
  const int64_t plane = g.N1 * g.N2;

  while (true) {
    if (tid == 0) {
      const int64_t it = (int64_t)atomicAdd(g.counter, 1ull);
      int64_t S0 = -1, q1 = 0, q2 = 0;
      if (it < n_items) {
        int64_t off = 0;
        for (int64_t d = 0; d < n1 + n2 - 1; ++d) {
          const int64_t lo1 = d - (n2 - 1) > 0 ? d - (n2 - 1) : 0;
          const int64_t hi1 = d < n1 - 1 ? d : n1 - 1;
          const int64_t pairs = hi1 - lo1 + 1;
          if (it < off + pairs * ns0) {
            const int64_t r = it - off;
            S0 = g.S0_lo + r / pairs;
            q1 = lo1 + r % pairs;
            q2 = d - q1;
            break;
          }
          off += pairs * ns0;
        }
      }
      item_s[0] = S0;
      item_s[1] = q1;
      item_s[2] = q2;
    }
    __syncthreads();
    const int64_t S0 = item_s[0];
    if (S0 < 0) break;
    const int64_t q1 = item_s[1], q2 = item_s[2];
    const int64_t fbase = (S0 - g.S0_lo) * n1 * n2;
    int* my_flag = g.flags + fbase + q1 * n2 + q2;
    Tile<T> t{g, sm, S0 * g.W - g.row_off, (g.S1_lo + q1) * NY, (g.S2_lo + q2) * NX, plane};

    // prologue: every input plane of the first level (all produced by earlier launches)
    t.fetch_in_planes(g.a_lo, true);
    cp_async_commit_wait();
    __syncthreads();

    for (int a = g.a_lo; a <= g.a_hi; ++a) {
      const int ib = a & 1, ob = (a + 1) & 1;
      if (a > g.a_lo) {
        // (0) level-granular dependences: the predecessors (S1-1, S2), (S1, S2-1),
        //     (S1-1, S2-1) must have published level a-1 (progress >= a - a_lo)
        if (tid == 0) {
          const int need = a - g.a_lo;
          if (q1 > 0)
            while (ld_acquire(g.flags + fbase + (q1 - 1) * n2 + q2) < need) __nanosleep(20);
          if (q2 > 0)
            while (ld_acquire(g.flags + fbase + q1 * n2 + q2 - 1) < need) __nanosleep(20);
          if (q1 > 0 && q2 > 0)
            while (ld_acquire(g.flags + fbase + (q1 - 1) * n2 + q2 - 1) < need) __nanosleep(20);
          __threadfence();
        }
        __syncthreads();
        t.fetch_carries(a);
        cp_async_commit_wait();  // also completes the In planes prefetched during level a-1
        __syncthreads();
      }
      // (1) one level ahead: the In planes of level a+1 into areas level a does not write
      if (a < g.a_hi) t.fetch_in_planes(a + 1, false);
      // (2) compute level a: rows [lo, hi] split in two groups, 3-plane register window
      const int rlo = t.lo(a), rhi = t.hi(a);
      const int mid = (rlo + rhi) >> 1;
      const int r0 = zg == 0 ? rlo : mid + 1, r1 = zg == 0 ? mid : rhi;
      // this thread's output cells: lines 2+2lp+{0,1}, cols 2+4xq+{0..3}
      const int ly_o = 2 + 2 * lp, lx_o = 2 + 4 * xq;
      int64_t zc, yc, xc;
      t.pos(a, 0, ly_o, lx_o, zc, yc, xc);
      bool lineok[2], colok[4];
#pragma unroll
      for (int i = 0; i < 2; ++i) lineok[i] = (yc + i >= 1) && (yc + i <= g.N1 - 2);
#pragma unroll
      for (int j = 0; j < 4; ++j) colok[j] = (xc + j >= 1) && (xc + j <= g.N2 - 2);
      T win[3][4][6];  // [plane r-1, r, r+1][input lines 2lp..2lp+3][input cols 4xq..4xq+5]
      // 8 consecutive elements (cols 4xq..4xq+7, 16-B aligned) per input line via
      // LDS.128; the first 6 are the thread's input columns
      auto load_plane = [&](int q, T (&dst)[4][6]) {
#pragma unroll
        for (int l = 0; l < 4; ++l) {
          const T* p = t.bufp(ib, q, 2 * lp + l, 4 * xq);
          T v[8];
          if constexpr (sizeof(T) == 4) {
            const float4 u0 = reinterpret_cast<const float4*>(p)[0];
            const float4 u1 = reinterpret_cast<const float4*>(p)[1];
            v[0] = u0.x; v[1] = u0.y; v[2] = u0.z; v[3] = u0.w;
            v[4] = u1.x; v[5] = u1.y; v[6] = u1.z; v[7] = u1.w;
          } else {
#pragma unroll
            for (int i = 0; i < 4; ++i) {
              const double2 u = reinterpret_cast<const double2*>(p)[i];
              v[2 * i] = u.x; v[2 * i + 1] = u.y;
            }
          }
#pragma unroll
          for (int c = 0; c < 6; ++c) dst[l][c] = v[c];
        }
      };
      if (r0 <= r1) {
        load_plane(r0, win[0]);      // plane q = r0 (row b = r0 - 1)
        load_plane(r0 + 1, win[1]);  // plane of row r0
        for (int r = r0; r <= r1; ++r) {
          load_plane(r + 2, win[2]);  // plane of row r + 1
          const int64_t z = t.i0 + r;
          const bool zok = (z >= 1) && (z <= g.N0 - 2);
          T out[2][4];
#pragma unroll
          for (int i = 0; i < 2; ++i) {
#pragma unroll
            for (int j = 0; j < 4; ++j) {
              T x[3][3][3];
#pragma unroll
              for (int dz = 0; dz < 3; ++dz)
#pragma unroll
                for (int dy = 0; dy < 3; ++dy)
#pragma unroll
                  for (int dx = 0; dx < 3; ++dx) x[dz][dy][dx] = win[dz][i + dy][j + dx];
              const T v = apply<T, KIND>(x, cf);
              out[i][j] = (zok && lineok[i] && colok[j]) ? v : x[1][1][1];
            }
          }
#pragma unroll
          for (int i = 0; i < 2; ++i) {
            T* p = t.bufp(ob, r + 1, ly_o + i, lx_o);  // 8-B aligned (fp32) / 16-B (fp64)
            if constexpr (sizeof(T) == 4) {
              reinterpret_cast<float2*>(p)[0] = make_float2(out[i][0], out[i][1]);
              reinterpret_cast<float2*>(p)[1] = make_float2(out[i][2], out[i][3]);
            } else {
              reinterpret_cast<double2*>(p)[0] = make_double2(out[i][0], out[i][1]);
              reinterpret_cast<double2*>(p)[1] = make_double2(out[i][2], out[i][3]);
            }
          }
#pragma unroll
          for (int l = 0; l < 4; ++l)
#pragma unroll
            for (int c = 0; c < 6; ++c) {
              win[0][l][c] = win[1][l][c];
              win[1][l][c] = win[2][l][c];
            }
        }
      }
      __syncthreads();
      // (3) copy out: Out planes / final level in full, else the successors' carries
      T* dst = static_cast<T*>(g.buf[(g.tau0 + a + 1) & 1]);
      const bool fin = (a == g.a_final);
      for (int r = rlo; r <= rhi; ++r) {
        bool full = fin;
        if (a == g.H) full = full || r == rlo || r == rhi;
        else if (a > g.H && a < g.L - 1) full = full || r <= rlo + 1 || r >= rhi - 1;
        else if (a == g.L - 1) full = true;
        const int64_t z = t.i0 + r;
        if (z < 1 || z > g.N0 - 2) continue;
        // full window (NY x NX) or only lines NY, NY+1 and columns NX, NX+1 of the window
        const int n = full ? NY * NX : 2 * NX + 2 * (NY - 2);
        for (int e = tid; e < n; e += NT) {
          int ly, lx;
          if (full) {
            ly = 2 + e / NX;
            lx = 2 + e % NX;
          } else if (e < 2 * NX) {
            ly = NY + (e / NX);
            lx = 2 + e % NX;
          } else {
            const int f = e - 2 * NX;
            ly = 2 + f / 2;
            lx = NX + (f & 1);
          }
          int64_t zz, y, x;
          t.pos(a, r + 1, ly, lx, zz, y, x);
          if (y >= 1 && y <= g.N1 - 2 && x >= 1 && x <= g.N2 - 2)
            dst[zz * plane + y * g.N2 + x] = *t.bufp(ob, r + 1, ly, lx);
        }
      }
      __syncthreads();  // every thread's stores of level a precede the release
      if (tid == 0) {
        __threadfence();
        st_release(my_flag, a - g.a_lo + 1);
      }
    }
    cp_async_commit_wait();
  }
}

template <typename T, int KIND>
cudaError_t launch_t(const Args& a, cudaStream_t s) {
  static int grid = 0;
  static size_t attr_bytes = 0;
  const size_t smem = (size_t)2 * a.Q * LY * SX * sizeof(T);
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
  fast3d_kernel<T, KIND><<<grid, NT, smem, s>>>(a);
  return cudaGetLastError();
}

}  // namespace fast3d

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
