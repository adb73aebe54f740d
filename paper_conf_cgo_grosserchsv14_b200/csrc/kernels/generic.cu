// generic.cu -- (1) the generic hybrid-tiled phase kernel, every class and dimension;
//               (2) the naive one-step-per-launch comparator kernels (K11).
//
// (1) follows Sec. 4.1 literally: one thread block per hexagon S0 of
// the current (T, p); the classical tiles S1..Sn and the tile-local time t' are
// sequential loops inside the block; the points of one (S1..Sn, t') step are spread over
// the threads cyclically ("iteration i is mapped to thread i mod Ti"), with a barrier
// after each step.  It reads and writes global memory directly -- the paper's Table 4
// configuration (a), PAPER.md:989 -- and serves as the reference executor for classes
// without a specialised kernel and as the ablation baseline.
#include <cstdlib>

#include "../stencil_ops.cuh"
#include "devcache.h"
#include "launch.h"

namespace hexs {

namespace {

// K_LINEAR: the descriptor's access set in its order, products then left-to-right sums (the
// oracle's expression tree; no contraction: --fmad=false)
template <typename T>
__device__ __forceinline__ T linear_point(const T* __restrict__ A, int64_t p, const LinearTerms& L) {
  T acc = (T)L.coef[0] * A[p + L.delta[0]];
  for (int k = 1; k < L.n; ++k) acc = acc + (T)L.coef[k] * A[p + L.delta[k]];
  return acc;
}

template <typename T, int KIND>
__device__ __forceinline__ void generic_point(const GenericArgs& g, int64_t tau, const int64_t* c,
                                              const Coef<T>& k) {
  if constexpr (KIND == K_FDTD2D) {
    const int stmt = (int)(tau % 3);
    const int64_t i = c[0], j = c[1], N0 = g.N[0], N1 = g.N[1];
    if (i < 0 || i >= N0 || j < 0 || j >= N1) return;
    T* ex = static_cast<T*>(g.f[0]);
    T* ey = static_cast<T*>(g.f[1]);
    T* hz = static_cast<T*>(g.f[2]);
    const int64_t p = i * N1 + j;
    if (stmt == 0) {
      if (i >= 1) ey[p] = fdtd_ey<T>(ey[p], hz[p], hz[p - N1], k);
    } else if (stmt == 1) {
      if (j >= 1) ex[p] = fdtd_ex<T>(ex[p], hz[p], hz[p - 1], k);
    } else {
      if (i <= N0 - 2 && j <= N1 - 2) hz[p] = fdtd_hz<T>(hz[p], ex[p + 1], ex[p], ey[p + N1], ey[p], k);
    }
  } else if constexpr (KIND == K_LINEAR) {
    int64_t p = 0;
    const int R = g.lin.R;
    for (int q = 0; q < g.dims; ++q) {
      if (c[q] < R || c[q] > g.N[q] - 1 - R) return;  // Dirichlet cells are never written
      p += c[q] * g.st[q];
    }
    const T* src = static_cast<const T*>(g.f[tau & 1]);
    T* dst = static_cast<T*>(g.f[(tau + 1) & 1]);
    dst[p] = linear_point<T>(src, p, g.lin);
  } else {
    int64_t p = 0;
    for (int q = 0; q < g.dims; ++q) {
      if (c[q] < 1 || c[q] > g.N[q] - 2) return;  // Dirichlet cells are never written
      p += c[q] * g.st[q];
    }
    const T* src = static_cast<const T*>(g.f[tau & 1]);
    T* dst = static_cast<T*>(g.f[(tau + 1) & 1]);
    dst[p] = point_from_memory<T, KIND>(src, p, g.st[0], g.dims == 3 ? g.st[1] : 0, k);
  }
}

// All levels of one classical tile (q1, q2) of hexagon S0.
template <typename T, int KIND>
__device__ __forceinline__ void generic_tile(const GenericArgs& g, int64_t S0, int64_t q1, int64_t q2,
                                             const Coef<T>& k) {
  const int64_t i0 = S0 * g.W - g.row_off;  // spatial coordinate of local row b = 0
  const int w1 = g.ncls >= 1 ? g.w[0] : 1, w2 = g.ncls >= 2 ? g.w[1] : 1;
  for (int a = g.a_lo; a <= g.a_hi; ++a) {  // tile-local time t', sequential
    const int64_t tau = g.tau0 + a;
    const int rows = g.hi[a] - g.lo[a] + 1;
    const int64_t base1 = (g.Slo[0] + q1) * w1 - (int64_t)g.dcls[0] * a;  // eq. (14)
    const int64_t base2 = (g.Slo[1] + q2) * w2 - (int64_t)g.dcls[1] * a;
    const int64_t total = (int64_t)rows * w1 * w2;
    for (int64_t e = threadIdx.x; e < total; e += blockDim.x) {  // s -> threads, cyclic
      const int x2 = (int)(e % w2);
      const int64_t r = e / w2;
      const int x1 = (int)(r % w1);
      const int b = (int)(r / w1) + g.lo[a];
      int64_t c[3] = {0, 0, 0};
      c[g.hd] = i0 + b;
      if (g.ncls >= 1) c[g.cls[0]] = base1 + x1;
      if (g.ncls >= 2) c[g.cls[1]] = base2 + x2;
      generic_point<T, KIND>(g, tau, c, k);
    }
    __syncthreads();
  }
}

template <typename T, int KIND>
__global__ void __launch_bounds__(256) generic_kernel(const __grid_constant__ GenericArgs g) {
  const int64_t S0 = g.S0_lo + blockIdx.x;
  const Coef<T> k{(T)g.k0, (T)g.k1};
  const int64_t n1 = g.ncls >= 1 ? g.Shi[0] - g.Slo[0] + 1 : 1;
  const int64_t n2 = g.ncls >= 2 ? g.Shi[1] - g.Slo[1] + 1 : 1;
  for (int64_t q1 = 0; q1 < n1; ++q1)      // classical tiles, sequential (Sec. 4.1)
    for (int64_t q2 = 0; q2 < n2; ++q2) generic_tile<T, KIND>(g, S0, q1, q2, k);
}

__device__ __forceinline__ int ld_acquire(const int* p) {
  int v;
  asm volatile("ld.acquire.gpu.global.b32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void st_release(int* p, int v) {
  asm volatile("st.release.gpu.global.b32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}

// Wavefront execution: the classical tiles of a hexagon form a 2-D dependence grid
// ((S1, S2) needs (S1-1, S2) and (S1, S2-1) -- eq. (14)'s skew makes every dependence point
// to a lower tile index).  Tiles on one anti-diagonal are independent, so a hexagon's
// classical tiles run concurrently on many SMs instead of sequentially on one (the paper's
// mapping, Sec. 4.1, leaves S1..Sn sequential; with 148 SMs and ~26-51 hexagons per phase
// on 512^3 that would idle most of the GPU).  Persistent CTAs fetch items in (diagonal,
// S0, S1) order; every item waits only for items fetched earlier, so the grid (all CTAs
// resident) cannot deadlock.
template <typename T, int KIND>
__global__ void __launch_bounds__(256) generic_wf_kernel(const __grid_constant__ GenericArgs g) {
  __shared__ int64_t item_s[3];
  const Coef<T> k{(T)g.k0, (T)g.k1};
  const int64_t n1 = g.Shi[0] - g.Slo[0] + 1;
  const int64_t n2 = g.ncls >= 2 ? g.Shi[1] - g.Slo[1] + 1 : 1;
  const int64_t ns0 = g.S0_hi - g.S0_lo + 1;
  const int64_t n_items = ns0 * n1 * n2;
  while (true) {
    if (threadIdx.x == 0) {
      const int64_t it = (int64_t)atomicAdd(g.counter, 1ull);
      int64_t S0 = -1, q1 = 0, q2 = 0;
      if (it < n_items) {
        // decode: anti-diagonal d = q1 + q2 (outer), then S0, then q1
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
        const int64_t base = (S0 - g.S0_lo) * n1 * n2;
        if (q1 > 0)
          while (ld_acquire(g.flags + base + (q1 - 1) * n2 + q2) == 0) __nanosleep(64);
        if (q2 > 0)
          while (ld_acquire(g.flags + base + q1 * n2 + q2 - 1) == 0) __nanosleep(64);
        __threadfence();  // gpu-scope fence: drop stale L1 lines before reading neighbours
      }
      item_s[0] = S0;
      item_s[1] = q1;
      item_s[2] = q2;
    }
    __syncthreads();
    const int64_t S0 = item_s[0], q1 = item_s[1], q2 = item_s[2];
    if (S0 < 0) break;
    generic_tile<T, KIND>(g, S0, q1, q2, k);  // ends with __syncthreads
    if (threadIdx.x == 0) {
      __threadfence();
      st_release(g.flags + (S0 - g.S0_lo) * n1 * n2 + q1 * n2 + q2, 1);
    }
  }
}

// ------------------------------------------------------------------------------------
// Naive comparator: one launch per time step, no time tiling.  2D: a thread owns one
// column and a strip of rows (vertical neighbours from the previous iteration stay in
// L1); 3D: a thread owns one (y, x) column and a strip of z-planes.
// ------------------------------------------------------------------------------------
constexpr int kNaiveStrip = 16;

template <typename T, int KIND>
__global__ void __launch_bounds__(256) naive2d_kernel(const T* __restrict__ src, T* __restrict__ dst,
                                                      int64_t N0, int64_t N1, Coef<T> k) {
  const int64_t j = 1 + blockIdx.x * (int64_t)blockDim.x + threadIdx.x;
  const int64_t i_start = 1 + (int64_t)blockIdx.y * kNaiveStrip;
  if (j > N1 - 2) return;
  const int64_t i_end = i_start + kNaiveStrip < N0 - 1 ? i_start + kNaiveStrip : N0 - 1;
  for (int64_t i = i_start; i < i_end; ++i) {
    const int64_t p = i * N1 + j;
    dst[p] = point_from_memory<T, KIND>(src, p, N1, 0, k);
  }
}

// 3D naive step: block = 64 (x) x 4 (y) columns marching over a z-strip; the z-neighbours
// stay in a register queue, the in-plane neighbours come from L1 (shared by the block's
// lines).  One read of each plane from DRAM per step when L1/L2 absorb the reuse.
constexpr int kNaive3DStrip = 32;
template <typename T, int KIND>
__global__ void __launch_bounds__(256) naive3d_kernel(const T* __restrict__ src, T* __restrict__ dst,
                                                      int64_t N0, int64_t N1, int64_t N2, Coef<T> k) {
  const int64_t x = 1 + blockIdx.x * 64 + threadIdx.x;
  const int64_t y = 1 + (int64_t)blockIdx.y * 4 + threadIdx.y;
  const int64_t z_start = 1 + (int64_t)blockIdx.z * kNaive3DStrip;
  if (x > N2 - 2 || y > N1 - 2) return;
  const int64_t z_end = z_start + kNaive3DStrip < N0 - 1 ? z_start + kNaive3DStrip : N0 - 1;
  const int64_t s0 = N1 * N2;
  if constexpr (KIND == K_STAR3D7 || KIND == K_GRADIENT3D) {
    int64_t p = z_start * s0 + y * N2 + x;
    T u = src[p - s0], c = src[p];
    for (int64_t z = z_start; z < z_end; ++z, p += s0) {
      const T d = src[p + s0];
      const T n = src[p - N2], s = src[p + N2], w = src[p - 1], e = src[p + 1];
      if constexpr (KIND == K_STAR3D7) dst[p] = star3d7<T>(c, n, s, w, e, u, d, k);
      else dst[p] = gradient3d<T>(c, n, s, w, e, u, d, k);
      u = c;
      c = d;
    }
  } else {
    for (int64_t z = z_start; z < z_end; ++z) {
      const int64_t p = z * s0 + y * N2 + x;
      dst[p] = point_from_memory<T, KIND>(src, p, s0, N2, k);
    }
  }
}

// 3D naive step, 128-bit version (fp32 star classes, N2 % 4 == 0): a thread owns 4
// consecutive x of one (y) line and marches a z-strip with a register queue of centre quads;
// the y-neighbour quads come through L1 (the block's 8 lines share them), the x edges by
// shuffle from the neighbouring lanes (scalar loads at the warp's ends).  One pass over the
// source and one over the destination per step when L1/L2 absorb the reuse: the 8 B/update
// bound of a non-time-tiled kernel.
template <int KIND, int kNaiveV4Rows, bool PF, int kNaiveV4Strip>
__global__ void __launch_bounds__(32 * kNaiveV4Rows) naive3d_v4_kernel(const float* __restrict__ src, float* __restrict__ dst,
                                                         int64_t N0, int64_t N1, int64_t N2, Coef<float> k) {
  const int lane = threadIdx.x;                                       // 32 lanes along x
  const int64_t x = ((int64_t)blockIdx.x * 32 + lane) * 4;            // first x of the quad
  const int64_t y = 1 + (int64_t)blockIdx.y * kNaiveV4Rows + threadIdx.y;
  const int64_t z_start = 1 + (int64_t)blockIdx.z * kNaiveV4Strip;
  const bool xin = x < N2, yin = y <= N1 - 2;                         // uniform per warp except the tail
  const int64_t z_end = z_start + kNaiveV4Strip < N0 - 1 ? z_start + kNaiveV4Strip : N0 - 1;
  const int64_t s0 = N1 * N2;  // (no early exit: every lane takes part in the shuffles)
  const float4 zero = make_float4(0.f, 0.f, 0.f, 0.f);
  auto ld4 = [&](int64_t p) { return (xin && yin) ? __ldg(reinterpret_cast<const float4*>(src + p)) : zero; };
  int64_t p = z_start * s0 + y * N2 + x;
  float4 u = ld4(p - s0), c = ld4(p), d = PF ? ld4(p + s0) : zero;
  for (int64_t z = z_start; z < z_end; ++z, p += s0) {
    // next plane's centre quad one iteration ahead (more loads in flight per warp)
    const float4 dn = PF ? (z + 1 < z_end ? ld4(p + 2 * s0) : zero) : zero;
    if (!PF) d = ld4(p + s0);
    const float4 n = ld4(p - N2), so = ld4(p + N2);
    float we = __shfl_up_sync(0xffffffffu, c.w, 1), ee = __shfl_down_sync(0xffffffffu, c.x, 1);
    if (lane == 0) we = (xin && yin && x > 0) ? src[p - 1] : 0.f;
    if (lane == 31) ee = (xin && yin && x + 4 < N2) ? src[p + 4] : 0.f;
    float4 o;
    if constexpr (KIND == K_STAR3D7) {
      o.x = star3d7<float>(c.x, n.x, so.x, we, c.y, u.x, d.x, k);
      o.y = star3d7<float>(c.y, n.y, so.y, c.x, c.z, u.y, d.y, k);
      o.z = star3d7<float>(c.z, n.z, so.z, c.y, c.w, u.z, d.z, k);
      o.w = star3d7<float>(c.w, n.w, so.w, c.z, ee, u.w, d.w, k);
    } else {
      o.x = gradient3d<float>(c.x, n.x, so.x, we, c.y, u.x, d.x, k);
      o.y = gradient3d<float>(c.y, n.y, so.y, c.x, c.z, u.y, d.y, k);
      o.z = gradient3d<float>(c.z, n.z, so.z, c.y, c.w, u.z, d.z, k);
      o.w = gradient3d<float>(c.w, n.w, so.w, c.z, ee, u.w, d.w, k);
    }
    if (x == 0) o.x = c.x;            // Dirichlet columns are never written: keep the value
    if (x + 3 == N2 - 1) o.w = c.w;
    if (xin && yin) *reinterpret_cast<float4*>(dst + p) = o;
    u = c;
    c = d;
    d = dn;
  }
}

// Naive step of a general linear stencil: one thread per interior point.
template <typename T>
__global__ void __launch_bounds__(256) naive_linear_kernel(const T* __restrict__ src, T* __restrict__ dst,
                                                           int64_t N0, int64_t N1, int64_t N2,
                                                           const __grid_constant__ LinearTerms L) {
  const int R = L.R;
  const int64_t x = R + blockIdx.x * (int64_t)blockDim.x + threadIdx.x;
  const int64_t y = R + (int64_t)blockIdx.y;
  const int64_t z = N2 > 1 ? R + (int64_t)blockIdx.z : 0;
  const int64_t X = N2 > 1 ? N2 : N1, Y = N2 > 1 ? N1 : N0;  // 2D: (y, x) = (i, j)
  if (x > X - 1 - R || y > Y - 1 - R) return;
  const int64_t p = N2 > 1 ? (z * N1 + y) * N2 + x : y * N1 + x;
  dst[p] = linear_point<T>(src, p, L);
}

template <typename T>
__global__ void __launch_bounds__(256) naive_fdtd_kernel(T* __restrict__ ex, T* __restrict__ ey,
                                                         T* __restrict__ hz, int64_t N0, int64_t N1,
                                                         int stmt, Coef<T> k) {
  const int64_t j = blockIdx.x * (int64_t)blockDim.x + threadIdx.x;
  const int64_t i_start = (int64_t)blockIdx.y * kNaiveStrip;
  if (j >= N1) return;
  const int64_t i_end = i_start + kNaiveStrip < N0 ? i_start + kNaiveStrip : N0;
  for (int64_t i = i_start; i < i_end; ++i) {
    const int64_t p = i * N1 + j;
    if (stmt == 0) {
      if (i >= 1) ey[p] = fdtd_ey<T>(ey[p], hz[p], hz[p - N1], k);
    } else if (stmt == 1) {
      if (j >= 1) ex[p] = fdtd_ex<T>(ex[p], hz[p], hz[p - 1], k);
    } else {
      if (i <= N0 - 2 && j <= N1 - 2) hz[p] = fdtd_hz<T>(hz[p], ex[p + 1], ex[p], ey[p + N1], ey[p], k);
    }
  }
}

template <typename T, int K>
int wf_grid_t() {
  static DeviceMemo<int> memo;  // persistent grid (all CTAs co-resident), per device
  int grid = 0;
  if (memo.get(&grid, [](int dev, int* g) {
        int sms = 0, per_sm = 0;
        cudaError_t e = cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
        if (e == cudaSuccess)
          e = cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, generic_wf_kernel<T, K>, 256, 0);
        *g = sms * (per_sm > 0 ? per_sm : 1);
        return e;
      }) != cudaSuccess)
    return 1;
  return grid;
}

template <typename T>
cudaError_t launch_generic_t(int kind, const GenericArgs& g, int grid, cudaStream_t s) {
  dim3 blk(256);
  switch (kind) {
#define HEXS_CASE(K)                                                  \
  case K:                                                             \
    if (g.wf) generic_wf_kernel<T, K><<<wf_grid_t<T, K>(), blk, 0, s>>>(g); \
    else generic_kernel<T, K><<<grid, blk, 0, s>>>(g);                \
    break;
    HEXS_CASE(K_JACOBI2D5) HEXS_CASE(K_STAR2D5) HEXS_CASE(K_BOX2D9) HEXS_CASE(K_FDTD2D)
    HEXS_CASE(K_STAR3D7) HEXS_CASE(K_GRADIENT3D) HEXS_CASE(K_BOX3D27) HEXS_CASE(K_GRADIENT2D)
    HEXS_CASE(K_LINEAR)
#undef HEXS_CASE
    default:
      return cudaErrorInvalidValue;
  }
  return cudaGetLastError();
}

template <typename T>
cudaError_t launch_naive_t(int kind, int dims, const NaiveArgs& a, cudaStream_t s) {
  const Coef<T> k{(T)a.k0, (T)a.k1};
  const int64_t N0 = a.N[0], N1 = a.N[1], N2 = a.N[2];
  if (kind == K_FDTD2D) {
    dim3 grid((unsigned)((N1 + 255) / 256), (unsigned)((N0 + kNaiveStrip - 1) / kNaiveStrip));
    naive_fdtd_kernel<T><<<grid, 256, 0, s>>>(static_cast<T*>(a.f[0]), static_cast<T*>(a.f[1]),
                                              static_cast<T*>(a.f[2]), N0, N1, a.stmt, k);
    return cudaGetLastError();
  }
  const T* src = static_cast<const T*>(a.src);
  T* dst = static_cast<T*>(a.dst);
  if (kind == K_LINEAR) {
    const int R = a.lin.R;
    const int64_t X = dims == 3 ? N2 : N1, Y = dims == 3 ? N1 : N0;
    dim3 grid((unsigned)((X - 2 * R + 255) / 256), (unsigned)(Y - 2 * R), dims == 3 ? (unsigned)(N0 - 2 * R) : 1u);
    naive_linear_kernel<T><<<grid, 256, 0, s>>>(src, dst, N0, N1, dims == 3 ? N2 : 1, a.lin);
    return cudaGetLastError();
  }
  if (dims == 2) {
    dim3 grid((unsigned)((N1 - 2 + 255) / 256), (unsigned)((N0 - 2 + kNaiveStrip - 1) / kNaiveStrip));
    switch (kind) {
#define HEXS_CASE(K) \
  case K: naive2d_kernel<T, K><<<grid, 256, 0, s>>>(src, dst, N0, N1, k); break;
      HEXS_CASE(K_JACOBI2D5) HEXS_CASE(K_STAR2D5) HEXS_CASE(K_BOX2D9) HEXS_CASE(K_GRADIENT2D)
#undef HEXS_CASE
      default: return cudaErrorInvalidValue;
    }
  } else {
    if constexpr (sizeof(T) == 4) {
      if ((kind == K_STAR3D7 || kind == K_GRADIENT3D) && N2 % 4 == 0 && N2 >= 4) {
        // 4 lines x 128 columns per block, z-strips of 32 planes: measured best on B200 among
        // (4 | 8 | 16 lines) x (16 | 32 | 64 | 128 planes) x (prefetch on / off): 704 GUp/s on
        // 512^3 (5.6 TB/s at the 8 B/update bound = 0.86 of the measured copy bandwidth)
        const float* fs = reinterpret_cast<const float*>(src);
        float* fd = reinterpret_cast<float*>(dst);
        const Coef<float> kf{(float)a.k0, (float)a.k1};
        constexpr int R = 4, S = 32;
        auto pick = [&](auto kc) {
          constexpr int K = decltype(kc)::value;
          dim3 g4((unsigned)((N2 / 4 + 31) / 32), (unsigned)((N1 - 2 + R - 1) / R), (unsigned)((N0 - 2 + S - 1) / S));
          naive3d_v4_kernel<K, R, false, S><<<g4, dim3(32, R), 0, s>>>(fs, fd, N0, N1, N2, kf);
        };
        if (kind == K_STAR3D7) pick(std::integral_constant<int, K_STAR3D7>{});
        else pick(std::integral_constant<int, K_GRADIENT3D>{});
        return cudaGetLastError();
      }
    }
    dim3 grid((unsigned)((N2 - 2 + 63) / 64), (unsigned)((N1 - 2 + 3) / 4),
              (unsigned)((N0 - 2 + kNaive3DStrip - 1) / kNaive3DStrip));
    dim3 blk(64, 4);
    switch (kind) {
#define HEXS_CASE(K) \
  case K: naive3d_kernel<T, K><<<grid, blk, 0, s>>>(src, dst, N0, N1, N2, k); break;
      HEXS_CASE(K_STAR3D7) HEXS_CASE(K_GRADIENT3D) HEXS_CASE(K_BOX3D27)
#undef HEXS_CASE
      default: return cudaErrorInvalidValue;
    }
  }
  return cudaGetLastError();
}

}  // namespace

cudaError_t launch_generic(int kind, int dtype, const GenericArgs& g, int grid, cudaStream_t s) {
  return dtype == 1 ? launch_generic_t<double>(kind, g, grid, s) : launch_generic_t<float>(kind, g, grid, s);
}

int generic_wf_grid(int kind, int dtype) {
  (void)kind;
  return dtype == 1 ? wf_grid_t<double, K_STAR3D7>() : wf_grid_t<float, K_STAR3D7>();
}

cudaError_t launch_naive(int kind, int dtype, int dims, const NaiveArgs& a, cudaStream_t s) {
  return dtype == 1 ? launch_naive_t<double>(kind, dims, a, s) : launch_naive_t<float>(kind, dims, a, s);
}

}  // namespace hexs
