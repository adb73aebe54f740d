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
#include "../stencil_ops.cuh"
#include "launch.h"

namespace hexs {

namespace {

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

template <typename T, int KIND>
__global__ void __launch_bounds__(256) generic_kernel(const __grid_constant__ GenericArgs g) {
  const int64_t S0 = g.S0_lo + blockIdx.x;
  const int64_t i0 = S0 * g.W - g.row_off;  // spatial coordinate of local row b = 0
  const Coef<T> k{(T)g.k0, (T)g.k1};
  const int w1 = g.ncls >= 1 ? g.w[0] : 1, w2 = g.ncls >= 2 ? g.w[1] : 1;
  const int64_t n1 = g.ncls >= 1 ? g.Shi[0] - g.Slo[0] + 1 : 1;
  const int64_t n2 = g.ncls >= 2 ? g.Shi[1] - g.Slo[1] + 1 : 1;
  for (int64_t q1 = 0; q1 < n1; ++q1) {      // classical tiles, sequential (Sec. 4.1)
    for (int64_t q2 = 0; q2 < n2; ++q2) {
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

template <typename T, int KIND>
__global__ void __launch_bounds__(256) naive3d_kernel(const T* __restrict__ src, T* __restrict__ dst,
                                                      int64_t N0, int64_t N1, int64_t N2, Coef<T> k) {
  const int64_t x = 1 + blockIdx.x * (int64_t)blockDim.x + threadIdx.x;
  const int64_t y = 1 + blockIdx.y;
  const int64_t z_start = 1 + (int64_t)blockIdx.z * kNaiveStrip;
  if (x > N2 - 2) return;
  const int64_t z_end = z_start + kNaiveStrip < N0 - 1 ? z_start + kNaiveStrip : N0 - 1;
  const int64_t s0 = N1 * N2;
  for (int64_t z = z_start; z < z_end; ++z) {
    const int64_t p = z * s0 + y * N2 + x;
    dst[p] = point_from_memory<T, KIND>(src, p, s0, N2, k);
  }
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

template <typename T>
cudaError_t launch_generic_t(int kind, const GenericArgs& g, int grid, cudaStream_t s) {
  dim3 blk(256);
  switch (kind) {
#define HEXS_CASE(K)                                                  \
  case K:                                                             \
    generic_kernel<T, K><<<grid, blk, 0, s>>>(g);                     \
    break;
    HEXS_CASE(K_JACOBI2D5) HEXS_CASE(K_STAR2D5) HEXS_CASE(K_BOX2D9) HEXS_CASE(K_FDTD2D)
    HEXS_CASE(K_STAR3D7) HEXS_CASE(K_GRADIENT3D) HEXS_CASE(K_BOX3D27) HEXS_CASE(K_GRADIENT2D)
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
    dim3 grid((unsigned)((N2 - 2 + 255) / 256), (unsigned)(N1 - 2),
              (unsigned)((N0 - 2 + kNaiveStrip - 1) / kNaiveStrip));
    switch (kind) {
#define HEXS_CASE(K) \
  case K: naive3d_kernel<T, K><<<grid, 256, 0, s>>>(src, dst, N0, N1, N2, k); break;
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

cudaError_t launch_naive(int kind, int dtype, int dims, const NaiveArgs& a, cudaStream_t s) {
  return dtype == 1 ? launch_naive_t<double>(kind, dims, a, s) : launch_naive_t<float>(kind, dims, a, s);
}

}  // namespace hexs
