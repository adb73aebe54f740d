// stencil_ops.cuh -- per-point arithmetic of every stencil class (device side).
//
// One definition per class, written on VALUES (not memory) so the register-wavefront
// kernels and the generic global-memory kernel evaluate the identical expression tree.
// The association order is fixed (left to right as written) and the library is built with
// --fmad=false, -prec-div=true, -prec-sqrt=true, no FTZ, so results are bit-identical to
// any IEEE implementation of the same expression.
//
// Expressions (Table 3 of the paper; Fig. 1 / Fig. 2 for Jacobi,
// PAPER.md:142-158; readings R7-R9 of DESIGN.md for the classes the paper does not spell
// out).  Neighbour names: 2D (i,j): n=i-1 s=i+1 w=j-1 e=j+1.  3D (z,y,x): u=z-1 d=z+1
// n=y-1 s=y+1 w=x-1 e=x+1.
#pragma once
#include <cstdint>

namespace hexs {

enum Kind : int {
  K_JACOBI2D5 = 0, K_STAR2D5 = 1, K_BOX2D9 = 2, K_FDTD2D = 3,
  K_STAR3D7 = 4, K_GRADIENT3D = 5, K_BOX3D27 = 6, K_GRADIENT2D = 7, K_LINEAR = 8
};

template <typename T> struct Coef { T k0, k1; };

// Blackwell packed FP32 (sm_100a FADD2 / FMUL2): a pair of fp32 values in one 64-bit
// register pair; each operator is two IEEE round-to-nearest fp32 operations in ONE
// instruction, element-wise bit-identical to the scalar ones (no FTZ, no contraction).
// The per-class expressions below, instantiated on F2, evaluate two points with the same
// association order -- half the FP32 instructions of the scalar sweep.
struct F2 { uint64_t v; };
__device__ __forceinline__ F2 f2_pack(float a, float b) {
  F2 r;
  asm("mov.b64 %0, {%1, %2};" : "=l"(r.v) : "f"(a), "f"(b));
  return r;
}
__device__ __forceinline__ void f2_unpack(F2 p, float& a, float& b) {
  asm("mov.b64 {%0, %1}, %2;" : "=f"(a), "=f"(b) : "l"(p.v));
}
__device__ __forceinline__ F2 operator+(F2 a, F2 b) {
  F2 d;
  asm("add.rn.f32x2 %0, %1, %2;" : "=l"(d.v) : "l"(a.v), "l"(b.v));
  return d;
}
// ptxas contracts mul.rn.f32x2 feeding add.rn.f32x2 into FFMA2 even under --fmad=false
// (probed: tools/probe_f32x2/contract.cu), which would round k0*c and the sum once instead
// of twice.  So the product is an FFMA2 whose addend is -0.0 read from constant memory:
// a*b + (-0) == a*b bit for bit (RN, no FTZ; +0 + -0 = +0), and an FMA result cannot be
// contracted again.
static __constant__ uint64_t kF2NegZero = 0x8000000080000000ull;
__device__ __forceinline__ F2 operator*(F2 a, F2 b) {
  F2 d;
  asm("fma.rn.f32x2 %0, %1, %2, %3;" : "=l"(d.v) : "l"(a.v), "l"(b.v), "l"(kF2NegZero));
  return d;
}

template <typename T> __device__ __forceinline__ T dev_sqrt(T x);
template <> __device__ __forceinline__ float dev_sqrt<float>(float x) { return __fsqrt_rn(x); }
template <> __device__ __forceinline__ double dev_sqrt<double>(double x) { return __dsqrt_rn(x); }
template <typename T> __device__ __forceinline__ T dev_rcp_div(T x);  // 1/x, IEEE
template <> __device__ __forceinline__ float dev_rcp_div<float>(float x) { return __fdiv_rn(1.0f, x); }
template <> __device__ __forceinline__ double dev_rcp_div<double>(double x) { return __ddiv_rn(1.0, x); }

// Fig. 1: 0.2f * (A[i][j] + A[i+1][j] + A[i-1][j] + A[i][j+1] + A[i][j-1]); Fig. 2 issues
// four add.f32 then one mul.f32 by 0f3E4CCCCD.
template <typename T>
__device__ __forceinline__ T jacobi2d5(T c, T n, T s, T w, T e, const Coef<T>& k) {
  return k.k0 * ((((c + s) + n) + e) + w);
}
// laplacian / heat 5-point: 5 loads, 6 FLOPs.
template <typename T>
__device__ __forceinline__ T star2d5(T c, T n, T s, T w, T e, const Coef<T>& k) {
  return k.k0 * c + k.k1 * (((n + s) + w) + e);
}
// gradient 2D: 5 loads, 15 FLOPs.
template <typename T>
__device__ __forceinline__ T gradient2d(T c, T n, T s, T w, T e, const Coef<T>& k) {
  T dn = c - n, ds = c - s, dw = c - w, de = c - e;
  T acc = dn * dn;
  acc = acc + ds * ds;
  acc = acc + dw * dw;
  acc = acc + de * de;
  return c + dev_rcp_div<T>(dev_sqrt<T>(k.k0 + acc));
}
// heat 2D 9-point: row-major accumulation of the 3x3 box then one scale (9 loads, 9 FLOPs).
// r{di}{dj} = A[i+di-1][j+dj-1].
template <typename T>
__device__ __forceinline__ T box2d9(T r00, T r01, T r02, T r10, T r11, T r12, T r20, T r21,
                                    T r22, const Coef<T>& k) {
  T acc = r00;
  acc = acc + r01; acc = acc + r02;
  acc = acc + r10; acc = acc + r11; acc = acc + r12;
  acc = acc + r20; acc = acc + r21; acc = acc + r22;
  return k.k0 * acc;
}
// laplacian / heat 3D 7-point: 7 loads, 8 FLOPs.
template <typename T>
__device__ __forceinline__ T star3d7(T c, T n, T s, T w, T e, T u, T d, const Coef<T>& k) {
  return k.k0 * c + k.k1 * (((((n + s) + w) + e) + u) + d);
}
// gradient 3D: 7 loads, 21 FLOPs (Table 3 lists 20; reading R8).
template <typename T>
__device__ __forceinline__ T gradient3d(T c, T n, T s, T w, T e, T u, T d, const Coef<T>& k) {
  T dn = c - n, ds = c - s, dw = c - w, de = c - e, du = c - u, dd = c - d;
  T acc = dn * dn;
  acc = acc + ds * ds;
  acc = acc + dw * dw;
  acc = acc + de * de;
  acc = acc + du * du;
  acc = acc + dd * dd;
  return c + dev_rcp_div<T>(dev_sqrt<T>(k.k0 + acc));
}
// FDTD-2D statements (PolyBench order ey, ex, hz; in place; k0 = 0.5, k1 = 0.7).
template <typename T>
__device__ __forceinline__ T fdtd_ey(T ey, T hz, T hz_im1, const Coef<T>& k) {
  return ey - k.k0 * (hz - hz_im1);
}
template <typename T>
__device__ __forceinline__ T fdtd_ex(T ex, T hz, T hz_jm1, const Coef<T>& k) {
  return ex - k.k0 * (hz - hz_jm1);
}
template <typename T>
__device__ __forceinline__ T fdtd_hz(T hz, T ex_jp1, T ex, T ey_ip1, T ey, const Coef<T>& k) {
  return hz - k.k1 * (((ex_jp1 - ex) + ey_ip1) - ey);
}

// Generic evaluation from memory (used by the generic and naive kernels).
// p = linear index of the point, s0/s1 = strides of the slowest / middle dimension.
template <typename T, int KIND>
__device__ __forceinline__ T point_from_memory(const T* __restrict__ A, int64_t p, int64_t s0,
                                               int64_t s1, const Coef<T>& k) {
  if constexpr (KIND == K_JACOBI2D5) {
    return jacobi2d5<T>(A[p], A[p - s0], A[p + s0], A[p - 1], A[p + 1], k);
  } else if constexpr (KIND == K_STAR2D5) {
    return star2d5<T>(A[p], A[p - s0], A[p + s0], A[p - 1], A[p + 1], k);
  } else if constexpr (KIND == K_GRADIENT2D) {
    return gradient2d<T>(A[p], A[p - s0], A[p + s0], A[p - 1], A[p + 1], k);
  } else if constexpr (KIND == K_BOX2D9) {
    return box2d9<T>(A[p - s0 - 1], A[p - s0], A[p - s0 + 1], A[p - 1], A[p], A[p + 1],
                     A[p + s0 - 1], A[p + s0], A[p + s0 + 1], k);
  } else if constexpr (KIND == K_STAR3D7) {
    return star3d7<T>(A[p], A[p - s1], A[p + s1], A[p - 1], A[p + 1], A[p - s0], A[p + s0], k);
  } else if constexpr (KIND == K_GRADIENT3D) {
    return gradient3d<T>(A[p], A[p - s1], A[p + s1], A[p - 1], A[p + 1], A[p - s0], A[p + s0], k);
  } else if constexpr (KIND == K_BOX3D27) {
    T acc = A[p - s0 - s1 - 1];
#pragma unroll
    for (int q = 1; q < 27; ++q) {
      const int dz = q / 9 - 1, dy = (q / 3) % 3 - 1, dx = q % 3 - 1;
      acc = acc + A[p + dz * s0 + dy * s1 + dx];
    }
    return k.k0 * acc;
  } else {
    return A[p];
  }
}

}  // namespace hexs
