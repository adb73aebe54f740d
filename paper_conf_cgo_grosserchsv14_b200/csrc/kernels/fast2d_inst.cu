// fast2d_inst.cu -- compiled once per variant id (-DHEXS_VARIANT=<id>); defines
// hexs::launch_fast2d_v<id>() for the (dtype, class, h, w0, NW) of fast2d_variants.h.
#include "fast2d_variants.h"
#include "devcache.h"
#include "hex2d_impl.cuh"

#ifndef HEXS_VARIANT
#error "compile with -DHEXS_VARIANT=<id>"
#endif

namespace hexs {

template <int ID> struct Sel;
#define HEXS_SEL(id, dc, T_, KIND_, H_, W0_, NW_) \
  template <> struct Sel<id> { using K = fast2d::Kernel<T_, KIND_, H_, W0_, NW_>; };
HEXS_FAST2D_VARIANTS(HEXS_SEL)
#undef HEXS_SEL

#define HEXS_CAT2(a, b) a##b
#define HEXS_CAT(a, b) HEXS_CAT2(a, b)
using KSel = Sel<HEXS_VARIANT>::K;

// Full-time hexagons on 16-B aligned rows: TMA-staged In rows (the hot kernel).
__global__ void __launch_bounds__(KSel::NT, KSel::MINB)
HEXS_CAT(fast2d_kernel_v, HEXS_VARIANT)(const __grid_constant__ Fast2DArgs g) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  KSel::run_tma(g, *reinterpret_cast<KSel::Smem*>(smem_raw));
}
// Full-time hexagons on unaligned rows (direct loads).
__global__ void __launch_bounds__(KSel::NT, 1)
HEXS_CAT(fast2d_kernel_unaligned_v, HEXS_VARIANT)(const __grid_constant__ Fast2DArgs g) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  KSel::template run_direct<false>(g, *reinterpret_cast<KSel::Smem*>(smem_raw));
}
// Hexagons cut by t = 0 or t = T_steps (levels outside [a_lo, a_hi] skipped).
__global__ void __launch_bounds__(KSel::NT, 1)
HEXS_CAT(fast2d_kernel_tcut_v, HEXS_VARIANT)(const __grid_constant__ Fast2DArgs g) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  KSel::template run_direct<true>(g, *reinterpret_cast<KSel::Smem*>(smem_raw));
}

cudaError_t HEXS_CAT(launch_fast2d_v, HEXS_VARIANT)(const Fast2DArgs& a, int grid, cudaStream_t s) {
  static DeviceMemo<int> attr;  // per device: dynamic shared-memory opt-in done
  const int smem = (int)sizeof(KSel::Smem);
  int done = 0;
  cudaError_t e = attr.get(&done, [&](int, int* v) {
    cudaError_t r = cudaFuncSetAttribute(HEXS_CAT(fast2d_kernel_v, HEXS_VARIANT),
                                         cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
    if (r == cudaSuccess)
      r = cudaFuncSetAttribute(HEXS_CAT(fast2d_kernel_unaligned_v, HEXS_VARIANT),
                               cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
    if (r == cudaSuccess)
      r = cudaFuncSetAttribute(HEXS_CAT(fast2d_kernel_tcut_v, HEXS_VARIANT),
                               cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
    *v = 1;
    return r;
  });
  if (e != cudaSuccess) return e;
  const bool aligned = ((a.N1 * (int64_t)sizeof(KSel::Elem)) % 16) == 0;
  if (a.a_lo > 0 || a.a_hi < KSel::L - 1)
    HEXS_CAT(fast2d_kernel_tcut_v, HEXS_VARIANT)<<<grid, KSel::NT, smem, s>>>(a);
  else if (aligned)
    HEXS_CAT(fast2d_kernel_v, HEXS_VARIANT)<<<grid, KSel::NT, smem, s>>>(a);
  else
    HEXS_CAT(fast2d_kernel_unaligned_v, HEXS_VARIANT)<<<grid, KSel::NT, smem, s>>>(a);
  return cudaGetLastError();
}

int HEXS_CAT(fast2d_chunk_v, HEXS_VARIANT)() { return KSel::C; }

}  // namespace hexs
