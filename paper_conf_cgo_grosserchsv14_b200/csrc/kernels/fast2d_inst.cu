// fast2d_inst.cu -- compiled once per variant id (-DHEXS_VARIANT=<id>); defines
// hexs::launch_fast2d_v<id>() for the (dtype, class, h, w0, NW) of fast2d_variants.h.
#include "fast2d_variants.h"
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

#ifndef HEXS_MINB
#define HEXS_MINB KSel::MINB
#endif

// Full-time hexagons (every launch except the first and last ones of a run).
__global__ void __launch_bounds__(KSel::NT, HEXS_MINB)
HEXS_CAT(fast2d_kernel_v, HEXS_VARIANT)(const __grid_constant__ Fast2DArgs g) {
  __shared__ KSel::Smem sm;
  KSel::template run<false>(g, sm);
}
// Hexagons cut by t = 0 or t = T_steps (levels outside [a_lo, a_hi] skipped).
__global__ void __launch_bounds__(KSel::NT, 1)
HEXS_CAT(fast2d_kernel_tcut_v, HEXS_VARIANT)(const __grid_constant__ Fast2DArgs g) {
  __shared__ KSel::Smem sm;
  KSel::template run<true>(g, sm);
}

cudaError_t HEXS_CAT(launch_fast2d_v, HEXS_VARIANT)(const Fast2DArgs& a, int grid, cudaStream_t s) {
  if (a.a_lo > 0 || a.a_hi < KSel::L - 1)
    HEXS_CAT(fast2d_kernel_tcut_v, HEXS_VARIANT)<<<grid, KSel::NT, 0, s>>>(a);
  else
    HEXS_CAT(fast2d_kernel_v, HEXS_VARIANT)<<<grid, KSel::NT, 0, s>>>(a);
  return cudaGetLastError();
}

int HEXS_CAT(fast2d_chunk_v, HEXS_VARIANT)() { return KSel::C; }

}  // namespace hexs
