// registry.cu -- maps (class, dtype, h, w0) to compiled fast-kernel variants.
#include "../internal.h"
#include "../stencil_ops.cuh"
#include "fast2d_variants.h"
#include "launch.h"

namespace hexs {

#define HEXS_DECL(id, dc, T_, KIND_, H_, W0_, NW_)                              \
  cudaError_t launch_fast2d_v##id(const Fast2DArgs& a, int grid, cudaStream_t s); \
  int fast2d_chunk_v##id();
HEXS_FAST2D_VARIANTS(HEXS_DECL)
#undef HEXS_DECL

int fast2d_variant(int kind, int dtype, int h, int w0) {
#define HEXS_MATCH(id, dc, T_, KIND_, H_, W0_, NW_) \
  if (kind == KIND_ && dtype == dc && h == H_ && w0 == W0_) return id;
  HEXS_FAST2D_VARIANTS(HEXS_MATCH)
#undef HEXS_MATCH
  return -1;
}

int fast2d_chunk_width(int variant) {
  switch (variant) {
#define HEXS_W(id, dc, T_, KIND_, H_, W0_, NW_) case id: return fast2d_chunk_v##id();
    HEXS_FAST2D_VARIANTS(HEXS_W)
#undef HEXS_W
    default: return 0;
  }
}

cudaError_t launch_fast2d(int variant, const Fast2DArgs& a, int grid, cudaStream_t s) {
  switch (variant) {
#define HEXS_L(id, dc, T_, KIND_, H_, W0_, NW_) case id: return launch_fast2d_v##id(a, grid, s);
    HEXS_FAST2D_VARIANTS(HEXS_L)
#undef HEXS_L
    default: return cudaErrorInvalidValue;
  }
}

// FDTD-2D fast kernel: any (h, w0) whose hexagon (W = 2 w0 + 2 + h + floor(h/2) rows, delta0
// = 1, delta1 = 1/2) fits the shared-memory ring and whose 2h+2 levels fit one ring block.
int fdtd_variant(int dtype, int h, int w0) {
  const int W = 2 * w0 + 2 + h + h / 2;
  if (2 * h + 2 > 64 || W > 40 || fdtd_smem_bytes(dtype, W) > 200 * 1024) return -1;
  return dtype == 1 ? 1 : 0;
}
// 3D fast kernel: any (h, w0) whose two level buffers fit in shared memory
// (2 x (w0 + 2h + 3) rows x (main + carry lines + carry columns) of one classical tile).
int fast3d_variant(int kind, int dtype, int h, int w0) {
  if (kind != K_STAR3D7 && kind != K_GRADIENT3D && kind != K_BOX3D27) return -1;
  const int Q = w0 + 2 * h + 3;
  if (fast3d_smem_bytes(dtype, Q) > 200 * 1024 || 2 * h + 2 > kMaxH) return -1;
  return kind * 2 + dtype;
}
int fast3d_tile(int variant, int* wy, int* wx) {
  *wy = fast3d_tile_lines(variant & 1);
  *wx = kFast3DNX;
  return 0;
}

}  // namespace hexs
