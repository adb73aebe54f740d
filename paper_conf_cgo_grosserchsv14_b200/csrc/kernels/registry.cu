// registry.cu -- maps (class, dtype, h, w0) to compiled fast-kernel variants.
#include "../internal.h"
#include "../stencil_ops.cuh"
#include "fast2d_variants.h"
#include "fast3d_variants.h"
#include "stream3d_variants.h"
#include "launch.h"

namespace hexs {

#define HEXS_DECL(id, dc, T_, KIND_, H_, W0_, NW_)                              \
  cudaError_t launch_fast2d_v##id(const Fast2DArgs& a, int grid, cudaStream_t s); \
  int fast2d_chunk_v##id();
HEXS_FAST2D_VARIANTS(HEXS_DECL)
#undef HEXS_DECL

int fast2d_variant(int kind, int dtype, int h, int w0, int w1) {
#define HEXS_MATCH(id, dc, T_, KIND_, H_, W0_, NW_)                  \
  if (kind == KIND_ && dtype == dc && h == H_ && w0 == W0_ &&         \
      (w1 <= 0 || w1 == NW_ * 32 * (int)(16 / sizeof(T_)))) return id;
  HEXS_FAST2D_VARIANTS(HEXS_MATCH)
#undef HEXS_MATCH
  return -1;
}

int fast2d_variant_count() {
  int n = 0;
#define HEXS_CNT(id, dc, T_, KIND_, H_, W0_, NW_) ++n;
  HEXS_FAST2D_VARIANTS(HEXS_CNT)
#undef HEXS_CNT
  return n;
}
bool fast2d_variant_info(int variant, int* kind, int* dtype, int* h, int* w0) {
#define HEXS_INFO(id, dc, T_, KIND_, H_, W0_, NW_) \
  if (variant == id) {                            \
    *kind = KIND_; *dtype = dc; *h = H_; *w0 = W0_; \
    return true;                                  \
  }
  HEXS_FAST2D_VARIANTS(HEXS_INFO)
#undef HEXS_INFO
  return false;
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
// 3D fast kernel: the compiled (class, dtype, h, w0) instantiations of fast3d_variants.h.
#define HEXS_F3_DECL(id, dc, T_, KIND_, H_, W0_, NY_, MINB_, ZS_, NX_) \
  cudaError_t launch_fast3d_v##id(const Fast3DArgs& a, cudaStream_t s);
HEXS_FAST3D_VARIANTS(HEXS_F3_DECL)
#undef HEXS_F3_DECL

int fast3d_variant(int kind, int dtype, int h, int w0, int wy) {
#define HEXS_F3_MATCH(id, dc, T_, KIND_, H_, W0_, NY_, MINB_, ZS_, NX_) \
  if (kind == KIND_ && dtype == dc && h == H_ && w0 == W0_ && (wy <= 0 || wy == NY_)) return id;
  HEXS_FAST3D_VARIANTS(HEXS_F3_MATCH)
#undef HEXS_F3_MATCH
  return -1;
}
int fast3d_variant_count() { return HEXS_FAST3D_COUNT; }
bool fast3d_variant_info(int variant, int* kind, int* dtype, int* h, int* w0) {
#define HEXS_F3_INFO(id, dc, T_, KIND_, H_, W0_, NY_, MINB_, ZS_, NX_) \
  if (variant == id) {                                           \
    *kind = KIND_; *dtype = dc; *h = H_; *w0 = W0_;              \
    return true;                                                 \
  }
  HEXS_FAST3D_VARIANTS(HEXS_F3_INFO)
#undef HEXS_F3_INFO
  return false;
}
bool fast3d_variant_matches(int variant, int kind, int dtype, int h, int w0) {
#define HEXS_F3_IS(id, dc, T_, KIND_, H_, W0_, NY_, MINB_, ZS_, NX_) \
  if (variant == id) return kind == KIND_ && dtype == dc && h == H_ && w0 == W0_;
  HEXS_FAST3D_VARIANTS(HEXS_F3_IS)
#undef HEXS_F3_IS
  return false;
}
int fast3d_tile(int variant, int* wy, int* wx) {
  *wy = 0;
  *wx = 0;
#define HEXS_F3_NY(id, dc, T_, KIND_, H_, W0_, NY_, MINB_, ZS_, NX_) \
  if (variant == id) {                                           \
    *wy = NY_;                                                   \
    *wx = NX_;                                                   \
  }
  HEXS_FAST3D_VARIANTS(HEXS_F3_NY)
#undef HEXS_F3_NY
  return *wy > 0 ? 0 : -1;
}
cudaError_t launch_fast3d(int variant, const Fast3DArgs& a, int /*grid: persistent*/, cudaStream_t s) {
  switch (variant) {
#define HEXS_F3_L(id, dc, T_, KIND_, H_, W0_, NY_, MINB_, ZS_, NX_) \
  case id: return launch_fast3d_v##id(a, s);
    HEXS_FAST3D_VARIANTS(HEXS_F3_L)
#undef HEXS_F3_L
    default: return cudaErrorInvalidValue;
  }
}

// Streaming 3D kernel: the compiled (class, h, w0) instantiations of stream3d_variants.h.
#define HEXS_S3_DECL(id, dc, T_, KIND_, H_, W0_, NXS_)                                \
  cudaError_t launch_stream3d_v##id(const Stream3DArgs& a, cudaStream_t s); \
  int stream3d_carry_block_v##id();
HEXS_STREAM3D_VARIANTS(HEXS_S3_DECL)
#undef HEXS_S3_DECL

int stream3d_variant(int kind, int dtype, int h, int w0) {
#define HEXS_S3_MATCH(id, dc, T_, KIND_, H_, W0_, NXS_) \
  if (kind == KIND_ && dtype == dc && h == H_ && w0 == W0_) return id;
  HEXS_STREAM3D_VARIANTS(HEXS_S3_MATCH)
#undef HEXS_S3_MATCH
  return -1;
}
int stream3d_carry_block(int variant) {
  switch (variant) {
#define HEXS_S3_CB(id, dc, T_, KIND_, H_, W0_, NXS_) case id: return stream3d_carry_block_v##id();
    HEXS_STREAM3D_VARIANTS(HEXS_S3_CB)
#undef HEXS_S3_CB
    default: return 0;
  }
}
cudaError_t launch_stream3d(int variant, const Stream3DArgs& a, cudaStream_t s) {
  switch (variant) {
#define HEXS_S3_L(id, dc, T_, KIND_, H_, W0_, NXS_) case id: return launch_stream3d_v##id(a, s);
    HEXS_STREAM3D_VARIANTS(HEXS_S3_L)
#undef HEXS_S3_L
    default: return cudaErrorInvalidValue;
  }
}

}  // namespace hexs
