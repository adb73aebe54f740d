// fast2d_variants.h -- the compiled instantiations of the fast 2D kernel:
// X(id, dtype_code, T, KIND, h, w0, NW).  Each id is compiled from fast2d_inst.cu with
// -DHEXS_VARIANT=id into its own object (parallel build).  (3, 7) is the default tile
// (DESIGN.md "tile selection"); the others serve the tile sweep and the tests.
#pragma once
#define HEXS_FAST2D_VARIANTS(X)                  \
  X(0, 0, float, K_STAR2D5, 3, 7, 4)             \
  X(1, 0, float, K_JACOBI2D5, 3, 7, 4)           \
  X(2, 0, float, K_BOX2D9, 3, 7, 4)              \
  X(3, 0, float, K_GRADIENT2D, 3, 7, 4)          \
  X(4, 1, double, K_STAR2D5, 3, 7, 4)            \
  X(5, 1, double, K_JACOBI2D5, 3, 7, 4)          \
  X(6, 1, double, K_BOX2D9, 3, 7, 4)             \
  X(7, 1, double, K_GRADIENT2D, 3, 7, 4)         \
  X(8, 0, float, K_STAR2D5, 1, 3, 4)             \
  X(9, 0, float, K_STAR2D5, 3, 10, 4)            \
  X(10, 0, float, K_STAR2D5, 2, 5, 4)            \
  X(11, 0, float, K_STAR2D5, 3, 5, 4)            \
  X(12, 0, float, K_STAR2D5, 4, 5, 4)            \
  X(13, 0, float, K_JACOBI2D5, 1, 3, 4)          \
  X(14, 0, float, K_BOX2D9, 3, 5, 4)             \
  X(15, 0, float, K_BOX2D9, 2, 5, 4)             \
  X(16, 0, float, K_BOX2D9, 2, 7, 4)             \
  X(17, 0, float, K_BOX2D9, 4, 5, 4)             \
  X(18, 0, float, K_BOX2D9, 3, 7, 8)             \
  X(19, 0, float, K_GRADIENT2D, 1, 3, 4)         \
  X(20, 0, float, K_GRADIENT2D, 2, 3, 4)         \
  X(21, 0, float, K_GRADIENT2D, 1, 1, 4)         \
  X(22, 0, float, K_STAR2D5, 2, 7, 4)            \
  X(23, 0, float, K_STAR2D5, 2, 9, 4)            \
  X(24, 0, float, K_BOX2D9, 2, 9, 4)             \
  X(25, 0, float, K_STAR2D5, 3, 9, 4)          \
  X(26, 0, float, K_STAR2D5, 2, 8, 4)          \
  X(27, 0, float, K_STAR2D5, 2, 6, 4)
#define HEXS_FAST2D_COUNT 28
