// stream3d_variants.h -- compiled instantiations of the streaming 3D phase kernel
// (kernels/stream3d.cu): X(id, dtype_code, T, KIND, h, w0, NXS).  NXS = depth of the
// shared-memory exchange ring (4: two steps of TMA lead; 3 for the taller (3, w0) hexagons so
// that two CTAs still fit one SM).  w0 must be odd (the hexagon's 2h+w0+1 rows pair up into
// warps of two mirror rows with identical level ranges).  Each id is compiled from stream3d.cu
// with -DHEXS_S3_VARIANT=id into its own object.
#pragma once
#define HEXS_STREAM3D_VARIANTS(X)          \
  X(0, 0, float, K_STAR3D7, 2, 7, 4)       \
  X(1, 0, float, K_STAR3D7, 3, 7, 3)       \
  X(2, 0, float, K_STAR3D7, 2, 5, 4)       \
  X(3, 0, float, K_STAR3D7, 3, 5, 4)       \
  X(4, 0, float, K_STAR3D7, 1, 7, 4)       \
  X(5, 0, float, K_GRADIENT3D, 2, 7, 4)    \
  X(6, 0, float, K_GRADIENT3D, 1, 7, 4)    \
  X(7, 0, float, K_STAR3D7, 1, 3, 4)
