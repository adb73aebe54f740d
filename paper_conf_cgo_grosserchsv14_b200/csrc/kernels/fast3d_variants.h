// fast3d_variants.h -- the compiled instantiations of the 3D phase kernel (kernels/hex3d.cu):
// X(id, dtype_code, T, KIND, h, w0, NY, MINB, ZS, NX): NY tile lines (y), MINB CTAs per SM, ZS
// threads per column (each sweeps 1/ZS of a level's rows), NX tile columns (x).  The
// hexagon shape is a compile-time parameter (every level's row range is unrolled, "constraint-based unrolling"); each id is
// compiled from hex3d.cu with -DHEXS_F3_VARIANT=id into its own object (parallel build).
// The first entry of a (class, dtype, h, w0) is its default: star3d7 fp32 (3, 7) runs 16 x 64 (y, x)
// tiles (596 vs 567 GUp/s for 32 x 32 on heat-3D 512^3; 8 x 128: 427; the 27-point and gradient sweeps
// measured equal or slower at 16 x 64; deeper / wider hexagons at 16 x 64, compiled for the sweep and
// removed: (4,7) 441, (3,9) 571 GUp/s, both bit-exact).  (2, 7) is the default 3D tile (Table 4's h = 2); the star3d7 fp32
// shapes serve the tile sweep and the tests; the long gradient / 27-point expressions split each
// column's rows over 2 threads (ZS = 2: 16 compute warps hide their latency; gradient 232 -> 321
// GUp/s); a
// tile whose classical width w[0] is set selects the variant with NY = w[0].  Other (h, w0) run the generic hybrid kernel.
#pragma once
#define HEXS_FAST3D_VARIANTS(X)                 \
  X(0, 0, float, K_STAR3D7, 2, 7, 32, 1, 1, 32)     \
  X(1, 1, double, K_STAR3D7, 2, 7, 16, 1, 1, 32)    \
  X(2, 0, float, K_GRADIENT3D, 2, 7, 32, 1, 2, 32)  \
  X(3, 1, double, K_GRADIENT3D, 2, 7, 16, 1, 1, 32) \
  X(4, 0, float, K_BOX3D27, 2, 7, 32, 1, 2, 32)     \
  X(5, 1, double, K_BOX3D27, 2, 7, 16, 1, 1, 32)    \
  X(6, 0, float, K_STAR3D7, 1, 3, 16, 2, 1, 32)     \
  X(7, 0, float, K_STAR3D7, 3, 2, 16, 2, 1, 32)     \
  X(8, 0, float, K_STAR3D7, 2, 3, 32, 1, 1, 32)     \
  X(16, 0, float, K_STAR3D7, 3, 7, 16, 1, 1, 64)   \
  X(9, 0, float, K_STAR3D7, 3, 7, 32, 1, 1, 32)     \
  X(10, 0, float, K_STAR3D7, 1, 7, 32, 1, 1, 32)    \
  X(11, 0, float, K_STAR3D7, 2, 5, 32, 1, 1, 32)    \
  X(12, 0, float, K_STAR3D7, 3, 5, 32, 1, 1, 32)    \
  X(13, 0, float, K_STAR3D7, 2, 7, 16, 2, 1, 32)    \
  X(14, 0, float, K_STAR3D7, 1, 3, 32, 2, 1, 32)    \
  X(15, 0, float, K_STAR3D7, 2, 7, 32, 1, 2, 32)    \
  X(17, 0, float, K_STAR3D7, 3, 7, 8, 1, 1, 128)   \
  X(18, 0, float, K_BOX3D27, 2, 7, 16, 1, 2, 64)   \
  X(19, 0, float, K_GRADIENT3D, 2, 7, 16, 1, 2, 64) \
  X(20, 0, float, K_STAR3D7, 2, 7, 16, 1, 1, 64)
#define HEXS_FAST3D_COUNT 21
