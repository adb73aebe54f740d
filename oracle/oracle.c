/*
 * oracle.c -- the plain, slow, obviously-correct CPU oracle for the hot path of
 * Grosser, Cohen, Holewinski, Sadayappan, Verdoolaege, "Hybrid Hexagonal/Classical
 * Tiling for GPUs", CGO'14.
 *
 * TEST INFRASTRUCTURE ONLY.  Only tests/, __graft_entry__.smoke() and bench.py's
 * cpu_baseline / `--impl reference` legs may load this library.  The product path
 * (paper_conf_cgo_grosserchsv14_b200/) never links, imports or calls it, and shares
 * no header, helper, table or constant with it.
 *
 * WHAT IT COMPUTES.  Hybrid tiling only reorders statement instances; every instance
 * is executed exactly once by the same expression from the same inputs ("we perform
 * no redundant computations", Sec. 2; the schedule is a bijection,
 * Sec. 3.3.3 / 3.6).  The result of the method is therefore exactly
 * the result of the original time loop of Fig. 1.  This file IS that
 * loop, written out for each stencil class, with a fixed per-point operation order:
 *
 *   buf0 = in; buf1 = in                       (both ping-pong buffers start as `in`,
 *                                               so Dirichlet boundary cells are valid in
 *                                               either parity -- DESIGN.md reading R10)
 *   for t in 0..T-1:  for every interior point p:  buf[(t+1)%2][p] = f(buf[t%2], p)
 *   out = buf[T%2]
 *
 * Interior = every coordinate in [1, N_d-2] (Fig. 1 loops i,j = 1..N-2).
 * FDTD-2D is the three-statement in-place kernel of Table 3 in
 * PolyBench form without the source row (reading R9).
 *
 * Per-point expressions (left-to-right association exactly as written, no contraction;
 * built with -ffp-contract=off, no fast-math; readings R7, R8, R13):
 *   jacobi2d5  : k*((((c+s)+n)+e)+w)            k = coef[0] (default 0.2f = 0x3E4CCCCD,
 *                s=A[i+1][j] n=A[i-1][j]         Fig. 1 operand order PAPER.md:146-148,
 *                e=A[i][j+1] w=A[i][j-1]         Fig. 2 add x4 then mul)
 *   star2d5    : c0*c + c1*(((n+s)+w)+e)        (laplacian 2D, 5 loads / 6 FLOPs, Table 3)
 *   box2d9     : k*(sum of the 3x3 box, row-major)  (heat 2D, 9 / 9, Table 3)
 *   gradient2d : c + 1/sqrt(eps + ((((c-n)^2+(c-s)^2)+(c-w)^2)+(c-e)^2))   (5 / 15)
 *   star3d7    : c0*c + c1*(((((n+s)+w)+e)+u)+d)  (laplacian 3D, 7 / 8)
 *                 u=A[z-1] d=A[z+1] n=A[.][y-1] s=A[.][y+1] w=A[..][x-1] e=A[..][x+1]
 *   box3d27    : k*(sum of the 3x3x3 box, lexicographic)   (heat 3D, 27 / 27)
 *   gradient3d : c + 1/sqrt(eps + sum_{n,s,w,e,u,d} (c-nb)^2)   (7 / 21; paper says 20)
 *   fdtd2d     : ey[i][j] -= ce*(hz[i][j]-hz[i-1][j])        i in [1,N0), j in [0,N1)
 *                ex[i][j] -= ce*(hz[i][j]-hz[i][j-1])        i in [0,N0), j in [1,N1)
 *                hz[i][j] -= ch*(((ex[i][j+1]-ex[i][j])+ey[i+1][j])-ey[i][j])
 *                                                            i in [0,N0-1), j in [0,N1-1)
 *                (x -= k*y means x = x - k*y; ce = coef[0] = 0.5, ch = coef[1] = 0.7)
 *
 * Coefficients arrive as doubles and are rounded once to the working precision
 * (C cast, round-to-nearest-even).  Pins (tests/test_oracle_*.py): Fig. 1/2 golden
 * 8x8 values, constant-field fixpoints, exact Dirichlet sine-mode eigenvalue decay,
 * scipy.ndimage.correlate iteration, exact integer path counting, the FDTD discrete
 * wave identity, gradient ramp closed form, cone sampler == full run.
 */
#include <math.h>
#include <stdint.h>
#include <stdlib.h>
#include <string.h>
#ifdef _OPENMP
#include <omp.h>
#endif

/* Stencil classes (oracle-local numbering; tests map them by name). */
enum {
  OR_JACOBI2D5 = 0, OR_STAR2D5 = 1, OR_BOX2D9 = 2, OR_FDTD2D = 3,
  OR_STAR3D7 = 4, OR_GRADIENT3D = 5, OR_BOX3D27 = 6, OR_GRADIENT2D = 7
};

int oracle_abi_version(void) { return 1; }

static int kind_dims(int kind) {
  switch (kind) {
    case OR_JACOBI2D5: case OR_STAR2D5: case OR_BOX2D9: case OR_FDTD2D: case OR_GRADIENT2D: return 2;
    case OR_STAR3D7: case OR_GRADIENT3D: case OR_BOX3D27: return 3;
    default: return 0;
  }
}

/* ------------------------------------------------------------------------------------
 * One interior point of a single-field stencil.  A = source level, p = linear index,
 * s0/s1 = strides of the two outer dimensions (s1 unused in 2D).  Written once as a
 * macro so that the float and double oracles are the same text.
 * ---------------------------------------------------------------------------------- */
#define ORACLE_POINT(T, SQRT)                                                          \
  static T point_##T(int kind, const T *A, int64_t p, int64_t s0, int64_t s1,         \
                     const T *k) {                                                     \
    switch (kind) {                                                                    \
      case OR_JACOBI2D5: {                                                             \
        T c = A[p], s = A[p + s0], n = A[p - s0], e = A[p + 1], w = A[p - 1];          \
        return k[0] * ((((c + s) + n) + e) + w);                                       \
      }                                                                                \
      case OR_STAR2D5: {                                                               \
        T c = A[p], n = A[p - s0], s = A[p + s0], w = A[p - 1], e = A[p + 1];          \
        return k[0] * c + k[1] * (((n + s) + w) + e);                                  \
      }                                                                                \
      case OR_BOX2D9: {                                                                \
        T acc = A[p - s0 - 1];                                                         \
        acc = acc + A[p - s0];     acc = acc + A[p - s0 + 1];                          \
        acc = acc + A[p - 1];      acc = acc + A[p];          acc = acc + A[p + 1];    \
        acc = acc + A[p + s0 - 1]; acc = acc + A[p + s0];     acc = acc + A[p + s0 + 1]; \
        return k[0] * acc;                                                             \
      }                                                                                \
      case OR_GRADIENT2D: {                                                            \
        T c = A[p];                                                                    \
        T dn = c - A[p - s0], ds = c - A[p + s0], dw = c - A[p - 1], de = c - A[p + 1]; \
        T acc = dn * dn;                                                               \
        acc = acc + ds * ds; acc = acc + dw * dw; acc = acc + de * de;                 \
        return c + (T)1 / SQRT(k[0] + acc);                                            \
      }                                                                                \
      case OR_STAR3D7: {                                                               \
        T c = A[p], n = A[p - s1], s = A[p + s1], w = A[p - 1], e = A[p + 1];          \
        T u = A[p - s0], d = A[p + s0];                                                \
        return k[0] * c + k[1] * (((((n + s) + w) + e) + u) + d);                      \
      }                                                                                \
      case OR_GRADIENT3D: {                                                            \
        T c = A[p];                                                                    \
        T dn = c - A[p - s1], ds = c - A[p + s1], dw = c - A[p - 1], de = c - A[p + 1]; \
        T du = c - A[p - s0], dd = c - A[p + s0];                                      \
        T acc = dn * dn;                                                               \
        acc = acc + ds * ds; acc = acc + dw * dw; acc = acc + de * de;                 \
        acc = acc + du * du; acc = acc + dd * dd;                                      \
        return c + (T)1 / SQRT(k[0] + acc);                                            \
      }                                                                                \
      case OR_BOX3D27: {                                                               \
        T acc = (T)0; int first = 1;                                                   \
        for (int dz = -1; dz <= 1; ++dz)                                               \
          for (int dy = -1; dy <= 1; ++dy)                                             \
            for (int dx = -1; dx <= 1; ++dx) {                                         \
              T v = A[p + dz * s0 + dy * s1 + dx];                                     \
              if (first) { acc = v; first = 0; } else { acc = acc + v; }               \
            }                                                                          \
        return k[0] * acc;                                                             \
      }                                                                                \
    }                                                                                  \
    return (T)0;                                                                       \
  }

ORACLE_POINT(float, sqrtf)
ORACLE_POINT(double, sqrt)

/* Number of coefficients each class consumes and their defaults (R7). */
static int n_coef(int kind) {
  switch (kind) {
    case OR_STAR2D5: case OR_STAR3D7: case OR_FDTD2D: return 2;
    default: return 1;
  }
}

/* ------------------------------------------------------------------------------------
 * Full naive time loop, single-field classes.  ext = extents slow->fast, row-major.
 * ---------------------------------------------------------------------------------- */
#define ORACLE_RUN(T)                                                                  \
  int oracle_run_##T(int kind, int dims, const int64_t *ext, const double *coef,       \
                     int ncoef, int64_t steps, const T *in, T *out, int nthreads) {    \
    if (kind == OR_FDTD2D || kind_dims(kind) != dims || ncoef < n_coef(kind) ||        \
        steps < 0)                                                                     \
      return 1;                                                                        \
    T k[2] = {(T)coef[0], ncoef > 1 ? (T)coef[1] : (T)0};                              \
    int64_t N0 = ext[0], N1 = ext[1], N2 = dims == 3 ? ext[2] : 1;                     \
    int64_t n = N0 * N1 * N2;                                                          \
    T *buf[2];                                                                         \
    buf[0] = out;                                                                      \
    buf[1] = (T *)malloc((size_t)n * sizeof(T));                                       \
    if (!buf[1]) return 2;                                                             \
    memmove(buf[0], in, (size_t)n * sizeof(T));                                        \
    memcpy(buf[1], in, (size_t)n * sizeof(T));                                         \
    int64_t s0 = dims == 3 ? N1 * N2 : N1, s1 = dims == 3 ? N2 : 0;                    \
    if (nthreads < 1) nthreads = 1;                                                    \
    for (int64_t t = 0; t < steps; ++t) {                                              \
      const T *src = buf[t % 2];                                                       \
      T *dst = buf[(t + 1) % 2];                                                       \
      if (dims == 2) {                                                                 \
        _Pragma("omp parallel for schedule(static) num_threads(nthreads)")             \
        for (int64_t i = 1; i < N0 - 1; ++i)                                           \
          for (int64_t j = 1; j < N1 - 1; ++j)                                         \
            dst[i * s0 + j] = point_##T(kind, src, i * s0 + j, s0, s1, k);             \
      } else {                                                                         \
        _Pragma("omp parallel for schedule(static) num_threads(nthreads)")             \
        for (int64_t z = 1; z < N0 - 1; ++z)                                           \
          for (int64_t y = 1; y < N1 - 1; ++y)                                         \
            for (int64_t x = 1; x < N2 - 1; ++x)                                       \
              dst[z * s0 + y * s1 + x] =                                               \
                  point_##T(kind, src, z * s0 + y * s1 + x, s0, s1, k);                \
      }                                                                                \
    }                                                                                  \
    if (steps % 2 == 1) memcpy(out, buf[1], (size_t)n * sizeof(T));                    \
    free(buf[1]);                                                                      \
    return 0;                                                                          \
  }

ORACLE_RUN(float)
ORACLE_RUN(double)

/* ------------------------------------------------------------------------------------
 * FDTD-2D, three in-place fields, statement order ey -> ex -> hz inside each step
 * (canonical time tau = 3t+k, Sec. 3.2).  Fields are updated in
 * place in ex, ey, hz (N0*N1 each).
 * ---------------------------------------------------------------------------------- */
#define ORACLE_FDTD(T)                                                                 \
  int oracle_fdtd_##T(const int64_t *ext, const double *coef, int ncoef, int64_t steps, \
                      T *ex, T *ey, T *hz, int nthreads) {                             \
    if (ncoef < 2 || steps < 0) return 1;                                              \
    const T ce = (T)coef[0], ch = (T)coef[1];                                          \
    const int64_t N0 = ext[0], N1 = ext[1];                                            \
    if (nthreads < 1) nthreads = 1;                                                    \
    for (int64_t t = 0; t < steps; ++t) {                                              \
      _Pragma("omp parallel for schedule(static) num_threads(nthreads)")               \
      for (int64_t i = 1; i < N0; ++i)                                                 \
        for (int64_t j = 0; j < N1; ++j)                                               \
          ey[i * N1 + j] = ey[i * N1 + j] - ce * (hz[i * N1 + j] - hz[(i - 1) * N1 + j]); \
      _Pragma("omp parallel for schedule(static) num_threads(nthreads)")               \
      for (int64_t i = 0; i < N0; ++i)                                                 \
        for (int64_t j = 1; j < N1; ++j)                                               \
          ex[i * N1 + j] = ex[i * N1 + j] - ce * (hz[i * N1 + j] - hz[i * N1 + j - 1]); \
      _Pragma("omp parallel for schedule(static) num_threads(nthreads)")               \
      for (int64_t i = 0; i < N0 - 1; ++i)                                             \
        for (int64_t j = 0; j < N1 - 1; ++j)                                           \
          hz[i * N1 + j] = hz[i * N1 + j] -                                            \
              ch * (((ex[i * N1 + j + 1] - ex[i * N1 + j]) + ey[(i + 1) * N1 + j]) -   \
                    ey[i * N1 + j]);                                                   \
    }                                                                                  \
    return 0;                                                                          \
  }

ORACLE_FDTD(float)
ORACLE_FDTD(double)

/* ------------------------------------------------------------------------------------
 * Cone sampler: the value at level `steps` of selected points, computed by the same
 * naive loop restricted to the box that can influence them (dependence radius 1 per
 * step for every class, so the box at level t is p +/- (steps - t), clipped to the
 * grid).  Used to check full-size GPU runs at sampled points.  Pinned against the
 * full run by tests/test_oracle_pins.py::test_cone_sampler_matches_full_run.
 * ---------------------------------------------------------------------------------- */
#define ORACLE_POINTS(T)                                                               \
  int oracle_points_##T(int kind, int dims, const int64_t *ext, const double *coef,    \
                        int ncoef, int64_t steps, const T *in, int npts,               \
                        const int64_t *coords, T *vals) {                              \
    if (kind == OR_FDTD2D || kind_dims(kind) != dims || ncoef < n_coef(kind)) return 1; \
    T k[2] = {(T)coef[0], ncoef > 1 ? (T)coef[1] : (T)0};                              \
    int64_t N[3] = {ext[0], ext[1], dims == 3 ? ext[2] : 1};                           \
    for (int q = 0; q < npts; ++q) {                                                   \
      int64_t P[3] = {coords[q * dims], coords[q * dims + 1],                          \
                      dims == 3 ? coords[q * dims + 2] : 0};                           \
      int64_t lo[3], hi[3], B[3];                                                      \
      for (int d = 0; d < 3; ++d) {                                                    \
        if (d < dims) {                                                                \
          lo[d] = P[d] - steps < 0 ? 0 : P[d] - steps;                                 \
          hi[d] = P[d] + steps > N[d] - 1 ? N[d] - 1 : P[d] + steps;                   \
        } else { lo[d] = 0; hi[d] = 0; }                                               \
        B[d] = hi[d] - lo[d] + 1;                                                      \
      }                                                                                \
      int64_t nb = B[0] * B[1] * B[2];                                                 \
      T *b0 = (T *)malloc((size_t)nb * sizeof(T)), *b1 = (T *)malloc((size_t)nb * sizeof(T)); \
      if (!b0 || !b1) { free(b0); free(b1); return 2; }                                \
      for (int64_t a = 0; a < B[0]; ++a)                                               \
        for (int64_t b = 0; b < B[1]; ++b)                                             \
          for (int64_t c = 0; c < B[2]; ++c) {                                         \
            int64_t g = dims == 3 ? ((lo[0] + a) * N[1] + (lo[1] + b)) * N[2] + lo[2] + c \
                                  : (lo[0] + a) * N[1] + (lo[1] + b);                  \
            b0[(a * B[1] + b) * B[2] + c] = in[g];                                     \
          }                                                                            \
      memcpy(b1, b0, (size_t)nb * sizeof(T));                                          \
      T *src = b0, *dst = b1;                                                          \
      int64_t bs0 = dims == 3 ? B[1] * B[2] : B[1], bs1 = dims == 3 ? B[2] : 0;        \
      for (int64_t t = 1; t <= steps; ++t) {                                           \
        int64_t rad = steps - t;                                                       \
        int64_t clo[3], chi[3];                                                        \
        for (int d = 0; d < dims; ++d) {                                               \
          clo[d] = P[d] - rad; chi[d] = P[d] + rad;                                    \
          if (clo[d] < 1) clo[d] = 1;                                                  \
          if (chi[d] > N[d] - 2) chi[d] = N[d] - 2;                                    \
        }                                                                              \
        if (dims == 2) { clo[2] = 0; chi[2] = 0; }                                     \
        for (int64_t a = clo[0]; a <= chi[0]; ++a)                                     \
          for (int64_t b = clo[1]; b <= chi[1]; ++b)                                   \
            for (int64_t c = clo[2]; c <= chi[2]; ++c) {                               \
              int64_t l = dims == 3                                                    \
                  ? ((a - lo[0]) * B[1] + (b - lo[1])) * B[2] + (c - lo[2])            \
                  : (a - lo[0]) * B[1] + (b - lo[1]);                                  \
              dst[l] = point_##T(kind, src, l, bs0, bs1, k);                           \
            }                                                                          \
        T *tmp = src; src = dst; dst = tmp;                                            \
      }                                                                                \
      int64_t l = dims == 3 ? ((P[0] - lo[0]) * B[1] + (P[1] - lo[1])) * B[2] + (P[2] - lo[2]) \
                            : (P[0] - lo[0]) * B[1] + (P[1] - lo[1]);                  \
      vals[q] = src[l];                                                                \
      free(b0); free(b1);                                                              \
    }                                                                                  \
    return 0;                                                                          \
  }

ORACLE_POINTS(float)
ORACLE_POINTS(double)

/* ------------------------------------------------------------------------------------
 * General linear stencil ("general descriptors"): any access set
 * of n offsets o_k (2D or 3D, any radius) with coefficients c_k, evaluated left to right
 *     acc = c_0 * A[p + o_0];  acc = acc + c_k * A[p + o_k]  (k = 1 .. n-1)
 * over the interior [R, N_d-1-R] of every dimension, R = max |o_k,d| (the cells within R of
 * an edge are Dirichlet, never written); the same ping-pong time loop as oracle_run (Fig. 1,
 * PAPER.md:142-148).  offs: n*dims int32 (slow -> fast), coefs: n doubles rounded once to T.
 * ---------------------------------------------------------------------------------- */
#define ORACLE_LINEAR(T)                                                               \
  int oracle_linear_##T(int dims, const int64_t *ext, int n, const int *offs,          \
                        const double *coefs, int64_t steps, const T *in, T *out,       \
                        int nthreads) {                                                \
    if ((dims != 2 && dims != 3) || n < 1 || n > 125 || steps < 0) return 1;           \
    int64_t N[3] = {ext[0], ext[1], dims == 3 ? ext[2] : 1};                           \
    int64_t st[3] = {dims == 3 ? N[1] * N[2] : N[1], dims == 3 ? N[2] : 1, 1};         \
    int R = 0;                                                                         \
    int64_t delta[125];                                                                \
    T c[125];                                                                          \
    for (int k = 0; k < n; ++k) {                                                      \
      delta[k] = 0;                                                                    \
      for (int d = 0; d < dims; ++d) {                                                 \
        int o = offs[k * dims + d];                                                    \
        if (o > R) R = o;                                                              \
        if (-o > R) R = -o;                                                            \
        delta[k] += (int64_t)o * st[d];                                                \
      }                                                                                \
      c[k] = (T)coefs[k];                                                              \
    }                                                                                  \
    if (dims == 2) N[2] = 1 + 2 * (int64_t)R; /* the loop below runs x in [R, N2-1-R] */ \
    int64_t n_el = N[0] * N[1] * (dims == 3 ? N[2] : 1);                               \
    T *buf[2];                                                                         \
    buf[0] = out;                                                                      \
    buf[1] = (T *)malloc((size_t)n_el * sizeof(T));                                    \
    if (!buf[1]) return 2;                                                             \
    memmove(buf[0], in, (size_t)n_el * sizeof(T));                                     \
    memcpy(buf[1], in, (size_t)n_el * sizeof(T));                                      \
    if (nthreads < 1) nthreads = 1;                                                    \
    for (int64_t t = 0; t < steps; ++t) {                                              \
      const T *src = buf[t % 2];                                                       \
      T *dst = buf[(t + 1) % 2];                                                       \
      _Pragma("omp parallel for schedule(static) num_threads(nthreads)")               \
      for (int64_t a = R; a < N[0] - R; ++a)                                           \
        for (int64_t b = R; b < N[1] - R; ++b)                                         \
          for (int64_t x = R; x < N[2] - R; ++x) {                                     \
            int64_t p = dims == 3 ? a * st[0] + b * st[1] + x : a * st[0] + b;         \
            T acc = c[0] * src[p + delta[0]];                                          \
            for (int k = 1; k < n; ++k) acc = acc + c[k] * src[p + delta[k]];          \
            dst[p] = acc;                                                              \
          }                                                                            \
    }                                                                                  \
    if (steps % 2 == 1) memcpy(out, buf[1], (size_t)n_el * sizeof(T));                 \
    free(buf[1]);                                                                      \
    return 0;                                                                          \
  }

ORACLE_LINEAR(float)
ORACLE_LINEAR(double)

/* Threads the OpenMP runtime would use (reported as `cores` by bench.py). */
int oracle_max_threads(void) {
#ifdef _OPENMP
  return omp_get_max_threads();
#else
  return 1;
#endif
}
