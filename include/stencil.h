/*
 * stencil.h -- C ABI of the B200-native hybrid hexagonal/classical tiled stencil library
 * (libhexstencil.so).  Implements the data-parallel hot path of Grosser, Cohen,
 * Holewinski, Sadayappan, Verdoolaege, "Hybrid Hexagonal/Classical Tiling for GPUs",
 * CGO'14: T time steps of an iterative affine stencil under
 * the hybrid schedule of Sec. 3.6.
 *
 * Conventions for every entry point
 *   - Returns stencil_status; nothing throws across the boundary.  On failure a
 *     thread-local message is available from stencil_last_error().
 *   - Arguments are plain pointers and sizes; no torch or CUDA types appear.  A "device
 *     pointer" is a CUDA global-memory address on the current device; a "stream" is a
 *     cudaStream_t passed as void* (NULL = legacy default stream).
 *   - Grids are dense, row-major, last dimension contiguous ("stride one",
 *     PAPER.md:636-641), extents listed slow -> fast and INCLUDING the boundary cells.
 *     Cells within the radius of an edge are Dirichlet: never written.
 *   - Ownership: the caller owns every device buffer (inputs, outputs and the plan's
 *     workspace, allocated e.g. with PyTorch).  The library never allocates, frees or
 *     retains device memory.  Descriptors and plans are library-owned host objects until
 *     stencil_destroy, immutable after creation; a plan may run on one stream at a time.
 *   - Errors: argument and feasibility errors are reported synchronously.  Kernel faults
 *     are asynchronous (sticky CUDA errors) and surface as STENCIL_E_CUDA on a later
 *     call.  There is no CPU fallback: without a CUDA device stencil_run fails with
 *     STENCIL_E_CUDA.
 */
#ifndef HEXSTENCIL_STENCIL_H
#define HEXSTENCIL_STENCIL_H

#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

#define STENCIL_ABI_VERSION 1

typedef enum {
  STENCIL_OK = 0,
  STENCIL_E_INVALID = 1,          /* bad argument, NULL handle, size/T mismatch */
  STENCIL_E_UNSUPPORTED = 2,      /* valid request outside what the library implements */
  STENCIL_E_INFEASIBLE_TILE = 3,  /* tile parameters violate eq. (1) or the kernel's limits */
  STENCIL_E_OOM = 4,              /* host allocation failed / workspace too small */
  STENCIL_E_CUDA = 5,             /* CUDA runtime error (incl. no device) */
  STENCIL_E_NCCL = 6              /* NCCL unavailable or failed (multi-GPU slab mode) */
} stencil_status;

typedef enum { STENCIL_F32 = 0, STENCIL_F64 = 1 } stencil_dtype;

/* Stencil classes (Table 3; per-point expressions in DESIGN.md). */
typedef enum {
  STENCIL_JACOBI2D5 = 0,   /* Fig. 1: k*((((c+s)+n)+e)+w), k = coef[0] (0.2)              */
  STENCIL_STAR2D5 = 1,     /* laplacian/heat 5-pt: c0*c + c1*(((n+s)+w)+e)  (0.5, 0.125)  */
  STENCIL_BOX2D9 = 2,      /* heat 2D 9-pt: k * row-major sum of the 3x3 box (1/9)        */
  STENCIL_FDTD2D = 3,      /* three in-place statements ey, ex, hz (0.5, 0.7); 3 fields   */
  STENCIL_STAR3D7 = 4,     /* laplacian/heat 3D 7-pt: c0*c + c1*(((((n+s)+w)+e)+u)+d)     */
  STENCIL_GRADIENT3D = 5,  /* c + 1/sqrt(eps + sum_6 (c-nb)^2)   (eps = 1e-2)             */
  STENCIL_BOX3D27 = 6,     /* heat 3D 27-pt: k * lexicographic sum of the 3x3x3 box (1/27)*/
  STENCIL_GRADIENT2D = 7,  /* c + 1/sqrt(eps + sum_4 (c-nb)^2)   (eps = 1e-2)             */
  STENCIL_LINEAR = 8       /* general linear stencil, 2D or 3D, any access set and radius:
                              c_0*A[p+o_0] + c_1*A[p+o_1] + ... (left to right); offsets and
                              coefficients required (n <= 64); radius = max |o| */
} stencil_kind;

typedef struct stencil_desc_s *stencil_desc_t;
typedef struct stencil_plan_s *stencil_plan_t;

/* Tile parameters of the hybrid schedule (Sec. 3.6: "parameterized with the values
 * h, w0, ..., wn").  A hexagonal tile spans 2h+2 (canonical) time
 * levels; w0 is the minimal hexagon width and must satisfy eq. (1);
 * w[i] is the classical tile width of the (i+1)-th non-hexagonal dimension.  All-zero
 * h, w0, w = choose defaults.  hex_dim selects the hexagonally tiled spatial dimension
 * (Sec. 3.6; must not be the innermost one). */
typedef struct {
  int32_t h;
  int32_t w0;
  int32_t w[3];
  int32_t hex_dim;  /* < 0: automatic (y for the streaming 3D star kernel, else dimension 0) */
  int32_t flags; /* STENCIL_EXEC_* */
} stencil_tile_t;

enum {
  STENCIL_EXEC_AUTO = 0,    /* fastest implemented hybrid-tiled kernel for the class      */
  STENCIL_EXEC_GENERIC = 1, /* generic hybrid kernel straight from global memory
                               (Table 4 configuration (a))                 */
  STENCIL_EXEC_NAIVE = 2,   /* non-time-tiled comparator: one launch per time step       */
  /* B200 replay of the optimisation ablation of Sec. 6.2 (Table 4): one 3D
   * hybrid phase kernel (kernels/ablation.cu) with the paper's CTA of 1 x 10 x 32 threads and
   * classical tiles w1 = 10, w2 = 32 (tile.w must be 0 or {10, 32}), hexagons over dimension 0,
   * differing only in the memory strategy.  3D radius-1 single-field classes (star3d7, box3d27,
   * gradient3d), STENCIL_F32 only (the paper's precision); anything else STENCIL_E_UNSUPPORTED. */
  STENCIL_EXEC_T4A = 3, /* (a) no shared memory: operands and results in global memory       */
  STENCIL_EXEC_T4B = 4, /* (b) copy-in box -> compute in shared memory -> copy-out phase      */
  STENCIL_EXEC_T4C = 5, /* (c) (b) with interleaved copy-out (store as computed)              */
  STENCIL_EXEC_T4D = 6, /* (d) (c) with tiles translated so the copy-in box is 128-B aligned  */
  STENCIL_EXEC_T4E = 7, /* (e) (d) + static reuse: fixed smem home per value (x mod 64)        */
  STENCIL_EXEC_T4F = 8  /* (f) (d) + dynamic reuse: explicit copy phase between x tiles        */
};

/* Create a stencil descriptor.
 *   dims        2 or 3 (must match the class)
 *   extents     dims values, slow -> fast, each >= 3 (boundary included)
 *   kind        stencil class
 *   radius      1 for the fixed classes; STENCIL_LINEAR: max |offset| over its access set
 *   offsets     optional (may be NULL): n_offsets*dims int32 offsets; if given they must
 *               equal the class's access set (validated, order free).  STENCIL_LINEAR:
 *               required, 1..64 offsets, evaluated in the given order
 *   coefficients optional (NULL = class defaults): n_coefficients doubles, rounded once
 *               to the working precision (see stencil_kind for the count and meaning);
 *               STENCIL_LINEAR: required, one per offset
 *   dtype       STENCIL_F32 or STENCIL_F64 (the arithmetic precision)
 * Host only; does not touch the GPU. */
stencil_status stencil_desc_create(stencil_desc_t *out, int dims, const int64_t *extents,
                                   stencil_kind kind, int radius, const int32_t *offsets,
                                   int n_offsets, const double *coefficients,
                                   int n_coefficients, stencil_dtype dtype);

/* Dependence analysis (Sec. 3.2-3.3.2): the memory-based dependence
 * distance vectors of the canonical schedule [k*t+i, s] (RAW, WAR, WAW of the ping-pong
 * or in-place layout), written as (dtau, ds_0..ds_{dims-1}) int32 rows into `dist`
 * (capacity `cap` rows); *n receives the count.  Host only. */
stencil_status stencil_desc_deps(stencil_desc_t desc, int32_t *dist, int cap, int *n);

/* Build an execution plan for T_steps time steps (a2 tile validation, a3 launch table).
 * tile may be NULL (= defaults).  Host only. */
stencil_status stencil_plan(stencil_plan_t *out, stencil_desc_t desc, int64_t T_steps,
                            const stencil_tile_t *tile);

/* Bytes of device workspace the plan needs (the second ping-pong buffer; 0 for the
 * in-place FDTD class).  The caller allocates it and hands it over with
 * stencil_plan_set_workspace before stencil_run.  dev_ptr must be 256-B aligned. */
stencil_status stencil_plan_workspace_size(stencil_plan_t plan, size_t *bytes);
stencil_status stencil_plan_set_workspace(stencil_plan_t plan, void *dev_ptr, size_t bytes);

/* Run the plan: out = T_steps steps applied to in.
 *   in, out   arrays of n_fields device pointers (1, or 3 for FDTD in the order
 *             ex, ey, hz), each the full grid, 16-B aligned.  in may alias out
 *             (in-place); in is never written otherwise.
 *   T_steps   must equal the plan's (STENCIL_E_INVALID otherwise); 0 copies in to out.
 *   stream    cudaStream_t as void*; all work is enqueued on it (asynchronous).
 * Per launch-table entry (T, p) one phase kernel is launched (host loop over T and the
 * two phases).  From the second call with the same in/out/workspace
 * pointers (and no profiling requested) the plan replays a CUDA graph of the whole launch
 * sequence, captured once on a private stream and launched on `stream` (same results,
 * less launch overhead; environment HEXS_NO_GRAPH=1 keeps every run eager).  The graphs
 * are released with the plan. */
stencil_status stencil_run(stencil_plan_t plan, const void *const *in, void *const *out,
                           int64_t T_steps, void *stream);

/* ---------------------------------------------------------------------------------
 * Multi-GPU slab mode.  One process per GPU; one non-innermost grid
 * dimension part_dim is split evenly over the ranks (part_dim < 0: the default -- 1 (y, a
 * classically tiled dimension of the 3D kernels, the north star's "slab-decomposes the
 * classically tiled spatial dimension") for 3D grids, 0 for 2D grids).  Rank q owns indices
 * [own_lo, own_hi) of part_dim and stores the local slab [loc_lo, loc_hi) = its owned indices
 * plus G = radius * (2h+2) ghost indices on every side that is not a global boundary ("halos of
 * width radius x time-tile depth"); every other dimension is whole.  Every rank runs the GLOBAL
 * run's launch table of the hybrid schedule (Sec. 3.6; when part_dim is the
 * hexagonal dimension the hexagon tiling is translated to the slab) over its slab, and before
 * every launch but the first the library refreshes the ghost indices of both ping-pong buffers
 * from rank +-1 by ncclSend / ncclRecv (one NCCL group) on an internal stream ordered against
 * the caller's stream by events; for part_dim > 0 the halos are strided in memory and are packed
 * / unpacked through a staging area at the end of the plan's workspace.  The slab's outermost
 * indices stay fixed; a launch spans at most 2h+2 levels, so wrong values never travel past the
 * ghosts and every owned point is exact after every launch; the ghosts are the only redundant
 * work, and the schedule is continuous (no time-block cuts).
 * NCCL is loaded at run time (the libnccl.so.2 the process already maps, e.g. PyTorch's;
 * environment HEXS_NCCL_LIB overrides); single-GPU use never needs it.  FDTD-2D is not
 * supported (STENCIL_E_UNSUPPORTED).
 * ------------------------------------------------------------------------------- */
typedef struct {
  int32_t rank, nranks, part_dim;
  int64_t global_ext[3];  /* the global extents                                              */
  int64_t local_ext[3];   /* extents of this rank's local slab (ghosts included)             */
  int64_t own_lo, own_hi; /* owned global indices of part_dim                                */
  int64_t loc_lo, loc_hi; /* global indices of part_dim held by the local slab               */
  int64_t ghost;          /* G = radius * time_block                                         */
  int64_t time_block;     /* 2h+2: levels a launch spans (the halo's time-tile depth)         */
  int64_t n_blocks;       /* stencil_dist_info: launches per run (an exchange before each but
                             the first); stencil_dist_layout: 0                               */
  int32_t h;              /* hexagon half-height the time block is a multiple of             */
  double ghost_fraction;  /* (local - owned) / owned indices: the redundant work             */
  int64_t launches_per_run; /* phase-kernel launches of one stencil_run (stencil_dist_info) */
  int32_t exchange;       /* stencil_dist_info: STENCIL_EXCHANGE_* the halos travel by          */
} stencil_dist_info_t;

enum {
  STENCIL_EXCHANGE_NONE = 0,   /* one rank, or an emulated rank without halo traffic                */
  STENCIL_EXCHANGE_NCCL = 1,   /* ncclSend / ncclRecv of packed halos on an internal stream         */
  STENCIL_EXCHANGE_P2P = 2,    /* device-initiated: a send kernel stores the halo lines into the
                                  neighbours' receive areas (NCCL symmetric window, LSA pointers)
                                  and publishes a sequence number; a wait kernel acquires theirs   */
  STENCIL_EXCHANGE_FUSED = 3   /* as P2P, but the 3D tile-wavefront phase kernel itself stores its
                                  send-zone lines into the neighbours' mirrors while it computes
                                  (y slabs of >= 2G lines; opt-in, environment HEXS_DIST_FUSED=1):
                                  the transfer overlaps the launch                                 */
};

/* Rank 0: a fresh NCCL unique id (128 bytes) for stencil_plan_dist; broadcast it to the other
 * ranks (e.g. with torch.distributed).  STENCIL_E_NCCL if NCCL cannot be loaded. */
stencil_status stencil_dist_unique_id(void *id_out);

/* Host-only layout of one rank (partition, ghost width, time block) -- exactly what
 * stencil_plan_dist uses; needs neither a GPU nor NCCL. */
stencil_status stencil_dist_layout(stencil_desc_t global_desc, int64_t T_steps, const stencil_tile_t *tile,
                                   int rank, int nranks, int part_dim, stencil_dist_info_t *info);

/* Collective over the nranks processes (each on its own current device): build this rank's
 * distributed plan for T_steps steps of the GLOBAL problem global_desc.  tile as for
 * stencil_plan (its h sets the time block; NULL = defaults).  nccl_unique_id: the 128 bytes
 * from stencil_dist_unique_id on rank 0.  part_dim: see above (< 0 = default).  The plan is then used like a
 * single-GPU plan: stencil_plan_workspace_size / set_workspace (shared by the block plans),
 * stencil_run(plan, in, out, T_steps, stream) with in / out the LOCAL slabs (local_ext,
 * 16-B aligned, in may alias out; every point of `in`, ghosts included, holds level 0 of the
 * global grid) -- on return the owned points of `out` hold level T_steps (ghosts are
 * scratch).  stencil_run on a distributed plan is collective (every rank calls it).
 * STENCIL_E_NCCL on communicator or transfer failure. */
stencil_status stencil_plan_dist(stencil_plan_t *out, stencil_desc_t global_desc, int64_t T_steps,
                                 const stencil_tile_t *tile, const void *nccl_unique_id, int rank,
                                 int nranks, int part_dim);

/* Host-only: rank `rank`'s local plan -- the plan stencil_plan_dist runs on the slab (extent
 * loc_hi - loc_lo along part_dim, the global hexagon tiling kept) -- as an ordinary plan
 * (introspection: launch table, schedule_of; or a single-GPU run of one rank's slab without
 * halo exchanges).  Destroy it with stencil_destroy. */
stencil_status stencil_dist_local_plan(stencil_plan_t *out, stencil_desc_t global_desc, int64_t T_steps,
                                       const stencil_tile_t *tile, int rank, int nranks, int part_dim);

/* Host-only: the outer rows (hexagonal coordinate z) whose halo lines of ping-pong buffer
 * `buffer` travel in the exchange before launch k >= 1 of a local plan (stencil_dist_local_plan)
 * of a slab partitioned along part_dim > 0 with the hexagonal dimension 0 whole: z holds level
 * L(z) in buffer L(z) % 2 and L(z) - 1 in the other, and the launch reads the older one only where
 * a z-neighbour is behind.  Writes up to cap rows, *n = their number; *n = -1 if the rule does
 * not apply (every row travels). */
stencil_status stencil_dist_halo_rows(stencil_plan_t local_plan, int part_dim, int64_t k, int buffer,
                                      int32_t *rows, int64_t cap, int64_t *n);

/* The layout of a distributed plan and its launches per run. */
stencil_status stencil_dist_info(stencil_plan_t plan, stencil_dist_info_t *info);

/* A borrowed handle to the local plan of a distributed plan (index 0) -- for introspection and
 * kernel-region profiling (stencil_plan_profile).  Owned by the distributed plan: never pass it
 * to stencil_destroy. */
stencil_status stencil_dist_block_plan(stencil_plan_t plan, int index, stencil_plan_t *block);

/* Destroy a descriptor or plan (tagged handles).  NULL is a no-op.  A plan keeps its own
 * copy of the descriptor, so destruction order is free. */
stencil_status stencil_destroy(void *handle);

/* Thread-local message of the last failing call on this thread ("" if none). */
const char *stencil_last_error(void);

/* ---------------------------------------------------------------------------------
 * Introspection (host only): used by tests to check the planner against the schedule
 * oracle and by the bench for the roofline model.
 * ------------------------------------------------------------------------------- */
typedef struct {
  int32_t dims, kind, dtype, n_fields, statements; /* statements k of tau = k*t + i */
  int32_t hex_dim;
  int32_t delta0_num, delta0_den, delta1_num, delta1_den; /* cone slopes along hex_dim */
  int32_t delta_cls[3];  /* classical skews delta1_i for the other dims (slow -> fast) */
  int32_t trans_cls[3];  /* classical tile translation offsets (Sec. 4.2.3) */
  int32_t h, w0, w[3];   /* effective tile parameters */
  int32_t H, W;          /* box height 2h+2 and width 2w0+2+floor(d0 h)+floor(d1 h) */
  int32_t F0, F1;        /* floor(delta0 h), floor(delta1 h) */
  int32_t executor;      /* STENCIL_EXEC_* actually used */
  int32_t fast_kernel;   /* 1 if a specialised register-wavefront kernel runs */
  int64_t n_launches;    /* launch-table entries (kernel launches per run) */
  int64_t T_steps, tau_levels;
  int64_t updates;       /* interior points x T_steps (FDTD: point-steps) */
  int64_t tile_points;   /* instances of one full hexagon per classical column */
  int64_t tile_in, tile_out; /* In / Out values of one full hexagon per column */
  size_t workspace_bytes;
  int32_t kernel;        /* STENCIL_KERNEL_*: the phase-kernel family that runs */
} stencil_plan_info_t;

enum {
  STENCIL_KERNEL_GENERIC = 0,   /* kernels/generic.cu: Sec. 4.1 mapping from global memory   */
  STENCIL_KERNEL_NAIVE = 1,     /* one launch per time step (comparator)                      */
  STENCIL_KERNEL_FAST2D = 2,    /* 2D register wavefront, TMA-staged In rows                  */
  STENCIL_KERNEL_FDTD = 3,      /* FDTD-2D shared-memory ring                                 */
  STENCIL_KERNEL_FAST3D = 4,    /* 3D tile wavefront, hexagons over (t, z), levels in smem    */
  STENCIL_KERNEL_STREAM3D = 5,  /* 3D streaming: hexagons over (t, y), z streamed, registers  */
  STENCIL_KERNEL_ABLATION = 6   /* Table 4 replay (STENCIL_EXEC_T4A..T4F)                      */
};

stencil_status stencil_plan_info(stencil_plan_t plan, stencil_plan_info_t *info);

/* One launch-table entry (a3): the hexagons S0 in [S0_lo, S0_hi] of time tile T and
 * phase p run in parallel; each covers canonical levels tau = tau0 + a for
 * a in [a_lo, a_hi]; its local row b is spatial coordinate s0 = S0*W + b - row_off. */
typedef struct {
  int64_t T;
  int32_t phase;
  int32_t a_lo, a_hi;
  int64_t tau0;
  int64_t S0_lo, S0_hi;
  int64_t row_off;
} stencil_launch_t;

stencil_status stencil_plan_launches(stencil_plan_t plan, stencil_launch_t *out, int64_t cap,
                                     int64_t *n);

/* Hexagon row bounds: for a in [0, 2h+1], rows b in [lo[a], hi[a]] (constraints
 * (6)-(13)).  cap >= 2h+2. */
stencil_status stencil_plan_hexagon(stencil_plan_t plan, int32_t *lo, int32_t *hi, int32_t cap);

/* Schedule of one instance (canonical time tau, spatial point s[dims]) as the tuple
 * [T, p, S0, S_1..S_n, t', s'_0, s'_1..s'_n] of Sec. 3.6 (eq. (14) with the plan's classical skews
 * and translation offsets; n = dims-1 classical dims in
 * slow -> fast order excluding hex_dim), written to sched (capacity 2*dims+3). */
stencil_status stencil_plan_schedule_of(stencil_plan_t plan, int64_t tau, const int64_t *s,
                                        int64_t *sched);

/* Device timing of the phase kernels (used by bench.py for the roofline's kernel time).
 * stencil_plan_profile(plan, max_runs) makes the next max_runs stencil_run calls run eagerly
 * and record one CUDA event on the run's stream right before its first phase-kernel launch
 * and one right after its last (the kernel region: every launch of the launch table, back to
 * back, without the run's boundary copies); 0 disables and frees the events.
 * stencil_plan_profile_read synchronises on the recorded events and returns the summed
 * kernel-region time (ms) over the recorded runs, the number of phase-kernel launches they
 * contain and the longest single run's kernel region (ms), then resets the recorder. */
stencil_status stencil_plan_profile(stencil_plan_t plan, int max_runs);
stencil_status stencil_plan_profile_read(stencil_plan_t plan, double *kernel_ms, int64_t *launches,
                                         double *max_launch_ms);

/* The tile-size model (a2; Sec. 3.7): for a hexagon (h, w0) along hex_dim,
 * the exact per-column points / In / Out of the full hexagon, the load-to-compute ratio as HBM
 * bytes per update, and the two B200 terms -- the unrolled body against the instruction cache
 * (family 1 = 2D register-wavefront kernel, 2 = 3D tile-wavefront kernel, 0 = generic kernel:
 * no code term) and the CTA-count (wave) efficiency -- with the predicted relative rate.
 * `selected` = 1 if the planner's automatic choice for this family is this tile.  Host only. */
typedef struct {
  int32_t h, w0;
  int64_t points, in, out;
  double bytes_per_update, body_bytes, code_eff;
  int64_t ctas, slots;
  double wave_eff, rate;
  int32_t selected;
} stencil_tile_eval_t;
stencil_status stencil_tile_model(stencil_desc_t desc, int h, int w0, int hex_dim, int family,
                                  stencil_tile_eval_t *out);

int stencil_abi_version(void);

#ifdef __cplusplus
}
#endif
#endif /* HEXSTENCIL_STENCIL_H */
