"""ctypes binding of include/stencil.h (argument marshalling only).

Every step of the hot path runs inside libhexstencil.so (C++ planner + sm_100a CUDA
kernels).  There is no Python or CPU fallback: if the library is missing, importing the
package raises, and without a CUDA device stencil_run fails with STENCIL_E_CUDA."""
from __future__ import annotations

import ctypes
import os

_HERE = os.path.dirname(os.path.abspath(__file__))
# HEXS_LIB selects an alternative build of the same library (e.g. the cycle-accounting
# build of tools/f3_timing.py); the default is the in-tree product build.
LIB_PATH = os.environ.get("HEXS_LIB") or os.path.join(_HERE, "lib", "libhexstencil.so")

STATUS = {0: "STENCIL_OK", 1: "STENCIL_E_INVALID", 2: "STENCIL_E_UNSUPPORTED",
          3: "STENCIL_E_INFEASIBLE_TILE", 4: "STENCIL_E_OOM", 5: "STENCIL_E_CUDA",
          6: "STENCIL_E_NCCL"}

KINDS = {"jacobi2d5": 0, "star2d5": 1, "box2d9": 2, "fdtd2d": 3, "star3d7": 4,
         "gradient3d": 5, "box3d27": 6, "gradient2d": 7, "linear": 8}
EXEC = {"auto": 0, "generic": 1, "naive": 2,  # + the Table 4 replay (a)-(f)
        "t4a": 3, "t4b": 4, "t4c": 5, "t4d": 6, "t4e": 7, "t4f": 8}

# every symbol include/stencil.h declares
SYMBOLS = ["stencil_desc_create", "stencil_desc_deps", "stencil_plan",
           "stencil_plan_workspace_size", "stencil_plan_set_workspace", "stencil_run",
           "stencil_destroy", "stencil_last_error", "stencil_plan_info",
           "stencil_plan_launches", "stencil_plan_hexagon", "stencil_plan_schedule_of",
           "stencil_plan_profile", "stencil_plan_profile_read", "stencil_abi_version",
           "stencil_dist_unique_id", "stencil_dist_layout", "stencil_plan_dist", "stencil_dist_info",
           "stencil_dist_block_plan", "stencil_tile_model", "stencil_dist_local_plan", "stencil_dist_halo_rows"]


class StencilError(RuntimeError):
    def __init__(self, status: int, message: str):
        super().__init__(f"{STATUS.get(status, status)}: {message}")
        self.status = status


class Tile(ctypes.Structure):
    _fields_ = [("h", ctypes.c_int32), ("w0", ctypes.c_int32), ("w", ctypes.c_int32 * 3),
                ("hex_dim", ctypes.c_int32), ("flags", ctypes.c_int32)]


class PlanInfo(ctypes.Structure):
    _fields_ = [("dims", ctypes.c_int32), ("kind", ctypes.c_int32), ("dtype", ctypes.c_int32),
                ("n_fields", ctypes.c_int32), ("statements", ctypes.c_int32),
                ("hex_dim", ctypes.c_int32),
                ("delta0_num", ctypes.c_int32), ("delta0_den", ctypes.c_int32),
                ("delta1_num", ctypes.c_int32), ("delta1_den", ctypes.c_int32),
                ("delta_cls", ctypes.c_int32 * 3), ("trans_cls", ctypes.c_int32 * 3), ("h", ctypes.c_int32), ("w0", ctypes.c_int32),
                ("w", ctypes.c_int32 * 3), ("H", ctypes.c_int32), ("W", ctypes.c_int32),
                ("F0", ctypes.c_int32), ("F1", ctypes.c_int32), ("executor", ctypes.c_int32),
                ("fast_kernel", ctypes.c_int32), ("n_launches", ctypes.c_int64),
                ("T_steps", ctypes.c_int64), ("tau_levels", ctypes.c_int64),
                ("updates", ctypes.c_int64), ("tile_points", ctypes.c_int64),
                ("tile_in", ctypes.c_int64), ("tile_out", ctypes.c_int64),
                ("workspace_bytes", ctypes.c_size_t), ("kernel", ctypes.c_int32)]

KERNELS = {0: "generic", 1: "naive", 2: "fast2d", 3: "fdtd", 4: "fast3d", 5: "stream3d", 6: "ablation"}


class DistInfo(ctypes.Structure):
    _fields_ = [("rank", ctypes.c_int32), ("nranks", ctypes.c_int32), ("part_dim", ctypes.c_int32),
                ("global_ext", ctypes.c_int64 * 3), ("local_ext", ctypes.c_int64 * 3),
                ("own_lo", ctypes.c_int64), ("own_hi", ctypes.c_int64), ("loc_lo", ctypes.c_int64),
                ("loc_hi", ctypes.c_int64), ("ghost", ctypes.c_int64), ("time_block", ctypes.c_int64),
                ("n_blocks", ctypes.c_int64), ("h", ctypes.c_int32), ("ghost_fraction", ctypes.c_double),
                ("launches_per_run", ctypes.c_int64), ("exchange", ctypes.c_int32)]

EXCHANGES = {0: "none", 1: "nccl", 2: "p2p", 3: "fused"}


class TileEval(ctypes.Structure):
    _fields_ = [("h", ctypes.c_int32), ("w0", ctypes.c_int32), ("points", ctypes.c_int64),
                ("in_", ctypes.c_int64), ("out", ctypes.c_int64), ("bytes_per_update", ctypes.c_double),
                ("body_bytes", ctypes.c_double), ("code_eff", ctypes.c_double), ("ctas", ctypes.c_int64),
                ("slots", ctypes.c_int64), ("wave_eff", ctypes.c_double), ("rate", ctypes.c_double),
                ("selected", ctypes.c_int32)]


class Launch(ctypes.Structure):
    _fields_ = [("T", ctypes.c_int64), ("phase", ctypes.c_int32), ("a_lo", ctypes.c_int32),
                ("a_hi", ctypes.c_int32), ("tau0", ctypes.c_int64), ("S0_lo", ctypes.c_int64),
                ("S0_hi", ctypes.c_int64), ("row_off", ctypes.c_int64)]


_lib = None


def lib() -> ctypes.CDLL:
    global _lib
    if _lib is not None:
        return _lib
    if not os.path.exists(LIB_PATH):
        raise ImportError(f"{LIB_PATH} is not built; run `python -c 'import __graft_entry__ as g; g.build()'`")
    L = ctypes.CDLL(LIB_PATH)
    vp, i32, i64, sz = ctypes.c_void_p, ctypes.c_int32, ctypes.c_int64, ctypes.c_size_t
    P = ctypes.POINTER
    L.stencil_desc_create.argtypes = [P(vp), ctypes.c_int, P(i64), ctypes.c_int, ctypes.c_int,
                                      P(i32), ctypes.c_int, P(ctypes.c_double), ctypes.c_int,
                                      ctypes.c_int]
    L.stencil_desc_deps.argtypes = [vp, P(i32), ctypes.c_int, P(ctypes.c_int)]
    L.stencil_plan.argtypes = [P(vp), vp, i64, P(Tile)]
    L.stencil_plan_workspace_size.argtypes = [vp, P(sz)]
    L.stencil_plan_set_workspace.argtypes = [vp, vp, sz]
    L.stencil_run.argtypes = [vp, P(vp), P(vp), i64, vp]
    L.stencil_destroy.argtypes = [vp]
    L.stencil_last_error.restype = ctypes.c_char_p
    L.stencil_plan_info.argtypes = [vp, P(PlanInfo)]
    L.stencil_plan_launches.argtypes = [vp, P(Launch), i64, P(i64)]
    L.stencil_plan_hexagon.argtypes = [vp, P(i32), P(i32), i32]
    L.stencil_plan_schedule_of.argtypes = [vp, i64, P(i64), P(i64)]
    L.stencil_plan_profile.argtypes = [vp, ctypes.c_int]
    L.stencil_plan_profile_read.argtypes = [vp, P(ctypes.c_double), P(i64), P(ctypes.c_double)]
    L.stencil_dist_unique_id.argtypes = [vp]
    L.stencil_dist_layout.argtypes = [vp, i64, P(Tile), ctypes.c_int, ctypes.c_int, ctypes.c_int, P(DistInfo)]
    L.stencil_plan_dist.argtypes = [P(vp), vp, i64, P(Tile), vp, ctypes.c_int, ctypes.c_int, ctypes.c_int]
    L.stencil_dist_info.argtypes = [vp, P(DistInfo)]
    L.stencil_dist_block_plan.argtypes = [vp, ctypes.c_int, P(vp)]
    L.stencil_dist_local_plan.argtypes = [P(vp), vp, i64, P(Tile), ctypes.c_int, ctypes.c_int, ctypes.c_int]
    L.stencil_tile_model.argtypes = [vp, ctypes.c_int, ctypes.c_int, ctypes.c_int, ctypes.c_int, P(TileEval)]
    L.stencil_dist_halo_rows.argtypes = [vp, ctypes.c_int, i64, ctypes.c_int, P(i32), i64, P(i64)]
    for name in SYMBOLS:
        f = getattr(L, name)
        if name not in ("stencil_last_error", "stencil_abi_version"):
            f.restype = ctypes.c_int
    L.stencil_abi_version.restype = ctypes.c_int
    _lib = L
    return L


def check(status: int) -> None:
    if status != 0:
        msg = lib().stencil_last_error().decode(errors="replace")
        raise StencilError(status, msg)
