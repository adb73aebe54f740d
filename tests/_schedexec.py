"""Test helper: executes a plan's launch table (the product planner's hybrid schedule, taken
from the C ABI's introspection) on numpy arrays, level-major within each launch -- valid because
the hexagons of one launch carry no dependence between them and every dependence inside a
hexagon points to a lower level (Sec. 3.3-3.6).  The per-point update is a numpy expression with
the oracle's association order for the stencil classes used here; CPU tests use it to check the
multi-GPU protocol (per-launch ghost exchange) without a GPU."""
import numpy as np


def star2d5_levels(src, dst, r0, r1, k0=np.float32(0.5), k1=np.float32(0.125)):
    c, n, s = src[r0:r1 + 1, 1:-1], src[r0 - 1:r1, 1:-1], src[r0 + 1:r1 + 2, 1:-1]
    w, e = src[r0:r1 + 1, :-2], src[r0:r1 + 1, 2:]
    dst[r0:r1 + 1, 1:-1] = k0 * c + k1 * (((n + s) + w) + e)


def star3d7_levels(src, dst, r0, r1, k0=np.float32(0.25), k1=np.float32(0.125)):
    c = src[r0:r1 + 1, 1:-1, 1:-1]
    u, d = src[r0 - 1:r1, 1:-1, 1:-1], src[r0 + 1:r1 + 2, 1:-1, 1:-1]
    n, s = src[r0:r1 + 1, :-2, 1:-1], src[r0:r1 + 1, 2:, 1:-1]
    w, e = src[r0:r1 + 1, 1:-1, :-2], src[r0:r1 + 1, 1:-1, 2:]
    dst[r0:r1 + 1, 1:-1, 1:-1] = k0 * c + k1 * (((((n + s) + w) + e) + u) + d)


UPDATE = {"star2d5": star2d5_levels, "star3d7": star3d7_levels}


def launch_executor(plan, kind):
    """execute(launch, bufs): one launch of `plan` (hexagons along dimension 0) on bufs[0/1]."""
    info = plan.info
    lo, hi = plan.hexagon()
    W = info["W"]
    upd = UPDATE[kind]

    def execute(ln, bufs):
        N0 = bufs[0].shape[0]
        for a in range(ln["a_lo"], ln["a_hi"] + 1):
            tau = ln["tau0"] + a
            src, dst = bufs[tau % 2], bufs[(tau + 1) % 2]
            for S0 in range(ln["S0_lo"], ln["S0_hi"] + 1):
                i0 = S0 * W - ln["row_off"]
                r0, r1 = max(i0 + lo[a], 1), min(i0 + hi[a], N0 - 2)
                if r0 <= r1:
                    upd(src, dst, r0, r1)

    return execute


def run_plan(plan, kind, grid, T):
    bufs = [grid.copy(), grid.copy()]
    ex = launch_executor(plan, kind)
    for ln in plan.launches():
        ex(ln, bufs)
    return bufs[T % 2]
