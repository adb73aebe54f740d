"""CPU oracle for the hybrid hexagonal/classical tiled stencil hot path.

TEST INFRASTRUCTURE ONLY.  Only tests/, __graft_entry__.smoke() and bench.py's
cpu_baseline / `--impl reference` legs may import this package.  The product package
(paper_conf_cgo_grosserchsv14_b200) never imports it and shares no code with it.

`oracle.c` is the naive time loop of Fig. 1 for every stencil class;
`schedule.py` is Sec. 3's schedule in exact arithmetic.  See the header of oracle.c for
the per-point expressions and DESIGN.md for the readings of the paper they follow.
"""
from __future__ import annotations

import ctypes
import os
from typing import Optional, Sequence, Tuple

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.path.join(_HERE, "liboracle.so")

# Oracle-local class numbering (mirrors the enum in oracle.c).
KINDS = {
    "jacobi2d5": 0, "star2d5": 1, "box2d9": 2, "fdtd2d": 3,
    "star3d7": 4, "gradient3d": 5, "box3d27": 6, "gradient2d": 7,
}
DIMS = {"jacobi2d5": 2, "star2d5": 2, "box2d9": 2, "fdtd2d": 2, "gradient2d": 2,
        "star3d7": 3, "gradient3d": 3, "box3d27": 3}

# Default coefficients (readings R7/R8/R9): Fig. 1's 0.2f for Jacobi; explicit
# heat with alpha = 1/8 for the 5-/7-point stars; 1/9 and 1/27 box means; eps = 1e-2 for
# gradient; PolyBench 0.5 / 0.7 for FDTD.
DEFAULT_COEF = {
    "jacobi2d5": (0.2,), "star2d5": (0.5, 0.125), "box2d9": (1.0 / 9.0,),
    "fdtd2d": (0.5, 0.7), "star3d7": (0.25, 0.125), "gradient3d": (1e-2,),
    "box3d27": (1.0 / 27.0,), "gradient2d": (1e-2,),
}

_lib: Optional[ctypes.CDLL] = None


def build(force: bool = False) -> str:
    """Compile oracle.c with gcc (-O3 -ffp-contract=off -fopenmp, no fast-math)."""
    import subprocess

    src = os.path.join(_HERE, "oracle.c")
    if not force and os.path.exists(LIB_PATH) and os.path.getmtime(LIB_PATH) >= os.path.getmtime(src):
        return LIB_PATH
    cmd = ["gcc", "-O3", "-std=c11", "-ffp-contract=off", "-fno-fast-math", "-fopenmp",
           "-fPIC", "-shared", "-o", LIB_PATH, src, "-lm"]
    subprocess.check_call(cmd)
    return LIB_PATH


def lib() -> ctypes.CDLL:
    global _lib
    if _lib is None:
        build()
        L = ctypes.CDLL(LIB_PATH)
        i64p = ctypes.POINTER(ctypes.c_int64)
        dp = ctypes.POINTER(ctypes.c_double)
        for T in ("float", "double"):
            f = getattr(L, f"oracle_run_{T}")
            f.argtypes = [ctypes.c_int, ctypes.c_int, i64p, dp, ctypes.c_int, ctypes.c_int64,
                          ctypes.c_void_p, ctypes.c_void_p, ctypes.c_int]
            f.restype = ctypes.c_int
            g = getattr(L, f"oracle_fdtd_{T}")
            g.argtypes = [i64p, dp, ctypes.c_int, ctypes.c_int64, ctypes.c_void_p,
                          ctypes.c_void_p, ctypes.c_void_p, ctypes.c_int]
            g.restype = ctypes.c_int
            p = getattr(L, f"oracle_points_{T}")
            p.argtypes = [ctypes.c_int, ctypes.c_int, i64p, dp, ctypes.c_int, ctypes.c_int64,
                          ctypes.c_void_p, ctypes.c_int, i64p, ctypes.c_void_p]
            p.restype = ctypes.c_int
            li = getattr(L, f"oracle_linear_{T}")
            li.argtypes = [ctypes.c_int, i64p, ctypes.c_int, ctypes.POINTER(ctypes.c_int), dp, ctypes.c_int64,
                           ctypes.c_void_p, ctypes.c_void_p, ctypes.c_int]
            li.restype = ctypes.c_int
        L.oracle_max_threads.restype = ctypes.c_int
        _lib = L
    return _lib


def _ctype(dtype) -> str:
    if dtype == np.float32:
        return "float"
    if dtype == np.float64:
        return "double"
    raise TypeError(f"unsupported dtype {dtype}")


def _i64(a: Sequence[int]):
    arr = (ctypes.c_int64 * len(a))(*[int(x) for x in a])
    return arr


def _dbl(a: Sequence[float]):
    return (ctypes.c_double * len(a))(*[float(x) for x in a])


def max_threads() -> int:
    return int(lib().oracle_max_threads())


def run(kind: str, grid: np.ndarray, steps: int, coef: Optional[Sequence[float]] = None,
        nthreads: int = 1) -> np.ndarray:
    """Naive time loop (Fig. 1) of a single-field class; returns level `steps`."""
    assert kind != "fdtd2d"
    a = np.ascontiguousarray(grid)
    coef = DEFAULT_COEF[kind] if coef is None else coef
    out = np.empty_like(a)
    f = getattr(lib(), f"oracle_run_{_ctype(a.dtype)}")
    rc = f(KINDS[kind], a.ndim, _i64(a.shape), _dbl(coef), len(coef), int(steps),
           a.ctypes.data, out.ctypes.data, int(nthreads))
    if rc != 0:
        raise ValueError(f"oracle_run failed rc={rc}")
    return out


def fdtd(ex: np.ndarray, ey: np.ndarray, hz: np.ndarray, steps: int,
         coef: Optional[Sequence[float]] = None, nthreads: int = 1) -> Tuple[np.ndarray, ...]:
    """FDTD-2D (three in-place statements per step); returns (ex, ey, hz) at step `steps`."""
    coef = DEFAULT_COEF["fdtd2d"] if coef is None else coef
    ex, ey, hz = (np.array(x, copy=True, order="C") for x in (ex, ey, hz))
    assert ex.dtype == ey.dtype == hz.dtype and ex.shape == ey.shape == hz.shape
    f = getattr(lib(), f"oracle_fdtd_{_ctype(ex.dtype)}")
    rc = f(_i64(ex.shape), _dbl(coef), len(coef), int(steps), ex.ctypes.data, ey.ctypes.data,
           hz.ctypes.data, int(nthreads))
    if rc != 0:
        raise ValueError(f"oracle_fdtd failed rc={rc}")
    return ex, ey, hz


def points(kind: str, grid: np.ndarray, steps: int, coords: np.ndarray,
           coef: Optional[Sequence[float]] = None) -> np.ndarray:
    """Values at level `steps` of the given points via their dependence cones."""
    a = np.ascontiguousarray(grid)
    coef = DEFAULT_COEF[kind] if coef is None else coef
    c = np.ascontiguousarray(np.asarray(coords, dtype=np.int64).reshape(-1, a.ndim))
    vals = np.empty(c.shape[0], dtype=a.dtype)
    f = getattr(lib(), f"oracle_points_{_ctype(a.dtype)}")
    rc = f(KINDS[kind], a.ndim, _i64(a.shape), _dbl(coef), len(coef), int(steps), a.ctypes.data,
           int(c.shape[0]), c.ctypes.data_as(ctypes.POINTER(ctypes.c_int64)), vals.ctypes.data)
    if rc != 0:
        raise ValueError(f"oracle_points failed rc={rc}")
    return vals


def linear(grid: np.ndarray, offsets: Sequence[Sequence[int]], coefficients: Sequence[float], steps: int,
           nthreads: int = 1) -> np.ndarray:
    """General linear stencil (oracle.c `oracle_linear`): level `steps` of
    A'[p] = c_0 A[p+o_0] + ... + c_{n-1} A[p+o_{n-1}] (left to right) over the interior
    [R, N-1-R], R = max |offset|."""
    a = np.ascontiguousarray(grid)
    offs = np.ascontiguousarray(np.asarray(offsets, dtype=np.int32).reshape(-1, a.ndim))
    coefs = [float(c) for c in coefficients]
    assert offs.shape[0] == len(coefs)
    out = np.empty_like(a)
    f = getattr(lib(), f"oracle_linear_{_ctype(a.dtype)}")
    rc = f(a.ndim, _i64(a.shape), len(coefs), offs.ctypes.data_as(ctypes.POINTER(ctypes.c_int)), _dbl(coefs),
           int(steps), a.ctypes.data, out.ctypes.data, int(nthreads))
    if rc != 0:
        raise ValueError(f"oracle_linear failed rc={rc}")
    return out
