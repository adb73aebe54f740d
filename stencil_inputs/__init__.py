"""Seeded synthetic inputs shared by the oracle-side tests and the product-side bench.

Holds none of the method's arithmetic: only a counter-based generator that maps
(seed, linear index) to a value, so that the oracle and the CUDA path can be fed the
identical bits.

Recipe: v = (splitmix64(idx XOR (seed * K)) >> 40) * 2**-24, K = 0x632BE59BD9B4E019.
Values are uniform on [0, 1) with 24 significant bits, so they are exact in fp32 and
fp64 alike.  Dense regular grids (Table 3 of the paper), row-major,
last dimension contiguous; the boundary cells carry the same distribution and are the
Dirichlet values.
"""
from __future__ import annotations

from typing import Sequence

import numpy as np

_K = np.uint64(0x632BE59BD9B4E019)
_G = np.uint64(0x9E3779B97F4A7C15)
_M1 = np.uint64(0xBF58476D1CE4E5B9)
_M2 = np.uint64(0x94D049BB133111EB)


def _splitmix64(x: np.ndarray) -> np.ndarray:
    z = x + _G
    z = (z ^ (z >> np.uint64(30))) * _M1
    z = (z ^ (z >> np.uint64(27))) * _M2
    return z ^ (z >> np.uint64(31))


def uniform(shape: Sequence[int], seed: int, dtype=np.float32, out: np.ndarray = None,
            chunk: int = 1 << 24, offset: int = 0) -> np.ndarray:
    """Fill an array of `shape` with the counter-based uniform values of `seed`; element k
    of the (flattened) array is the value of linear index offset + k, so a slab of a
    larger grid can be generated on its own (multi-GPU ranks)."""
    shape = tuple(int(s) for s in shape)
    n = int(np.prod(shape))
    if out is None:
        out = np.empty(shape, dtype=dtype)
    flat = out.reshape(-1)
    key = np.uint64((int(seed) * int(_K)) & 0xFFFFFFFFFFFFFFFF)
    with np.errstate(over="ignore"):
        for lo in range(0, n, chunk):
            hi = min(n, lo + chunk)
            idx = np.arange(lo + offset, hi + offset, dtype=np.uint64)
            z = _splitmix64(idx ^ key)
            flat[lo:hi] = (z >> np.uint64(40)).astype(np.float64) * (2.0 ** -24)
    return out


def fields(shape: Sequence[int], seed: int, n: int, dtype=np.float32):
    """n independent fields (e.g. FDTD's ex, ey, hz) from seeds seed, seed+1, ..."""
    return [uniform(shape, seed + k, dtype) for k in range(n)]


def uniform_box(global_shape: Sequence[int], lo: Sequence[int], hi: Sequence[int], seed: int,
                dtype=np.float32) -> np.ndarray:
    """The sub-box [lo, hi) of the grid `uniform(global_shape, seed)` -- generated on its own (a
    rank's slab of a partition along any dimension), bit-identical to slicing the full grid."""
    gs = [int(s) for s in global_shape]
    lo = [int(v) for v in lo]
    hi = [int(v) for v in hi]
    strides = [int(np.prod(gs[q + 1:])) for q in range(len(gs))]
    out = np.empty([b - a for a, b in zip(lo, hi)], dtype=dtype)
    key = np.uint64((int(seed) * int(_K)) & 0xFFFFFFFFFFFFFFFF)
    # linear indices of one outermost slice of the box (broadcast over the inner dimensions)
    inner = np.zeros([1] + [b - a for a, b in zip(lo[1:], hi[1:])], dtype=np.uint64)
    for q in range(1, len(gs)):
        shp = [1] * len(gs)
        shp[q] = hi[q] - lo[q]
        inner = inner + (np.arange(lo[q], hi[q], dtype=np.uint64) * np.uint64(strides[q])).reshape(shp)
    with np.errstate(over="ignore"):
        for k, z in enumerate(range(lo[0], hi[0])):
            idx = inner[0] + np.uint64(z * strides[0])
            v = _splitmix64(idx ^ key)
            out[k] = (v >> np.uint64(40)).astype(np.float64) * (2.0 ** -24)
    return out
