"""Python API over the C ABI (include/stencil.h).

PyTorch supplies device memory and streams only; planning and every time step run in
libhexstencil.so.

    st = Stencil("star2d5", (8192, 8192))            # stencil_desc_create
    plan = Plan(st, T_steps=512)                      # stencil_plan (+ workspace via torch)
    out = plan.run(grid)                              # stencil_run on the current stream
"""
from __future__ import annotations

import ctypes
from typing import Dict, List, Optional, Sequence, Tuple, Union

from . import _lib
from ._lib import EXEC, KINDS, Launch, PlanInfo, StencilError, Tile, check, lib

_DTYPES = {"float32": 0, "float64": 1}


def _dtype_code(dtype) -> int:
    name = str(dtype).replace("torch.", "").replace("<class 'numpy.", "").rstrip("'>")
    if name not in _DTYPES:
        raise StencilError(1, f"unsupported dtype {dtype}")
    return _DTYPES[name]


class Stencil:
    """A stencil descriptor: class, grid extents (slow -> fast, boundary included), dtype."""

    def __init__(self, kind: str, extents: Sequence[int], dtype="float32",
                 coefficients: Optional[Sequence[float]] = None,
                 offsets: Optional[Sequence[Sequence[int]]] = None):
        if kind not in KINDS:
            raise StencilError(1, f"unknown stencil kind {kind!r}")
        self.kind = kind
        self.extents = tuple(int(e) for e in extents)
        self.dims = len(self.extents)
        self.dtype_code = _dtype_code(dtype)
        ext = (ctypes.c_int64 * self.dims)(*self.extents)
        coef_p, ncoef = None, 0
        if coefficients is not None:
            coef_p = (ctypes.c_double * len(coefficients))(*[float(c) for c in coefficients])
            ncoef = len(coefficients)
        off_p, noff = None, 0
        if offsets is not None:
            flat = [int(v) for o in offsets for v in o]
            off_p = (ctypes.c_int32 * len(flat))(*flat)
            noff = len(offsets)
        radius = 1
        if kind == "linear":  # a general access set: its radius is the largest |offset|
            if offsets is None or coefficients is None:
                raise StencilError(1, "a linear stencil needs offsets and coefficients")
            radius = max(abs(int(v)) for o in offsets for v in o)
        self.radius = radius
        h = ctypes.c_void_p()
        check(lib().stencil_desc_create(ctypes.byref(h), self.dims, ext, KINDS[kind], radius, off_p,
                                        noff, coef_p, ncoef, self.dtype_code))
        self._h = h

    @property
    def n_fields(self) -> int:
        return 3 if self.kind == "fdtd2d" else 1

    def dependences(self) -> List[Tuple[int, ...]]:
        n = ctypes.c_int()
        check(lib().stencil_desc_deps(self._h, None, 0, ctypes.byref(n)))
        buf = (ctypes.c_int32 * (n.value * (self.dims + 1)))()
        check(lib().stencil_desc_deps(self._h, buf, n.value, ctypes.byref(n)))
        d = self.dims + 1
        return [tuple(buf[i * d:(i + 1) * d]) for i in range(n.value)]

    def __del__(self):
        h = getattr(self, "_h", None)
        if h is not None and h.value and _lib._lib is not None:
            _lib._lib.stencil_destroy(h)
            self._h = None


class Plan:
    """An execution plan for T_steps steps: tile validation + launch table (host only);
    `run` enqueues the phase kernels on the current CUDA stream."""

    def __init__(self, stencil: Stencil, T_steps: int, h: int = 0, w0: int = 0,
                 w: Sequence[int] = (0, 0, 0), hex_dim: int = -1, executor: str = "auto"):
        self.stencil = stencil
        self.T_steps = int(T_steps)
        t = Tile(int(h), int(w0), (ctypes.c_int32 * 3)(*list(w)[:3]), int(hex_dim), EXEC[executor])
        hp = ctypes.c_void_p()
        check(lib().stencil_plan(ctypes.byref(hp), stencil._h, self.T_steps, ctypes.byref(t)))
        self._h = hp
        self._ws = None

    @classmethod
    def _adopt(cls, stencil: "Stencil", handle, T_steps: int) -> "Plan":
        """Wrap a plan handle created elsewhere in the library (e.g. a slab's local plan)."""
        p = cls.__new__(cls)
        p.stencil = stencil
        p.T_steps = int(T_steps)
        p._h = handle
        p._ws = None
        return p

    # ---- introspection --------------------------------------------------------------
    @property
    def info(self) -> Dict[str, object]:
        i = PlanInfo()
        check(lib().stencil_plan_info(self._h, ctypes.byref(i)))
        out = {}
        for name, _ in PlanInfo._fields_:
            v = getattr(i, name)
            out[name] = list(v) if isinstance(v, ctypes.Array) else v
        return out

    @property
    def executor_name(self) -> str:
        """Which kernel family runs: fast2d / fdtd / fast3d / stream3d (specialised) or generic / naive."""
        return _lib.KERNELS[self.info["kernel"]]

    def launches(self) -> List[Dict[str, int]]:
        n = ctypes.c_int64()
        check(lib().stencil_plan_launches(self._h, None, 0, ctypes.byref(n)))
        arr = (Launch * max(1, n.value))()
        check(lib().stencil_plan_launches(self._h, arr, n.value, ctypes.byref(n)))
        return [{k: getattr(arr[i], k) for k, _ in Launch._fields_} for i in range(n.value)]

    def hexagon(self) -> Tuple[List[int], List[int]]:
        H = self.info["H"]
        lo = (ctypes.c_int32 * H)()
        hi = (ctypes.c_int32 * H)()
        check(lib().stencil_plan_hexagon(self._h, lo, hi, H))
        return list(lo), list(hi)

    def schedule_of(self, tau: int, s: Sequence[int]) -> Tuple[int, ...]:
        d = self.stencil.dims
        sp = (ctypes.c_int64 * d)(*[int(x) for x in s])
        out = (ctypes.c_int64 * (2 * d + 3))()
        check(lib().stencil_plan_schedule_of(self._h, int(tau), sp, out))
        return tuple(out)

    @property
    def workspace_bytes(self) -> int:
        n = ctypes.c_size_t()
        check(lib().stencil_plan_workspace_size(self._h, ctypes.byref(n)))
        return n.value

    # ---- execution ------------------------------------------------------------------
    def _ensure_workspace(self, device):
        import torch

        nbytes = self.workspace_bytes
        if nbytes == 0:
            check(lib().stencil_plan_set_workspace(self._h, None, 0))
            return
        if self._ws is None or self._ws.device != device:
            self._ws = torch.empty(nbytes + 256, dtype=torch.uint8, device=device)
        ptr = self._ws.data_ptr()
        ptr = (ptr + 255) // 256 * 256
        check(lib().stencil_plan_set_workspace(self._h, ctypes.c_void_p(ptr), nbytes))

    def run(self, inputs, out=None, stream=None):
        """Run T_steps steps.  inputs: a CUDA tensor (or a list of 3 for FDTD: ex, ey, hz),
        contiguous, dtype/shape of the descriptor.  out: same structure (default: new
        tensors; may be the inputs themselves for in-place).  Returns out."""
        import torch

        single = not isinstance(inputs, (list, tuple))
        ins = [inputs] if single else list(inputs)
        if len(ins) != self.stencil.n_fields:
            raise StencilError(1, f"expected {self.stencil.n_fields} field(s)")
        for x in ins:
            if not x.is_cuda or not x.is_contiguous() or tuple(x.shape) != self.stencil.extents:
                raise StencilError(1, "inputs must be contiguous CUDA tensors of the descriptor's shape")
            if _dtype_code(x.dtype) != self.stencil.dtype_code:
                raise StencilError(1, "input dtype differs from the descriptor's")
        if out is None:
            outs = [torch.empty_like(x) for x in ins]
        else:
            outs = [out] if single else list(out)
            # stencil_run writes whole grids through these pointers: same checks as the inputs
            if len(outs) != len(ins):
                raise StencilError(1, f"expected {len(ins)} output field(s)")
            for o in outs:
                if not isinstance(o, torch.Tensor) or not o.is_cuda or not o.is_contiguous():
                    raise StencilError(1, "outputs must be contiguous CUDA tensors")
                if tuple(o.shape) != self.stencil.extents:
                    raise StencilError(1, "output shape differs from the descriptor's extents")
                if _dtype_code(o.dtype) != self.stencil.dtype_code:
                    raise StencilError(1, "output dtype differs from the descriptor's")
                if o.device != ins[0].device:
                    raise StencilError(1, "outputs must live on the inputs' device")
        if any(x.device != ins[0].device for x in ins):
            raise StencilError(1, "all input fields must live on one device")
        self._ensure_workspace(ins[0].device)
        n = len(ins)
        in_p = (ctypes.c_void_p * n)(*[x.data_ptr() for x in ins])
        out_p = (ctypes.c_void_p * n)(*[x.data_ptr() for x in outs])
        if stream is None:
            stream = torch.cuda.current_stream(ins[0].device)
        sp = ctypes.c_void_p(stream.cuda_stream if hasattr(stream, "cuda_stream") else int(stream))
        check(lib().stencil_run(self._h, in_p, out_p, self.T_steps, sp))
        return outs[0] if single else outs

    def profile(self, max_runs: int) -> None:
        """Record per-launch CUDA events for the next max_runs runs (0 disables)."""
        check(lib().stencil_plan_profile(self._h, int(max_runs)))

    def profile_read(self) -> Dict[str, float]:
        ms, n, mx = ctypes.c_double(), ctypes.c_int64(), ctypes.c_double()
        check(lib().stencil_plan_profile_read(self._h, ctypes.byref(ms), ctypes.byref(n), ctypes.byref(mx)))
        return {"kernel_ms": ms.value, "launches": n.value, "max_launch_ms": mx.value}

    def run_ptrs(self, in_ptrs: Sequence[int], out_ptrs: Sequence[int], stream_ptr: int = 0):
        """Raw-pointer entry (device pointers as ints), e.g. for host-side drivers."""
        n = len(in_ptrs)
        in_p = (ctypes.c_void_p * n)(*in_ptrs)
        out_p = (ctypes.c_void_p * n)(*out_ptrs)
        check(lib().stencil_run(self._h, in_p, out_p, self.T_steps, ctypes.c_void_p(stream_ptr)))

    def __del__(self):
        h = getattr(self, "_h", None)
        if h is not None and h.value and _lib._lib is not None:
            _lib._lib.stencil_destroy(h)
            self._h = None


def run(kind: str, grid, T_steps: int, coefficients=None, **tile):
    """One-shot helper: plan and run `kind` for T_steps on `grid` (CUDA tensor or list)."""
    g0 = grid[0] if isinstance(grid, (list, tuple)) else grid
    st = Stencil(kind, tuple(g0.shape), dtype=g0.dtype, coefficients=coefficients)
    return Plan(st, T_steps, **tile).run(grid)
