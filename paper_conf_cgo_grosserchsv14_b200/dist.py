"""Multi-GPU slab mode over the C ABI's distributed plans.

One process per GPU.  The library (csrc/dist.cpp, include/stencil.h) partitions one
non-innermost grid dimension (`part_dim`; default y in 3D -- a classically tiled dimension --
and rows in 2D), keeps G = radius * (2h+2) ghost indices per interior side, runs the global
launch table of the hybrid schedule over the local slab and refreshes the ghosts of both
ping-pong buffers with ncclSend / ncclRecv before every launch but the first.  Python only bootstraps: rank 0 asks the library for
an NCCL unique id and torch.distributed broadcasts it; PyTorch provides the device memory.

    dp = DistPlan("star3d7", (1024, 1024, 1024), T=256)    # collective
    local = dp.scatter(global_grid)                        # this rank's slab (ghosts included)
    dp.run(local)                                          # collective; owned points -> level T
    owned = dp.owned(local)

`layout(...)` is the same partition as a host-only call (no GPU, no NCCL): the CPU tests
(tests/test_dist_gloo.py) drive the library's layout with the oracle as the per-block compute
and a gloo halo exchange (`exchange_halos`) to check the protocol bit for bit.
"""
from __future__ import annotations

import ctypes
import json
import os
import sys
from dataclasses import dataclass
from typing import Callable, List, Optional, Sequence, Tuple

import torch
import torch.distributed as dist

from . import _lib
from ._lib import DistInfo, EXEC, KINDS, StencilError, Tile, check, lib
from .api import _dtype_code


@dataclass(frozen=True)
class Layout:
    rank: int
    nranks: int
    part_dim: int
    global_ext: Tuple[int, ...]
    local_ext: Tuple[int, ...]
    own_lo: int
    own_hi: int
    loc_lo: int
    loc_hi: int
    ghost: int
    time_block: int
    n_blocks: int
    h: int
    ghost_fraction: float

    @property
    def own_local(self) -> Tuple[int, int]:
        return self.own_lo - self.loc_lo, self.own_hi - self.loc_lo

    def take(self, a, lo: int, hi: int):
        """a[..., lo:hi, ...] along the partitioned dimension (numpy or torch)."""
        idx = [slice(None)] * self.part_dim + [slice(lo, hi)]
        return a[tuple(idx)]



def _tile(h=0, w0=0, w=(0, 0, 0), hex_dim=-1, executor="auto") -> Tile:
    return Tile(int(h), int(w0), (ctypes.c_int32 * 3)(*list(w)[:3]), int(hex_dim), EXEC[executor])


def _desc(kind: str, ext: Sequence[int], dtype="float32"):
    if kind not in KINDS:
        raise StencilError(1, f"unknown stencil kind {kind!r}")
    e = (ctypes.c_int64 * len(ext))(*[int(x) for x in ext])
    h = ctypes.c_void_p()
    check(lib().stencil_desc_create(ctypes.byref(h), len(ext), e, KINDS[kind], 1, None, 0, None, 0,
                                    _dtype_code(dtype)))
    return h


def _layout_of(info: DistInfo, dims: int, global_ext: Sequence[int]) -> Layout:
    return Layout(info.rank, info.nranks, info.part_dim, tuple(int(x) for x in global_ext),
                  tuple(int(info.local_ext[q]) for q in range(dims)), info.own_lo, info.own_hi, info.loc_lo,
                  info.loc_hi, info.ghost, info.time_block, info.n_blocks, info.h, info.ghost_fraction)


def layout(kind: str, global_ext: Sequence[int], T: int, rank: int, nranks: int, dtype="float32",
           part_dim: int = -1, **tile) -> Layout:
    """This rank's slab layout, exactly as stencil_plan_dist builds it (host only)."""
    d = _desc(kind, global_ext, dtype)
    try:
        info = DistInfo()
        t = _tile(**tile)
        check(lib().stencil_dist_layout(d, int(T), ctypes.byref(t), int(rank), int(nranks), int(part_dim),
                                        ctypes.byref(info)))
        return _layout_of(info, len(global_ext), global_ext)
    finally:
        lib().stencil_destroy(d)


def local_plan(kind: str, global_ext: Sequence[int], T: int, rank: int, nranks: int, dtype="float32",
               part_dim: int = -1, **tile):
    """Rank `rank`'s local plan (host only; stencil_dist_local_plan): the global launch table of
    the hybrid schedule restricted to the slab -- what a distributed plan runs between its halo
    exchanges."""
    from .api import Plan, Stencil

    lay = layout(kind, global_ext, T, rank, nranks, dtype, part_dim, **tile)
    d = _desc(kind, global_ext, dtype)
    try:
        h = ctypes.c_void_p()
        t = _tile(**tile)
        check(lib().stencil_dist_local_plan(ctypes.byref(h), d, int(T), ctypes.byref(t), int(rank), int(nranks),
                                            int(part_dim)))
    finally:
        lib().stencil_destroy(d)
    return Plan._adopt(Stencil(kind, lay.local_ext, dtype=dtype), h, T), lay


def halo_rows(plan, part_dim: int, k: int, buffer: int) -> Optional[List[int]]:
    """The outer rows whose halo lines of `buffer` travel before launch k of a local plan
    (stencil_dist_halo_rows), or None when every row travels."""
    n = ctypes.c_int64()
    check(lib().stencil_dist_halo_rows(plan._h, int(part_dim), int(k), int(buffer), None, 0, ctypes.byref(n)))
    if n.value < 0:
        return None
    arr = (ctypes.c_int32 * max(1, n.value))()
    check(lib().stencil_dist_halo_rows(plan._h, int(part_dim), int(k), int(buffer), arr, n.value, ctypes.byref(n)))
    return list(arr[:n.value])


def exchange_halos(local: torch.Tensor, lay: Layout, group=None, rows: Optional[Sequence[int]] = None) -> None:
    """The library's halo step over torch.distributed (for CPU/gloo tests of the protocol):
    send my first / last G owned indices of the partitioned dimension down / up, receive the
    neighbours' into my ghosts (strided slabs through contiguous staging, as the library does);
    `rows`: only these outer (dimension-0) rows travel (the library's needed-state lists)."""
    G = lay.ghost
    lo, hi = lay.own_local
    sel = (lambda t: t) if rows is None else (lambda t: t[list(rows)])
    ops, unpack = [], []
    if lay.rank > 0:
        rl = torch.empty_like(sel(lay.take(local, lo - G, lo)).contiguous())
        ops.append(dist.P2POp(dist.isend, sel(lay.take(local, lo, lo + G)).contiguous(), lay.rank - 1, group))
        ops.append(dist.P2POp(dist.irecv, rl, lay.rank - 1, group))
        unpack.append((lo - G, lo, rl))
    if lay.rank < lay.nranks - 1:
        rh = torch.empty_like(sel(lay.take(local, hi, hi + G)).contiguous())
        ops.append(dist.P2POp(dist.isend, sel(lay.take(local, hi - G, hi)).contiguous(), lay.rank + 1, group))
        ops.append(dist.P2POp(dist.irecv, rh, lay.rank + 1, group))
        unpack.append((hi, hi + G, rh))
    if ops:
        for req in dist.batch_isend_irecv(ops):
            req.wait()
    for a, b, buf in unpack:
        if rows is None:
            lay.take(local, a, b).copy_(buf)
        else:
            view = lay.take(local, a, b)
            for i, z in enumerate(rows):
                view[z].copy_(buf[i])


def run_protocol(bufs: Sequence[torch.Tensor], lay: Layout, plan, execute_launch: Callable, group=None) -> None:
    """The distributed run of csrc/dist.cpp::run_dist with an injected launch executor and a
    torch.distributed exchange: for each launch of the rank's local plan, refresh the ghost
    planes of both ping-pong buffers (but before the first), then run the launch."""
    for k, ln in enumerate(plan.launches()):
        if k > 0 and lay.nranks > 1:
            for bi, b in enumerate(bufs):
                exchange_halos(b, lay, group, halo_rows(plan, lay.part_dim, k, bi))
        execute_launch(ln, bufs)


class DistPlan:
    """A distributed plan (stencil_plan_dist) of T steps of `kind` on the global grid
    `global_ext`, over the ranks of `group` (one GPU each).  Collective constructor."""

    def __init__(self, kind: str, global_ext: Sequence[int], T: int, group=None, dtype="float32",
                 part_dim: int = -1, rank: Optional[int] = None, nranks: Optional[int] = None,
                 unique_id: Optional[bytes] = None, **tile):
        """rank / nranks / unique_id: explicit (no process group) -- e.g. the loopback mode
        (HEXS_DIST_LOOPBACK=1), where all ranks are plans of one process on one device and share
        one id (any 128 bytes)."""
        self.kind = kind
        self.global_ext = tuple(int(e) for e in global_ext)
        self.T = int(T)
        self.group = group
        self.rank = dist.get_rank(group) if dist.is_initialized() else 0
        self.nranks = dist.get_world_size(group) if dist.is_initialized() else 1
        if rank is not None:
            self.rank, self.nranks = int(rank), int(nranks)
        emu = os.environ.get("HEXS_DIST_EMULATE_RANK")  # "r/P": play rank r of P alone (projection)
        if emu:
            r, P = (int(x) for x in emu.split("/"))
            os.environ.setdefault("HEXS_DIST_EMULATE", "1")  # "2": with the halo copies
            self.rank, self.nranks = r, P
        self._d = _desc(kind, self.global_ext, dtype)
        uid = (ctypes.c_char * 128)()
        if unique_id is not None:
            ctypes.memmove(uid, bytes(unique_id)[:128].ljust(128, b"\0"), 128)
        elif self.rank == 0:
            check(lib().stencil_dist_unique_id(uid))
        if self.nranks > 1 and not emu and unique_id is None:
            obj = [bytes(uid) if self.rank == 0 else None]
            dist.broadcast_object_list(obj, src=dist.get_global_rank(group, 0) if group is not None else 0,
                                       group=group)
            ctypes.memmove(uid, obj[0], 128)
        t = _tile(**tile)
        h = ctypes.c_void_p()
        check(lib().stencil_plan_dist(ctypes.byref(h), self._d, self.T, ctypes.byref(t), uid, self.rank,
                                      self.nranks, int(part_dim)))
        self._h = h
        info = DistInfo()
        check(lib().stencil_dist_info(h, ctypes.byref(info)))
        self.layout = _layout_of(info, len(self.global_ext), self.global_ext)
        self.launches_per_run = int(info.launches_per_run)
        self.exchange = _lib.EXCHANGES.get(int(info.exchange), str(info.exchange))
        self._ws = None
        self.dtype = dtype

    # ---- data placement ---------------------------------------------------------------
    def scatter(self, global_grid) -> torch.Tensor:
        """This rank's local slab (owned + ghost indices) of a full global grid, on its GPU."""
        lay = self.layout
        part = lay.take(global_grid, lay.loc_lo, lay.loc_hi)
        t = part if isinstance(part, torch.Tensor) else torch.from_numpy(part.copy())
        return t.contiguous().cuda()

    def owned(self, local: torch.Tensor) -> torch.Tensor:
        lo, hi = self.layout.own_local
        return self.layout.take(local, lo, hi)

    # ---- execution ----------------------------------------------------------------------
    @property
    def block_plan(self):
        """Borrowed handle of the D-step local plan (introspection / per-launch profiling)."""
        bp = ctypes.c_void_p()
        check(lib().stencil_dist_block_plan(self._h, 0, ctypes.byref(bp)))
        return bp

    def _ensure_workspace(self, device):
        n = ctypes.c_size_t()
        check(lib().stencil_plan_workspace_size(self._h, ctypes.byref(n)))
        if n.value == 0:
            return
        if self._ws is None or self._ws.device != device:
            self._ws = torch.empty(n.value + 256, dtype=torch.uint8, device=device)
            ptr = (self._ws.data_ptr() + 255) // 256 * 256
            # (once per allocation: setting it uploads the halo row lists synchronously)
            check(lib().stencil_plan_set_workspace(self._h, ctypes.c_void_p(ptr), n.value))

    def run(self, local: torch.Tensor, out: Optional[torch.Tensor] = None, stream=None) -> torch.Tensor:
        """Collective: T steps; `local` holds level 0 on every plane of the slab.  Returns the
        slab whose owned planes hold level T (in place unless `out` is given)."""
        lay = self.layout
        if not local.is_cuda or not local.is_contiguous() or tuple(local.shape) != lay.local_ext:
            raise StencilError(1, f"local slab must be a contiguous CUDA tensor of shape {lay.local_ext}")
        if out is None:
            out = local
        elif tuple(out.shape) != lay.local_ext or not out.is_contiguous() or out.device != local.device:
            raise StencilError(1, "out must match the local slab")
        self._ensure_workspace(local.device)
        if stream is None:
            stream = torch.cuda.current_stream(local.device)
        ip = (ctypes.c_void_p * 1)(local.data_ptr())
        op = (ctypes.c_void_p * 1)(out.data_ptr())
        check(lib().stencil_run(self._h, ip, op, self.T, ctypes.c_void_p(stream.cuda_stream)))
        return out

    def updates(self) -> int:
        """Interior points x T of the GLOBAL problem (the metric's numerator)."""
        n = 1
        for e in self.global_ext:
            n *= e - 2
        return n * self.T

    def __del__(self):
        if _lib._lib is None:
            return
        for attr in ("_h", "_d"):
            h = getattr(self, attr, None)
            if h is not None and h.value:
                _lib._lib.stencil_destroy(h)
                setattr(self, attr, None)


def bench_main(args, cfg, configs, metric, helpers):
    """bench.py under torchrun (or HEXS_FORCE_DIST=1 at N = 1): every rank runs its slab of the
    config's grid through a distributed plan.  Weak scaling for the configs whose outer extent
    grows with N (`weak`), strong scaling for the fixed-size 3D grid."""
    import stencil_inputs

    kind, ext, T, cname = configs[cfg][:4]
    scaling = configs[cfg][4] if len(configs[cfg]) > 4 else "weak"
    rank = int(os.environ.get("RANK", "0"))
    world = int(os.environ.get("WORLD_SIZE", "1"))
    local_rank = int(os.environ.get("LOCAL_RANK", "0"))
    torch.cuda.set_device(local_rank)
    if "RANK" not in os.environ:  # a single process (N = 1 without torchrun): a group of one
        import socket

        sk = socket.socket()
        sk.bind(("127.0.0.1", 0))
        os.environ.update({"RANK": "0", "WORLD_SIZE": "1", "LOCAL_RANK": "0", "MASTER_ADDR": "127.0.0.1",
                           "MASTER_PORT": str(sk.getsockname()[1])})
        sk.close()
    if not dist.is_initialized():
        dist.init_process_group("nccl", device_id=torch.device("cuda", local_rank))
    gext = ((ext[0] * world,) + tuple(ext[1:])) if scaling == "weak" else tuple(ext)
    tile = {}
    if getattr(args, "tile", ""):  # h,w0: the local plans' hexagon (tuning)
        v = [int(x) for x in args.tile.split(",")]
        tile = {"h": v[0], "w0": v[1]}
    part_dim = int(os.environ.get("HEXS_DIST_PART_DIM", "-1"))  # default: y in 3D (classical)
    dp = DistPlan(kind, gext, T, part_dim=part_dim, **tile)
    lay = dp.layout
    pd = lay.part_dim
    # each rank generates only its slab of the global synthetic grid (same counter-based recipe)
    box_lo = [0] * len(gext)
    box_hi = list(gext)
    box_lo[pd], box_hi[pd] = lay.loc_lo, lay.loc_hi
    local_np = stencil_inputs.uniform_box(gext, box_lo, box_hi, seed=0)
    host_in = torch.from_numpy(local_np).pin_memory()
    local0 = host_in.cuda()
    local = torch.empty_like(local0)
    stream = torch.cuda.current_stream()

    def step():
        dp.run(local0, local)

    for _ in range(max(3, args.warmup)):
        step()
    torch.cuda.synchronize()
    dist.barrier()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    sampler = helpers.ClockSampler(local_rank)
    sampler.__enter__()
    torch.cuda.synchronize()
    dist.barrier()
    e0.record(stream)
    for _ in range(args.steps):
        step()
    e1.record(stream)
    torch.cuda.synchronize()
    sampler.__exit__(None, None, None)
    ms = torch.tensor([e0.elapsed_time(e1) / args.steps], device="cuda")
    dist.all_reduce(ms, op=dist.ReduceOp.MAX)
    ms = float(ms.item())
    value = dp.updates() / (ms * 1e-3) / 1e9

    # end to end through the public API: pinned H2D of the rank's slab, the distributed run
    # (halo exchanges included), D2H of the owned planes; two slab buffer pairs and H2D / D2H
    # streams overlap a step's transfers with its neighbours' compute
    lo, hi = lay.own_local
    own_shape = tuple(lay.take(host_in, lo, hi).shape)
    host_out = [torch.empty(own_shape, dtype=host_in.dtype).pin_memory() for _ in range(2)]
    ins = [local0, torch.empty_like(local0)]
    outs = [local, torch.empty_like(local)]
    h2d, d2h = torch.cuda.Stream(), torch.cuda.Stream()
    ev_in = [torch.cuda.Event() for _ in range(2)]
    ev_done = [torch.cuda.Event() for _ in range(2)]
    ev_out = [torch.cuda.Event() for _ in range(2)]
    for k in range(2):
        ins[k].copy_(local0)
        dp.run(ins[k], outs[k])
    torch.cuda.synchronize()
    dist.barrier()
    f0, f1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    f0.record(stream)
    h2d.wait_event(f0)
    for i in range(args.steps):
        k = i % 2
        with torch.cuda.stream(h2d):
            if i >= 2:
                h2d.wait_event(ev_done[k])  # step i-2 consumed this input slab
            ins[k].copy_(host_in, non_blocking=True)
            ev_in[k].record(h2d)
        stream.wait_event(ev_in[k])
        if i >= 2:
            stream.wait_event(ev_out[k])  # step i-2's result has left this output slab
        dp.run(ins[k], outs[k])
        ev_done[k].record(stream)
        with torch.cuda.stream(d2h):
            d2h.wait_event(ev_done[k])
            host_out[k].copy_(lay.take(outs[k], lo, hi), non_blocking=True)
            ev_out[k].record(d2h)
    stream.wait_event(ev_out[(args.steps - 1) % 2])
    stream.wait_event(ev_out[args.steps % 2])
    f1.record(stream)
    torch.cuda.synchronize()
    e2e_ms = torch.tensor([f0.elapsed_time(f1) / args.steps], device="cuda")
    dist.all_reduce(e2e_ms, op=dist.ReduceOp.MAX)
    e2e_ms = float(e2e_ms.item())
    # the pipelined result equals the device-resident run's owned planes
    assert torch.equal(host_out[(args.steps - 1) % 2], lay.take(local, lo, hi).cpu()), "pipelined e2e result differs"

    # phase-kernel roofline of the D-step block plan: kernel-region events of one run
    bp = dp.block_plan
    check(lib().stencil_plan_profile(bp, 1))
    dp.run(local0, local)
    kms, nl, mx = ctypes.c_double(), ctypes.c_int64(), ctypes.c_double()
    check(lib().stencil_plan_profile_read(bp, ctypes.byref(kms), ctypes.byref(nl), ctypes.byref(mx)))
    check(lib().stencil_plan_profile(bp, 0))
    binfo = _lib.PlanInfo()
    check(lib().stencil_plan_info(bp, ctypes.byref(binfo)))
    bpu = 4 * (binfo.tile_in + binfo.tile_out) / binfo.tile_points
    upd_block = binfo.updates  # one D-step block on the local slab (ghost planes included)
    peak, peak_src = helpers.load_peaks()
    roof = None
    if nl.value > 0:
        achieved = upd_block * bpu / (kms.value * 1e-3) / 1e9
        roof = {"bound": "hbm", "achieved": achieved, "peak": peak, "unit": "GB/s", "frac": achieved / peak,
                "traffic": None, "peak_source": peak_src,
                "kernel": helpers.KERNEL_NAMES.get(_lib.KERNELS[binfo.kernel], _lib.KERNELS[binfo.kernel]),
                "bytes_per_update": bpu, "block_kernel_ms": kms.value, "block_launches": nl.value,
                "note": "the local plan on the rank's slab (ghosts included); ghost traffic not in "
                        "bytes_per_update"}
    if rank == 0:
        nbytes_in = host_in.numel() * host_in.element_size()
        nbytes_out = host_out[0].numel() * host_out[0].element_size()
        line = {"metric": metric, "value": value, "unit": "GStencil-updates/s", "n_gpus": world,
                "steps": args.steps, "warmup": args.warmup, "ms_per_step": ms,
                "higher_is_better": True, "scaling": scaling, "vs_baseline": None, "dtype": "f32",
                "data": "synthetic",
                "config": {"workload": cname + (f" weak-scaled to {gext[0]} planes over {world} GPUs"
                                                if scaling == "weak" else f" over {world} GPUs"),
                           "kind": kind, "extents": list(gext), "T": T, "partition": f"dim {pd} slabs",
                           "time_block": lay.time_block, "ghost_indices": lay.ghost, "halo_exchange": dp.exchange,
                           "ghost_fraction": lay.ghost_fraction, "local_extents": list(lay.local_ext),
                           "l2": "inputs larger than L2 (per-rank slab > 126 MB)"},
                "roofline": roof,
                "cpu_baseline": None,
                "e2e": {"value": dp.updates() / (e2e_ms * 1e-3) / 1e9, "unit": "GStencil-updates/s",
                        "h2d_bytes_per_step": nbytes_in * world, "d2h_bytes_per_step": nbytes_out * world,
                        "ms_per_step": e2e_ms,
                        "pipelined": "2 slab buffer pairs; H2D and D2H streams overlap the neighbouring steps' compute"},
                "gpu_launches": dp.launches_per_run * args.steps,
                "clocks": sampler.summary()}
        emu = os.environ.get("HEXS_DIST_EMULATE_RANK")
        if emu:  # a projection, not a measurement of N GPUs: say so and report the rank's rate
            r, P = (int(x) for x in emu.split("/"))
            own = lay.own_hi - lay.own_lo
            line["emulated_rank"] = {"rank": r, "nranks": P, "owned_indices": own, "part_dim": pd,
                                     "rank_gups": value * own / gext[pd],
                                     "note": "one GPU runs rank r's slab alone (ghosts fixed, no NCCL): compute-only "
                                             "projection; 'value' is the whole-grid rate of that rank's time"}
        print(json.dumps(line), flush=True)
    dist.barrier()
    dist.destroy_process_group()
