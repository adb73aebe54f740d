"""Multi-GPU slab mode: one process per GPU, the outermost grid dimension
slab-partitioned over the ranks, halos of width radius x D exchanged over torch.distributed
(NCCL over NVLink 5 / NVSwitch on the GPU box) once per time block of D steps.

Per rank the local grid is its owned planes plus G = r*D ghost planes on every side that is
not a global boundary.  A block runs the hybrid-tiled hot path (the C ABI's stencil_run) for
D steps on the local grid, whose outermost ghost plane acts as a frozen (Dirichlet) plane;
after D steps every owned plane is exact, because the dependence cone of an owned point over
D steps reaches r*D planes (overlapped tiling at rank edges only -- inside a rank the hybrid
schedule has no redundant work).  The exchange then refreshes the ghost
planes from the neighbours' owned planes (ncclSend/ncclRecv pairs via batch_isend_irecv).

Only the host-side partition / exchange logic lives here; every time step runs in
libhexstencil.so.  CPU tests (tests/test_dist_gloo.py) drive the same class over the gloo
backend with an injected compute callable to check the partition and halo logic.
"""
from __future__ import annotations

import json
import os
from dataclasses import dataclass
from typing import Callable, List, Optional, Sequence, Tuple

import torch
import torch.distributed as dist


@dataclass(frozen=True)
class Slab:
    rank: int
    nranks: int
    N0: int          # global extent of the partitioned (outermost) dimension
    own_lo: int      # owned global planes [own_lo, own_hi)
    own_hi: int
    loc_lo: int      # local grid covers global planes [loc_lo, loc_hi)
    loc_hi: int
    ghost: int       # G

    @property
    def local_extent(self) -> int:
        return self.loc_hi - self.loc_lo

    @property
    def own_local(self) -> Tuple[int, int]:
        return self.own_lo - self.loc_lo, self.own_hi - self.loc_lo


def partition(N0: int, nranks: int, rank: int, ghost: int) -> Slab:
    """Owned ranges split as evenly as possible; ghosts clipped at the global boundary."""
    base, extra = divmod(N0, nranks)
    lo = rank * base + min(rank, extra)
    hi = lo + base + (1 if rank < extra else 0)
    if hi - lo < ghost:
        raise ValueError(f"slab of {hi - lo} planes is thinner than the ghost width {ghost}")
    return Slab(rank, nranks, N0, lo, hi, max(0, lo - ghost), min(N0, hi + ghost), ghost)


def exchange_halos(local: torch.Tensor, slab: Slab, group=None) -> None:
    """Refresh the ghost planes of `local` (leading dim = planes) from the neighbours:
    send my first / last G owned planes down / up, receive their owned planes into my
    ghosts.  One batch of point-to-point ops (NCCL group send/recv on GPUs)."""
    G = slab.ghost
    lo, hi = slab.own_local
    ops = []
    if slab.rank > 0:
        ops.append(dist.P2POp(dist.isend, local[lo:lo + G], slab.rank - 1, group))
        ops.append(dist.P2POp(dist.irecv, local[lo - G:lo], slab.rank - 1, group))
    if slab.rank < slab.nranks - 1:
        ops.append(dist.P2POp(dist.isend, local[hi - G:hi], slab.rank + 1, group))
        ops.append(dist.P2POp(dist.irecv, local[hi:hi + G], slab.rank + 1, group))
    if ops:
        for req in dist.batch_isend_irecv(ops):
            req.wait()


def time_blocks(T: int, D: int) -> List[int]:
    """Block lengths: D steps each, the remainder last."""
    out = [D] * (T // D)
    if T % D:
        out.append(T % D)
    return out


class SlabRunner:
    """Runs `T` steps of a stencil on a slab-partitioned grid.

    compute(local_tensor, steps) advances the local grid by `steps` steps in place; by
    default it is the C-ABI hybrid-tiled path on the rank's GPU (one Plan per distinct
    block length, built once)."""

    def __init__(self, kind: str, global_extents: Sequence[int], T: int, D: int = 64,
                 group=None, compute: Optional[Callable[[torch.Tensor, int], None]] = None,
                 dtype=torch.float32, **tile):
        self.kind = kind
        self.ext = tuple(int(e) for e in global_extents)
        self.T = int(T)
        self.D = int(max(1, min(D, T))) if T > 0 else 1
        self.group = group
        self.rank = dist.get_rank(group)
        self.nranks = dist.get_world_size(group)
        self.slab = partition(self.ext[0], self.nranks, self.rank, ghost=self.D)
        self.local_ext = (self.slab.local_extent,) + self.ext[1:]
        self.blocks = time_blocks(self.T, self.D)
        self._compute = compute
        self._plans = {}
        self._tile = tile
        self._dtype = dtype

    def _gpu_compute(self, local: torch.Tensor, steps: int) -> None:
        from .api import Plan, Stencil

        plan = self._plans.get(steps)
        if plan is None:
            st = Stencil(self.kind, self.local_ext, dtype=self._dtype)
            plan = self._plans[steps] = Plan(st, steps, **self._tile)
        plan.run(local, out=local)

    def compute(self, local: torch.Tensor, steps: int) -> None:
        if self._compute is not None:
            self._compute(local, steps)
        else:
            self._gpu_compute(local, steps)

    def scatter_view(self, global_grid) -> torch.Tensor:
        """The rank's local part (owned + ghost planes) of a full global grid."""
        s = self.slab
        return global_grid[s.loc_lo:s.loc_hi]

    def run(self, local: torch.Tensor) -> torch.Tensor:
        """Advance `local` (owned + ghost planes, ghosts valid at level 0) by T steps.
        Returns local; its owned planes hold level T."""
        for i, steps in enumerate(self.blocks):
            if i > 0:
                exchange_halos(local, self.slab, self.group)
            self.compute(local, steps)
        return local

    def updates(self) -> int:
        """Interior points x T of the GLOBAL problem (the metric's numerator)."""
        n = 1
        for e in self.ext:
            n *= e - 2
        return n * self.T

    def redundant_fraction(self) -> float:
        s = self.slab
        return (s.local_extent - (s.own_hi - s.own_lo)) / max(1, s.own_hi - s.own_lo)


def bench_main(args, cfg, configs, metric, helpers=None):
    """bench.py --gpus N under torchrun: weak scaling, each rank owns the config's grid.
    `helpers` is the bench module (clock sampler, roofline model, peaks)."""
    import stencil_inputs

    kind, ext, T, cname = configs[cfg]
    rank = int(os.environ["RANK"])
    world = int(os.environ["WORLD_SIZE"])
    local_rank = int(os.environ.get("LOCAL_RANK", "0"))
    torch.cuda.set_device(local_rank)
    dist.init_process_group("nccl", device_id=torch.device("cuda", local_rank))
    gext = (ext[0] * world,) + tuple(ext[1:])
    D = int(os.environ.get("HEXS_TIME_BLOCK", "128"))
    runner = SlabRunner(kind, gext, T, D=D)

    # each rank generates only its local planes of the global synthetic grid (same recipe)
    s = runner.slab
    plane = 1
    for e in gext[1:]:
        plane *= e
    local_np = stencil_inputs.uniform((s.local_extent,) + tuple(gext[1:]), seed=0, offset=s.loc_lo * plane)
    host_in = torch.from_numpy(local_np).pin_memory()
    local0 = host_in.cuda()
    local = torch.empty_like(local0)
    stream = torch.cuda.current_stream()

    def step():
        local.copy_(local0)
        runner.run(local)

    for _ in range(max(3, args.warmup)):
        step()
    torch.cuda.synchronize()
    dist.barrier()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    sampler = helpers.ClockSampler(local_rank) if helpers is not None else None
    if sampler is not None:
        sampler.__enter__()
    e0.record(stream)
    for _ in range(args.steps):
        step()
    e1.record(stream)
    torch.cuda.synchronize()
    if sampler is not None:
        sampler.__exit__(None, None, None)
    ms = torch.tensor([e0.elapsed_time(e1) / args.steps], device="cuda")
    dist.all_reduce(ms, op=dist.ReduceOp.MAX)
    ms = float(ms.item())
    value = runner.updates() / (ms * 1e-3) / 1e9

    # end to end through the public API: pinned H2D of the rank's slab, the run (halo
    # exchanges included), D2H of the owned planes; two slab buffers and H2D / D2H streams
    # overlap a step's transfers with its neighbours' compute (as the single-GPU bench does)
    lo, hi = s.own_local
    host_out = [torch.empty_like(host_in[lo:hi]).pin_memory() for _ in range(2)]
    locs = [local, torch.empty_like(local)]
    h2d, d2h = torch.cuda.Stream(), torch.cuda.Stream()
    ev_in = [torch.cuda.Event() for _ in range(2)]
    ev_done = [torch.cuda.Event() for _ in range(2)]
    ev_out = [torch.cuda.Event() for _ in range(2)]
    for k in range(2):  # warm both slab buffers (the library captures a CUDA graph per pointer set)
        for _ in range(2):
            locs[k].copy_(local0)
            runner.run(locs[k])
    dist.barrier()
    torch.cuda.synchronize()
    f0, f1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    f0.record(stream)
    h2d.wait_event(f0)
    for i in range(args.steps):
        k = i % 2
        with torch.cuda.stream(h2d):
            if i >= 2:
                # the slab buffer is both input and output: its previous step's compute AND
                # the download of that step's result must be done before it is overwritten
                h2d.wait_event(ev_done[k])
                h2d.wait_event(ev_out[k])
            locs[k].copy_(host_in, non_blocking=True)
            ev_in[k].record(h2d)
        stream.wait_event(ev_in[k])
        if i >= 2:
            stream.wait_event(ev_out[k])
        runner.run(locs[k])
        ev_done[k].record(stream)
        with torch.cuda.stream(d2h):
            d2h.wait_event(ev_done[k])
            host_out[k].copy_(locs[k][lo:hi], non_blocking=True)
            ev_out[k].record(d2h)
    stream.wait_event(ev_out[(args.steps - 1) % 2])
    stream.wait_event(ev_out[args.steps % 2])
    f1.record(stream)
    torch.cuda.synchronize()
    e2e_ms = torch.tensor([f0.elapsed_time(f1) / args.steps], device="cuda")
    dist.all_reduce(e2e_ms, op=dist.ReduceOp.MAX)
    e2e_ms = float(e2e_ms.item())
    # the pipelined result equals a device-resident run's owned planes
    ref = local0.clone()
    runner.run(ref)
    torch.cuda.synchronize()
    assert torch.equal(host_out[(args.steps - 1) % 2], ref[lo:hi].cpu()), "pipelined e2e result differs"
    host_out = host_out[0]

    # phase-kernel roofline of the main block plan (algorithmic bytes / measured launch time)
    roof = None
    plan = runner._plans.get(runner.D)
    launches = sum(runner._plans[b].info["n_launches"] for b in runner.blocks)
    if plan is not None and helpers is not None:
        plan.profile(1)
        step()
        prof = plan.profile_read()
        plan.profile(0)
        info = plan.info
        bpu = helpers.bytes_per_update_tiled(info, 4, plan)
        avg = prof["kernel_ms"] / max(1, prof["launches"])
        alg = info["updates"] / info["n_launches"] * bpu
        peak, peak_src = helpers.load_peaks()
        roof = {"bound": "hbm", "achieved": alg / (avg * 1e-3) / 1e9, "peak": peak, "unit": "GB/s",
                "frac": alg / (avg * 1e-3) / 1e9 / peak, "traffic": None, "peak_source": peak_src,
                "kernel": helpers.KERNEL_NAMES.get(plan.executor_name, plan.executor_name),
                "bytes_per_update": bpu, "avg_launch_ms": avg}
    if rank == 0:
        nbytes_in = host_in.numel() * host_in.element_size()
        nbytes_out = host_out.numel() * host_out.element_size()
        line = {"metric": metric, "value": value, "unit": "GStencil-updates/s", "n_gpus": world,
                "steps": args.steps, "warmup": args.warmup, "ms_per_step": ms,
                "higher_is_better": True, "scaling": "weak", "vs_baseline": None, "dtype": "f32",
                "data": "synthetic",
                "config": {"workload": cname + f" weak-scaled to {gext[0]} planes over {world} GPUs",
                           "kind": kind, "extents": list(gext), "T": T, "time_block": runner.D,
                           "ghost_planes": runner.slab.ghost,
                           "redundant_fraction": runner.redundant_fraction(),
                           "l2": "inputs larger than L2 (per-rank slab > 126 MB)"},
                "roofline": roof,
                "cpu_baseline": None,
                "e2e": {"value": runner.updates() / (e2e_ms * 1e-3) / 1e9, "unit": "GStencil-updates/s",
                        "h2d_bytes_per_step": nbytes_in * world, "d2h_bytes_per_step": nbytes_out * world,
                        "ms_per_step": e2e_ms,
                        "pipelined": "2 slab buffers; H2D and D2H streams overlap the neighbouring steps' compute"},
                "gpu_launches": launches * args.steps,
                "clocks": sampler.summary() if sampler is not None else None}
        print(json.dumps(line), flush=True)
    dist.destroy_process_group()
