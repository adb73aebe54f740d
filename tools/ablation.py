"""B200 replay of the optimisation ablation of Sec. 6.2 (Table 4 / Table 5).

  python tools/ablation.py time  [--shape 512,512,512] [--T 48]      -> one JSON line per config
  python tools/ablation.py one CFG [--shape ...] [--T ...]           -> a single run (for ncu)
  python tools/ablation.py table METRICS.csv TIMES.jsonl             -> the markdown table

Configurations: (a)-(f) = STENCIL_EXEC_T4A..T4F (kernels/ablation.cu: Table 4's tile h=2, w0=7,
w1=10, w2=32, CTA 1x10x32); "generic" = the Sec. 4.1 mapping of kernels/generic.cu (its own
classical tiles, global memory); "fast3d" = the product 3D kernel at the same (h, w0) with its own
classical tile (levels in shared memory, TMA-staged, register-blocked rows); "auto" = what the
planner picks.  Work = interior updates; GFLOP/s counts 27 flops per update (26 adds + 1 mul,
as the paper's Table 4 / Table 1 consistency check implies: 105 GFLOPS / 27 = 3.9 GStencil/s).
"""
import argparse
import csv
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

CFGS = [("a", "t4a", {}), ("b", "t4b", {}), ("c", "t4c", {}), ("d", "t4d", {}), ("e", "t4e", {}),
        ("f", "t4f", {}), ("generic", "generic", {"h": 2, "w0": 7}), ("fast3d", "auto", {"h": 2, "w0": 7}),
        ("auto", "auto", {})]
KIND = "box3d27"
FLOPS = 27


def _plan(name, shape, T):
    from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil

    for n, ex, tile in CFGS:
        if n == name:
            return Plan(Stencil(KIND, shape), T, executor=ex, hex_dim=0, **tile)
    raise SystemExit(f"unknown config {name}")


def _input(shape):
    import torch

    g = torch.Generator(device="cuda").manual_seed(7)
    return torch.rand(shape, generator=g, device="cuda", dtype=torch.float32)


def cmd_time(args):
    import torch

    shape = tuple(int(v) for v in args.shape.split(","))
    x = _input(shape)
    out = torch.empty_like(x)
    upd = (shape[0] - 2) * (shape[1] - 2) * (shape[2] - 2) * args.T
    for name, _, _ in CFGS:
        plan = _plan(name, shape, args.T)
        plan.run(x, out=out)  # eager first run (attributes, occupancy)
        torch.cuda.synchronize()
        plan.profile(args.reps)
        for _ in range(args.reps):
            plan.run(x, out=out)
        torch.cuda.synchronize()
        prof = plan.profile_read()
        ms = prof["kernel_ms"] / args.reps
        info = plan.info
        print(json.dumps({"config": name, "kernel": plan.executor_name, "h": info["h"], "w0": info["w0"],
                          "w": info["w"][:2], "shape": list(shape), "T": args.T, "ms": ms,
                          "gups": upd / ms / 1e6, "gflops": FLOPS * upd / ms / 1e6,
                          "launches": prof["launches"] // args.reps}), flush=True)


def cmd_one(args):
    import torch

    shape = tuple(int(v) for v in args.shape.split(","))
    x = _input(shape)
    plan = _plan(args.cfg, shape, args.T)
    plan.run(x)
    torch.cuda.synchronize()


METRICS = ["gpu__time_duration.sum", "dram__bytes_read.sum", "dram__bytes_write.sum", "lts__t_bytes.sum",
           "lts__t_sectors_srcunit_tex_op_read.sum", "smsp__inst_executed_op_global_ld.sum", "smsp__inst_executed_op_shared_ld.sum",
           "l1tex__data_pipe_lsu_wavefronts_mem_shared_op_ld.sum",
           "smsp__sass_average_data_bytes_per_sector_mem_global_op_ld.pct"]


def cmd_table(args):
    """Sum the per-launch ncu rows of each config (file per config: <dir>/abl_<cfg>.csv) and
    normalise by the run's updates; join with the timing lines."""
    times = {}
    for line in open(args.times):
        line = line.strip()
        if line.startswith("{"):
            d = json.loads(line)
            times[d["config"]] = d
    shape = tuple(int(v) for v in args.shape.split(","))
    upd = (shape[0] - 2) * (shape[1] - 2) * (shape[2] - 2) * args.T
    rows = []
    for name, _, _ in CFGS:
        path = os.path.join(args.dir, f"abl_{name}.csv")
        if not os.path.exists(path):
            continue
        lines = [l for l in open(path) if l.startswith('"')]
        rd = list(csv.reader(lines))
        if not rd:
            continue
        hdr = rd[0]
        tot = {m: 0.0 for m in METRICS}
        eff_w = eff_n = 0.0
        # long format: one row per (launch, metric); byte / ns / count units as ncu prints them
        for r in rd[1:]:
            d = dict(zip(hdr, r))
            m, v = d.get("Metric Name"), d.get("Metric Value", "").replace(",", "")
            if m not in METRICS:
                continue
            try:
                v = float(v)
            except ValueError:
                continue
            if m.endswith(".pct"):  # gld efficiency: mean over the launches
                eff_w += v
                eff_n += 1
            else:
                tot[m] += v
        t = times.get(name, {})
        rows.append((name, t, tot, eff_w / eff_n if eff_n else float("nan")))
    t0 = next(iter(times.values()), {})
    print(f"box3d27 (the paper's heat 3D), fp32.  Rates: {t0.get('shape')} T={t0.get('T')}, CUDA events around "
          f"the phase kernels of a run (tools/ablation.py time).  Counters: {shape[0]}x{shape[1]}x{shape[2]}, "
          f"T={args.T} ({upd / 1e9:.3f} G updates), ncu over every launch of one run, per update.\n")
    print("| config | kernel (h,w0; w1 x w2) | GUp/s | GFLOP/s | vs (a) | DRAM B/upd (rd+wr) | DRAM rd B/upd | "
          "L2 rd sectors/upd | L2 B/upd | global ld (warp instr)/upd | shared ld wavefronts/request | gld efficiency |")
    print("|---|---|---|---|---|---|---|---|---|---|---|---|")
    base = None
    for name, t, tot, eff in rows:
        g = t.get("gups", float("nan"))
        if name == "a":
            base = g
        dram = (tot["dram__bytes_read.sum"] + tot["dram__bytes_write.sum"]) / upd
        l2 = tot["lts__t_bytes.sum"] / upd
        gld = tot["smsp__inst_executed_op_global_ld.sum"] / upd
        drd = tot["dram__bytes_read.sum"] / upd
        l2rd = tot["lts__t_sectors_srcunit_tex_op_read.sum"] / upd
        req = tot["smsp__inst_executed_op_shared_ld.sum"]
        spr = tot["l1tex__data_pipe_lsu_wavefronts_mem_shared_op_ld.sum"] / req if req else float("nan")
        kern = f"{t.get('kernel', '?')} ({t.get('h')},{t.get('w0')}; {t.get('w', ['?', '?'])[0]}x{t.get('w', ['?', '?'])[1]})"
        rel = f"{g / base:.2f}x" if base else "-"
        print(f"| ({name}) | {kern} | {g:.1f} | {FLOPS * g:.0f} | {rel} | {dram:.2f} | {drd:.2f} | {l2rd:.3f} | "
              f"{l2:.2f} | {gld:.4f} | {spr:.2f} | {eff:.0f}% |")


def main():
    ap = argparse.ArgumentParser()
    sub = ap.add_subparsers(dest="cmd", required=True)
    a = sub.add_parser("time")
    a.add_argument("--shape", default="512,512,512")
    a.add_argument("--T", type=int, default=48)
    a.add_argument("--reps", type=int, default=3)
    b = sub.add_parser("one")
    b.add_argument("cfg")
    b.add_argument("--shape", default="256,256,256")
    b.add_argument("--T", type=int, default=12)
    c = sub.add_parser("table")
    c.add_argument("dir")
    c.add_argument("times")
    c.add_argument("--shape", default="256,256,256")
    c.add_argument("--T", type=int, default=12)
    args = ap.parse_args()
    {"time": cmd_time, "one": cmd_one, "table": cmd_table}[args.cmd](args)


if __name__ == "__main__":
    main()
