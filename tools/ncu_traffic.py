"""Per-launch DRAM traffic of a config's phase kernel from an ncu launch list.

On the GPU box (one stencil_run, every launch of the phase kernel, cold-cache, serialised):
  ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum \
      --clock-control none -k regex:KERNEL --csv --log-file gpurun_out/launches_CFG.csv \
      python tools/run_once.py CFG 1
Here: python tools/ncu_traffic.py CFG gpurun_out/launches_CFG.csv
  -> profiles/round2/traffic_CFG.json (read by bench.py for roofline.traffic).
Also records L2 bytes per update (lts__t_bytes.sum) and the CTAs-per-launch histogram
(launch__grid_size) when the launch list carries them."""
import csv
import json
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)


def main(cfg, path):
    import bench
    from paper_conf_cgo_grosserchsv14_b200 import Plan, Stencil

    rows = [r for r in csv.reader(open(path)) if len(r) > 10]
    hdr = rows[0]
    ki, mi, vi, ui = hdr.index("Kernel Name"), hdr.index("Metric Name"), hdr.index("Metric Value"), hdr.index("Metric Unit")
    idi = hdr.index("ID")
    scale = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "nsecond": 1e-9, "usecond": 1e-6, "msecond": 1e-3,
             "second": 1.0}
    per = {}
    for r in rows[1:]:
        d = per.setdefault(r[idi], {"kernel": r[ki]})
        d[r[mi]] = float(r[vi].replace(",", "")) * scale.get(r[ui], 1.0)
    launches = list(per.values())
    kind, ext, T, _ = bench.CONFIGS[cfg][:4]
    plan = Plan(Stencil(kind, ext), T)
    info = plan.info
    tot_b = sum(l["dram__bytes_read.sum"] + l["dram__bytes_write.sum"] for l in launches)
    tot_t = sum(l["gpu__time_duration.sum"] for l in launches)
    bpu = bench.bytes_per_update_tiled(info, 4, plan)
    hist = {}
    for l in launches:
        if "launch__grid_size" in l:
            g = int(l["launch__grid_size"])
            hist[g] = hist.get(g, 0) + 1
    lts = sum(l.get("lts__t_bytes.sum", 0.0) for l in launches)
    out = {"config": cfg, "kernel": launches[0]["kernel"][:120], "launches": len(launches),
           "plan_launches": info["n_launches"], "tile": {"h": info["h"], "w0": info["w0"]},
           "dram_bytes_total": tot_b, "dram_bytes_per_launch": tot_b / len(launches),
           "dram_bytes_per_update": tot_b / info["updates"],
           "algorithmic_bytes_per_update": bpu,
           "kernel_time_total_s_cold_serialised": tot_t,
           "l2_bytes_per_update": lts / info["updates"] if lts else None,
           "ctas_per_launch_histogram": {str(k): v for k, v in sorted(hist.items())},
           "source": os.path.basename(path)}
    os.makedirs(os.path.join(ROOT, "profiles", "round2"), exist_ok=True)
    dst = os.path.join(ROOT, "profiles", "round2", f"traffic_{cfg}.json")
    json.dump(out, open(dst, "w"), indent=1)
    print(json.dumps(out, indent=1))


if __name__ == "__main__":
    main(sys.argv[1], sys.argv[2])
