"""Summarise an ncu report: key throughput, occupancy, stall and traffic metrics."""
import csv
import subprocess
import sys

KEYS = ["gpu__time_duration.sum", "sm__cycles_elapsed.avg", "sm__cycles_active.avg", "sm__cycles_active.max",
        "sm__cycles_active.min", "dram__bytes_read.sum", "dram__bytes_write.sum", "lts__t_bytes.sum",
        "sm__warps_active.avg.per_cycle_active", "smsp__issue_active.avg.pct_of_peak_sustained_active",
        "smsp__inst_executed.sum", "launch__registers_per_thread", "launch__grid_size",
        "launch__occupancy_limit_registers", "launch__occupancy_limit_shared_mem",
        "l1tex__data_pipe_lsu_wavefronts_mem_shared.sum", "l1tex__data_bank_conflicts_pipe_lsu_mem_shared.sum",
        "smsp__sass_thread_inst_executed_op_fadd_pred_on.sum", "smsp__sass_thread_inst_executed_op_fmul_pred_on.sum",
        "smsp__sass_thread_inst_executed_op_ffma_pred_on.sum", "sm__pipe_fma_cycles_active.avg.pct_of_peak_sustained_active",
        "smsp__inst_executed_op_shfl.sum", "dram__throughput.avg.pct_of_peak_sustained_elapsed",
        "local_load", "l1tex__t_bytes_pipe_lsu_mem_local_op_ld.sum", "l1tex__t_bytes_pipe_lsu_mem_local_op_st.sum"]


def main(path):
    raw = subprocess.run(["ncu", "-i", path, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    rows = list(csv.reader(raw.splitlines()))
    hdr, unit = rows[0], rows[1]
    for v in rows[2:]:
        d = dict(zip(hdr, v))
        u = dict(zip(hdr, unit))
        print("kernel:", d.get("Kernel Name", "")[:80])
        for k in KEYS:
            for name in hdr:
                if name == k:
                    print(f"  {k:70s} {d[name]:>20s} {u[name]}")
        stalls = []
        for name in hdr:
            if name.startswith("smsp__average_warps_issue_stalled_") and name.endswith("_per_issue_active.ratio"):
                try:
                    stalls.append((float(d[name].replace(",", "")), name[len("smsp__average_warps_issue_stalled_"):-len("_per_issue_active.ratio")]))
                except ValueError:
                    pass
        stalls.sort(reverse=True)
        print("  stalls per issue:", ", ".join(f"{n}={v:.2f}" for v, n in stalls[:8] if v > 0.02))


if __name__ == "__main__":
    main(sys.argv[1])
