"""Print the key ncu metrics of a .ncu-rep (first kernel) — used to write profiles/*.md."""
import csv, subprocess, sys

KEYS = ["gpu__time_duration.sum", "sm__throughput.avg.pct_of_peak_sustained_elapsed",
        "smsp__issue_active.avg.pct_of_peak_sustained_active", "sm__cycles_active.avg",
        "gpc__cycles_elapsed.max", "smsp__inst_executed.sum", "smsp__thread_inst_executed.sum",
        "smsp__warps_active.avg.per_cycle_active", "smsp__warps_eligible.avg.per_cycle_active",
        "sm__pipe_fp64_cycles_active.avg.pct_of_peak_sustained_active",
        "sm__inst_executed_pipe_alu.avg.pct_of_peak_sustained_active",
        "sm__inst_executed_pipe_fma.avg.pct_of_peak_sustained_active",
        "sm__inst_executed_pipe_xu.avg.pct_of_peak_sustained_active",
        "sm__inst_executed_pipe_lsu.avg.pct_of_peak_sustained_active",
        "sm__inst_executed_pipe_uniform.avg.pct_of_peak_sustained_active",
        "dram__bytes_read.sum", "dram__bytes_write.sum", "launch__registers_per_thread",
        "launch__grid_size", "launch__occupancy_limit_registers", "sm__warps_active.avg.pct_of_peak_sustained_active",
        "sm__pipe_fmaheavy_cycles_active.avg.pct_of_peak_sustained_active"]


def main(path):
    out = subprocess.run(["ncu", "-i", path, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    rows = list(csv.reader(out.splitlines()))
    h, u, v = rows[0], rows[1], rows[2]
    d = {a: (b, c) for a, b, c in zip(h, u, v)}
    for k in KEYS:
        if k in d:
            print(f"{k:70s} {d[k][1]:>22s} {d[k][0]}")
    st = [(float(c.replace(',', '')), a) for a, b, c in zip(h, u, v)
          if a.startswith("smsp__average_warps_issue_stalled") and a.endswith("per_issue_active.ratio")]
    if "smsp__inst_executed.sum" in d and "smsp__thread_inst_executed.sum" in d:
        inst = float(d["smsp__inst_executed.sum"][1].replace(",", ""))
        tinst = float(d["smsp__thread_inst_executed.sum"][1].replace(",", ""))
        print(f"{'warp execution efficiency (thread_inst / (32 inst))':70s} {tinst / (32 * inst):>22.4f}")
    for val, name in sorted(st, reverse=True)[:8]:
        print(f"  stall {name.replace('smsp__average_warps_issue_stalled_', '').replace('_per_issue_active.ratio', ''):28s} {val:.3f}")


if __name__ == "__main__":
    main(sys.argv[1])
