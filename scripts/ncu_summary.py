"""Summarise .ncu-rep files: key metrics + top warp stall reasons.
    python scripts/ncu_summary.py gpurun_out/x.ncu-rep ..."""
import csv
import io
import subprocess
import sys

KEYS = ["gpu__time_duration.sum", "dram__bytes_read.sum", "dram__bytes_write.sum",
        "dram__throughput.avg.pct_of_peak_sustained_elapsed", "lts__t_bytes.sum",
        "lts__t_sector_hit_rate.pct", "sm__throughput.avg.pct_of_peak_sustained_elapsed",
        "sm__warps_active.avg.pct_of_peak_sustained_active", "smsp__issue_active.avg.pct_of_peak_sustained_active",
        "smsp__inst_executed.sum", "sm__pipe_fma_cycles_active.avg.pct_of_peak_sustained_active",
        "sm__pipe_alu_cycles_active.avg.pct_of_peak_sustained_active",
        "sm__inst_executed_pipe_xu.avg.pct_of_peak_sustained_active",
        "l1tex__throughput.avg.pct_of_peak_sustained_active", "launch__registers_per_thread",
        "launch__grid_size", "launch__occupancy_limit_registers", "sm__cycles_elapsed.avg.per_second"]


def raw(path):
    out = subprocess.run(["ncu", "-i", path, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(out)))
    return rows[0], rows[1], rows[2:]


for p in sys.argv[1:]:
    h, units, rows = raw(p)
    for r in rows:
        name = r[h.index("Kernel Name")] if "Kernel Name" in h else "?"
        print(f"== {p}  {name[:80]}")
        for k in KEYS:
            if k in h:
                i = h.index(k)
                print(f"   {k:70s} {r[i]:>14s} {units[i]}")
        st = [(h[i], r[i]) for i in range(len(h))
              if h[i].startswith("smsp__average_warp_latency_issue_stalled") or
              (h[i].startswith("smsp__warp_issue_stalled_") and h[i].endswith("_per_warp_active.pct"))]
        def f(x):
            try:
                return float(x)
            except ValueError:
                return 0.0
        st = sorted(st, key=lambda x: -f(x[1]))[:7]
        print("   stalls:", ", ".join(f"{a.split('stalled_')[1].replace('_per_warp_active.pct','')}={b}" for a, b in st))
