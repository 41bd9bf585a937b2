"""DRAM traffic per launch from one `ncu --set full` capture, for bench.py's
roofline "traffic" field:
    python scripts/ncu_traffic.py <tenant> <report.ncu-rep> [--out profiles/ncu_traffic.json]"""
import argparse
import csv
import io
import json
import os
import subprocess


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("tenant")
    ap.add_argument("report")
    ap.add_argument("--out", default=os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))),
                                                  "profiles", "ncu_traffic.json"))
    a = ap.parse_args()
    out = subprocess.run(["ncu", "-i", a.report, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(out)))
    h, units, data = rows[0], rows[1], rows[2:]
    scale = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9}
    recs = []
    for r in data:
        def val(k):
            i = h.index(k)
            return float(r[i].replace(",", "")) * scale.get(units[i], 1)
        recs.append({"kernel": r[h.index("Kernel Name")], "read": val("dram__bytes_read.sum"),
                     "write": val("dram__bytes_write.sum"),
                     "time_us": float(r[h.index("gpu__time_duration.sum")].replace(",", "")) *
                     (1e-3 if units[h.index("gpu__time_duration.sum")] == "nsecond" else
                      1e3 if units[h.index("gpu__time_duration.sum")] == "msecond" else 1)})
    rec = recs[0]
    db = json.load(open(a.out)) if os.path.exists(a.out) else {}
    db[a.tenant] = {"dram_bytes_per_launch": rec["read"] + rec["write"], "dram_read": rec["read"],
                    "dram_write": rec["write"], "kernel": rec["kernel"], "ncu_time_us": rec["time_us"],
                    "source": os.path.basename(a.report) + " (ncu --set full --clock-control none, one launch)"}
    json.dump(db, open(a.out, "w"), indent=1)
    print(json.dumps(db[a.tenant]))


if __name__ == "__main__":
    main()
