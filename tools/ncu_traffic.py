"""Summarise ncu --set full reports into profiles/ (per-launch DRAM traffic and
key counters) for bench.py's roofline.traffic field.

  python tools/ncu_traffic.py gpurun_out/prof_mandel_bench.ncu-rep:skl_map_vec:mandelbrot ...
  python tools/ncu_traffic.py profiles/r01_ncu_raw_lmosem.csv:skl_map_vec:lmosem   (raw page CSV)

Writes/updates profiles/ncu_traffic.json: {workload: {kernel, bytes_per_launch,
dram_read, dram_write, duration_ns, ...}}.
"""
import csv
import io
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
KEYS = {
    "gpu__time_duration.sum": "duration",
    "dram__bytes_read.sum": "dram_read",
    "dram__bytes_write.sum": "dram_write",
    "gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed": "dram_pct_of_peak",
    "sm__throughput.avg.pct_of_peak_sustained_elapsed": "sm_pct_of_peak",
    "sm__pipe_fma_cycles_active.avg.pct_of_peak_sustained_active": "fma_pipe_pct",
    "sm__pipe_alu_cycles_active.avg.pct_of_peak_sustained_active": "alu_pipe_pct",
    "sm__warps_active.avg.pct_of_peak_sustained_active": "warps_active_pct",
    "launch__registers_per_thread": "registers",
    "smsp__inst_executed.sum": "inst_executed",
    "smsp__issue_active.avg.pct_of_peak_sustained_active": "issue_active_pct",
    "smsp__thread_inst_executed_per_inst_executed.ratio": "threads_per_inst",
    "lts__throughput.avg.pct_of_peak_sustained_elapsed": "lts_pct_of_peak",
    "l1tex__throughput.avg.pct_of_peak_sustained_elapsed": "l1tex_pct_of_peak",
    "launch__grid_size": "grid",
    "launch__block_size": "block",
}
SCALE = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "nsecond": 1, "usecond": 1e3,
         "msecond": 1e6, "second": 1e9, "ns": 1, "us": 1e3, "ms": 1e6, "s": 1e9}


def summarise(rep: str, kernel: str):
    # a report, or the raw page already exported to CSV (profiles/r01_ncu_raw_*.csv)
    if rep.endswith(".csv"):
        out = open(rep).read()
    else:
        out = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(out)))
    head, units = rows[0], rows[1]
    res = None
    for r in rows[2:]:
        d = dict(zip(head, r))
        if kernel not in d.get("Kernel Name", ""):
            continue
        res = {"kernel": d["Kernel Name"]}
        for k, name in KEYS.items():
            if k not in d:
                continue
            u = units[head.index(k)]
            try:
                v = float(d[k].replace(",", ""))
            except ValueError:
                continue
            res[name] = v * SCALE.get(u, 1) if u in SCALE else v
        res["duration_ns"] = res.pop("duration", None)
        res["bytes_per_launch"] = res.get("dram_read", 0) + res.get("dram_write", 0)
    return res


if __name__ == "__main__":
    path = os.path.join(ROOT, "profiles", "ncu_traffic.json")
    data = json.load(open(path)) if os.path.exists(path) else {}
    for arg in sys.argv[1:]:
        rep, kernel, work = arg.split(":")
        s = summarise(rep, kernel)
        if s:
            # a raw CSV keeps the name of the report it was exported from
            s["report"] = data.get(work, {}).get("report") if rep.endswith(".csv") else os.path.basename(rep)
            data[work] = s
            print(work, json.dumps(s))
    with open(path, "w") as f:
        json.dump(data, f, indent=1, sort_keys=True)
