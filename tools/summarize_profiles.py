"""Summarise gpurun_out/ ncu artefacts into profiles/ (run here, no GPU needed).

    python tools/summarize_profiles.py <round-tag>
Reads gpurun_out/launches_C2.csv (launch list of the bench command) and
gpurun_out/prof_<cfg>.ncu-rep (one `ncu --set full` capture of the solve kernel)
and writes profiles/<tag>_launches_C2.md, profiles/<tag>_ncu_<cfg>.md and
profiles/ncu_traffic_<cfg>.json (read by bench.py for roofline.traffic).
"""
import csv
import glob
import io
import json
import os
import subprocess
import sys
from collections import defaultdict

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
OUT = os.path.join(ROOT, "gpurun_out")
PROF = os.path.join(ROOT, "profiles")
SCALE = {"nsecond": 1e-3, "ns": 1e-3, "usecond": 1.0, "us": 1.0, "msecond": 1e3, "ms": 1e3, "second": 1e6, "s": 1e6}
METRICS = [
    "gpu__time_duration.sum", "dram__bytes_read.sum", "dram__bytes_write.sum", "gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed",
    "lts__t_bytes.sum", "sm__warps_active.avg.pct_of_peak_sustained_active", "sm__throughput.avg.pct_of_peak_sustained_elapsed",
    "smsp__thread_inst_executed_per_inst_executed.ratio", "launch__registers_per_thread", "launch__grid_size",
    "launch__block_size", "l1tex__t_sectors_pipe_lsu_mem_global_op_ld.sum", "l1tex__t_requests_pipe_lsu_mem_global_op_ld.sum",
    "smsp__inst_executed.sum", "sm__cycles_elapsed.avg.per_second",
]


def launches(tag):
    for path in sorted(glob.glob(os.path.join(OUT, "launches_*.csv"))):
        launches_one(tag, path, os.path.basename(path)[9:-4])


def launches_one(tag, path, cfg):
    lines = [ln for ln in open(path) if not ln.startswith("==")]
    rows = list(csv.DictReader(io.StringIO("".join(lines))))
    agg = defaultdict(lambda: [0, 0.0])
    for r in rows:
        if r.get("Metric Name") != "gpu__time_duration.sum":
            continue
        us = float(r["Metric Value"].replace(",", "")) * SCALE.get(r["Metric Unit"], 1.0)
        agg[r["Kernel Name"]][0] += 1
        agg[r["Kernel Name"]][1] += us
    tot = sum(v[1] for v in agg.values())
    with open(os.path.join(PROF, f"{tag}_launches_{cfg}.md"), "w") as f:
        f.write(f"# {tag}: ncu launch list of `python bench.py --config {cfg} --steps 2 --warmup 3 --no-cpu-baseline`\n\n")
        f.write("`ncu --metrics gpu__time_duration.sum --clock-control none -c 400` -- cold-cache, serialised "
                "per-launch times: compare SHARES, not absolutes.\n\n")
        f.write("| kernel | launches | total us | mean us | share |\n|---|---|---|---|---|\n")
        for k, (c, t) in sorted(agg.items(), key=lambda x: -x[1][1]):
            f.write(f"| `{k[:90]}` | {c} | {t:.1f} | {t / c:.1f} | {100 * t / tot:.2f}% |\n")
    print("wrote launches summary")


def ncu_full(tag):
    for rep in sorted(glob.glob(os.path.join(OUT, "prof_*.ncu-rep"))):
        cfg = os.path.basename(rep)[5:-8]
        raw = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
        rows = list(csv.reader(io.StringIO(raw)))
        if len(rows) < 3:
            continue
        hdr, units, vals = rows[0], rows[1], rows[2]
        d = {h: (v, u) for h, u, v in zip(hdr, units, vals)}
        with open(os.path.join(PROF, f"{tag}_ncu_{cfg}.md"), "w") as f:
            f.write(f"# {tag}: `ncu --set full` of one `gpr_kernel` launch ({cfg}, `tools/one_solve.py {cfg}`)\n\n")
            f.write("| metric | value | unit |\n|---|---|---|\n")
            for mname in METRICS:
                if mname in d:
                    f.write(f"| {mname} | {d[mname][0]} | {d[mname][1]} |\n")
        def val(name):
            v, u = d[name]
            x = float(v.replace(",", ""))
            return x * {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9}.get(u, 1)
        tr = val("dram__bytes_read.sum") + val("dram__bytes_write.sum")
        json.dump({"config": cfg, "dram_bytes_per_launch": tr, "source": f"profiles/{tag}_ncu_{cfg}.md",
                   "kernel": "gpr_kernel"}, open(os.path.join(PROF, f"ncu_traffic_{cfg}.json"), "w"), indent=1)
        print("wrote", cfg, tr / 1e9, "GB")


if __name__ == "__main__":
    tag = sys.argv[1] if len(sys.argv) > 1 else "r01"
    os.makedirs(PROF, exist_ok=True)
    launches(tag)
    ncu_full(tag)
