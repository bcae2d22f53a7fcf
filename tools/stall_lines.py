"""Warp-stall samples per source line from an ncu SASS source page (run here):
    nvdisasm --print-line-info <cubin> > k.sass   (cubin: cuobjdump -xelf all libmcm.so)
    ncu -i prof.ncu-rep --page source --csv --print-source sass > k.csv
    python tools/stall_lines.py k.sass k.csv paper_conf_icpp_devecikuc13_b200/csrc/solve.cuh [top]"""
import csv, re, sys, collections
sass = open(sys.argv[1]).read().splitlines()
amap = {}
cur = None
for ln in sass:
    m = re.search(r'File "([^"]+)", line (\d+)', ln)
    if m:
        cur = (m.group(1).split('/')[-1], int(m.group(2)))
        continue
    m = re.search(r'/\*([0-9a-f]{4,})\*/', ln)
    if m and cur:
        amap[int(m.group(1), 16)] = cur
rows = list(csv.reader(open(sys.argv[2])))
hdr = rows[1]
ia = hdr.index("Address"); isamp = hdr.index("Warp Stall Sampling (All Samples)")
base0 = int(rows[2][ia], 16)
cols = [i for i, h in enumerate(hdr) if h.startswith("stall_") and "Not Issued" not in h]
agg = collections.defaultdict(lambda: collections.Counter())
tot = 0
for r in rows[2:]:
    try:
        a = int(r[ia], 16) - base0
        s = float(r[isamp] or 0)
    except Exception:
        continue
    key = amap.get(a, ("?", 0))
    agg[key]["all"] += s
    tot += s
    for i in cols:
        try:
            agg[key][hdr[i]] += float(r[i] or 0)
        except ValueError:
            pass
src = open(sys.argv[3]).read().splitlines()
top = sorted(agg.items(), key=lambda x: -x[1]["all"])[:int(sys.argv[4]) if len(sys.argv) > 4 else 40]
for (f, l), c in top:
    br = ", ".join(f"{k[6:]} {100*v/c['all']:.0f}%" for k, v in c.most_common(4) if k != "all" and v > 0)
    txt = src[l - 1].strip()[:70] if f == "solve.cuh" and 0 < l <= len(src) else ""
    print(f"{100*c['all']/tot:5.1f}% {f}:{l:<5} {txt:70s} | {br}")
