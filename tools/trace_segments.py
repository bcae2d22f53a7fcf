"""Per-GR timeline of a phase trace: python tools/trace_segments.py trace.bin
For every GR: its levels (grid / tail), their time and widest frontier; then the
fix+push loops until the next GR: count (grid / tail), time, worklist sizes."""
import sys

import numpy as np

t = np.fromfile(sys.argv[1], dtype=np.int64).reshape(-1, 3)
t = t[t[:, 0] < 100]
segs = []
cur = None
for i in range(1, len(t)):
    tag, sz, te = (int(x) for x in t[i])
    d = (te - t[i - 1][2]) / 1e3
    kind = tag // 2
    if tag == 99:
        continue
    if kind == 1:  # GR level 0 starts a GR segment
        cur = {"lv_g": 0, "lv_c": 0, "t_gr": 0.0, "maxf": 0, "loops_g": 0, "loops_c": 0, "t_loop": 0.0, "wl": []}
        segs.append(cur)
    if cur is None:
        continue
    if kind in (1, 2):
        cur["lv_g" if tag % 2 else "lv_c"] += 1
        cur["t_gr"] += d
        cur["maxf"] = max(cur["maxf"], sz)
    elif kind in (3, 4):
        if kind == 4:
            cur["loops_g" if tag % 2 else "loops_c"] += 1
            cur["wl"].append(sz)
        cur["t_loop"] += d
print(f"{'GR':>3} {'lv grid':>7} {'lv tail':>7} {'ms GR':>7} {'max fr':>8} | {'loops g':>7} {'loops t':>7} {'ms loops':>8} {'wl max':>8} {'wl med':>7}")
for k, s in enumerate(segs):
    wl = s["wl"] or [0]
    print(f"{k:3d} {s['lv_g']:7d} {s['lv_c']:7d} {s['t_gr'] / 1e3:7.3f} {s['maxf']:8d} | {s['loops_g']:7d} {s['loops_c']:7d} "
          f"{s['t_loop'] / 1e3:8.3f} {max(wl):8d} {int(np.median(wl)):7d}")
