"""Median solve time of one config (A/B of build variants via MCM_LIB, or of options; GPU box):
    [MCM_LIB=build_ab/x.so] python tools/ab_solve.py C2 20 [label] [opt=val,...]"""
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import synth  # noqa: E402
import paper_conf_icpp_devecikuc13_b200 as pkg  # noqa: E402

name, reps = sys.argv[1], int(sys.argv[2])
label = sys.argv[3] if len(sys.argv) > 3 else os.environ.get("MCM_LIB", "in-tree")
opts = {}
if len(sys.argv) > 4:
    for kv in sys.argv[4].split(","):
        k, v = kv.split("=")
        opts[k] = float(v) if "." in v else int(v)
g = synth.config(name)
mt = pkg.Matcher(torch.from_numpy(g.indptr).cuda(), torch.from_numpy(g.indices).cuda(), g.m, g.n, **opts)
ts, lv, lp, gr, lm, pu, im = [], [], [], [], [], [], []
for r in range(reps + 1):
    card, _, _ = mt.solve()
    st = mt.stats()
    assert card == st["card"]
    if r:
        ts.append(st["ms_total"]); lv.append(st["gr_levels"]); lp.append(st["loops"]); gr.append(st["ms_gr"])
        lm.append(st["ms_loop"]); pu.append(st["pushes"]); im.append(st["ms_init"])
print(f"{label:10s} {name} card={card} ms med={statistics.median(ts):.2f} mean={statistics.mean(ts):.2f} "
      f"min={min(ts):.2f} max={max(ts):.2f} gr_ms med={statistics.median(gr):.2f} levels med={statistics.median(lv)} "
      f"loops med={statistics.median(lp)} init_ms med={statistics.median(im):.3f} loop_ms med={statistics.median(lm):.2f} us/push(loop) "
      f"{1e3 * sum(lm) / max(1, sum(pu)):.3f}", flush=True)
