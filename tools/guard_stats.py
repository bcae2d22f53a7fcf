"""Repeated solves; prints guard re-activations and cardinality per run (GPU box)."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import synth  # noqa: E402
import paper_conf_icpp_devecikuc13_b200 as pkg  # noqa: E402

name = sys.argv[1]
reps = int(sys.argv[2]) if len(sys.argv) > 2 else 5
opts = {}
if len(sys.argv) > 3:
    for kv in sys.argv[3].split(","):
        k, v = kv.split("=")
        opts[k] = float(v) if "." in v else int(v)
g = synth.config(name, float(os.environ.get("SCALE", "1")))
ip = torch.from_numpy(g.indptr).cuda()
ix = torch.from_numpy(g.indices).cuda()
mt = pkg.Matcher(ip, ix, g.m, g.n, **opts)
for r in range(reps):
    card, _, _ = mt.solve()
    st = mt.stats()
    print(name, opts, r, card, "guard", st["guard_reactivated"], "loops", st["loops"], "blocked", st["blocked"],
          "dead", st["dead"], "ms", round(st["ms_total"], 2), flush=True)
