"""One create + (warmup) solves of a config, for ncu captures: python tools/one_solve.py C2 [reps] [opt=val,...]"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import synth  # noqa: E402
import paper_conf_icpp_devecikuc13_b200 as pkg  # noqa: E402

name = sys.argv[1]
reps = int(sys.argv[2]) if len(sys.argv) > 2 else 2
opts = {}
if len(sys.argv) > 3:
    for kv in sys.argv[3].split(","):
        k, v = kv.split("=")
        opts[k] = float(v) if "." in v else int(v)
g = synth.config(name)
ip = torch.from_numpy(g.indptr).cuda()
ix = torch.from_numpy(g.indices).cuda()
mt = pkg.Matcher(ip, ix, g.m, g.n, **opts)
for _ in range(reps):
    card, _, _ = mt.solve()
print(name, card, mt.stats())
