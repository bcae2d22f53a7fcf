"""Load imbalance per grid phase (GPU box):
    MCM_TRACE=20000 MCM_TRACE_FILE=t.bin MCM_CTATIME=4000 MCM_CTATIME_FILE=c.bin \\
        python tools/cta_imbalance.py C4 [opts]
Runs one solve (after a warm-up) and splits every grid phase into: work (phase
start -> the median CTA's arrival at the closing barrier), imbalance (median -> last
CTA's arrival) and barrier (last arrival -> release), summed per phase tag."""
import collections
import os
import sys

import numpy as np

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import synth  # noqa: E402
import paper_conf_icpp_devecikuc13_b200 as pkg  # noqa: E402

TAGS = {1: "gr_level0", 2: "gr_level", 3: "fix", 4: "push", 5: "gr_window", 0: "other"}
name = sys.argv[1]
opts = dict(kv.split("=") for kv in sys.argv[2].split(",")) if len(sys.argv) > 2 else {}
opts = {k: (float(v) if "." in v else int(v)) for k, v in opts.items()}
g = synth.config(name)
mt = pkg.Matcher(torch.from_numpy(g.indptr).cuda(), torch.from_numpy(g.indices).cuda(), g.m, g.n, **opts)
mt.solve()
mt.solve()
t = np.fromfile(os.environ["MCM_TRACE_FILE"], dtype=np.int64).reshape(-1, 3)
t = t[t[:, 0] < 100]  # one record per barrier, in phase order (ph = record index)
c = np.fromfile(os.environ["MCM_CTATIME_FILE"], dtype=np.int64)
nph, grid = int(c[0]), int(c[1])
a = c[2:].reshape(nph, grid)
acc = collections.defaultdict(lambda: np.zeros(4))
for ph in range(1, min(nph, len(t))):
    row = a[ph]
    if (row == 0).any() or t[ph, 0] % 2 == 0:  # not a grid barrier (tail phases) or not recorded
        continue
    start, end = t[ph - 1, 2], t[ph, 2]
    med, mx = np.median(row), row.max()
    key = TAGS.get(t[ph, 0] // 2, str(t[ph, 0] // 2))
    acc[key] += np.array([1, med - start, mx - med, end - mx]) / np.array([1, 1e3, 1e3, 1e3])
print(f"{name} {opts}: per grid phase tag -- phases, work / imbalance / barrier (ms, summed)")
for k, v in sorted(acc.items(), key=lambda kv: -kv[1][1:].sum()):
    print(f"  {k:10s} n={int(v[0]):5d} work={v[1] / 1e3:7.3f} imbalance={v[2] / 1e3:7.3f} barrier={v[3] / 1e3:7.3f}")
