"""Run-to-run spread of a parallel solve (GPU box): the same graph solved REPS times
from the device greedy M0 (default) and from one fixed host M0 (init=given,
column-order first-free greedy computed here), to see whether the spread of loops /
time comes from the initial matching or from the push-loop races.

    python tools/variance.py C2 [reps]
"""
import os
import statistics
import sys

import numpy as np

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import synth  # noqa: E402
import paper_conf_icpp_devecikuc13_b200 as pkg  # noqa: E402


def host_greedy(g):
    # column-order, first free row of Gamma(v) (CSC from the CSR)
    order = np.argsort(g.indices, kind="stable")
    rows = np.repeat(np.arange(g.m, dtype=np.int64), np.diff(g.indptr))[order]
    cptr = np.zeros(g.n + 1, np.int64)
    np.add.at(cptr, g.indices.astype(np.int64) + 1, 1)
    cptr = np.cumsum(cptr)
    rm = np.full(g.m, -1, np.int32)
    cm = np.full(g.n, -1, np.int32)
    for v in range(g.n):
        for u in rows[cptr[v]:cptr[v + 1]]:
            if rm[u] < 0:
                rm[u] = v
                cm[v] = u
                break
    return rm, cm


def main():
    name = sys.argv[1]
    reps = int(sys.argv[2]) if len(sys.argv) > 2 else 15
    g = synth.config(name)
    ip = torch.from_numpy(g.indptr).cuda()
    ix = torch.from_numpy(g.indices).cuda()
    rm0, cm0 = host_greedy(g)
    for label, opts in (("device greedy", {}), ("fixed host M0", {"init": "given"})):
        mt = pkg.Matcher(ip, ix, g.m, g.n, **opts)
        ts, loops, levels, inits = [], [], [], []
        for _ in range(reps + 1):
            rm = torch.from_numpy(rm0).cuda()
            cm = torch.from_numpy(cm0).cuda()
            card, _, _ = mt.solve(rm, cm)
            st = mt.stats()
            ts.append(st["ms_total"]); loops.append(st["loops"]); levels.append(st["gr_levels"])
            inits.append(st["init_card"])
        ts, loops, levels = ts[1:], loops[1:], levels[1:]
        print(f"{name} {label:14s} card={card} init={inits[-1]} ms med={statistics.median(ts):.2f} "
              f"min={min(ts):.2f} max={max(ts):.2f} loops med={statistics.median(loops)} range={min(loops)}-{max(loops)} "
              f"levels med={statistics.median(levels)}")
        mt.close()


if __name__ == "__main__":
    main()
