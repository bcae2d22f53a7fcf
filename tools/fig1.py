"""Fig. 1 ablation of the paper on the synthetic configs:
G-PR-First (Alg. 3/6) / G-PR-NoShr / G-PR-Shr  x  GR strategy (adaptive k = 0.3,
0.7, 1, 1.5, 2; fixed 10, 50).  Geometric mean of the solve time (ms, best of
REPS) over the configs; GPU box.

    python tools/fig1.py [paper|build] C1 C2 C3 C5 > profiles/r01_fig1.md
paper: the paper's complete GR and post-GR-only shrink (gr_early=0, compact_adapt=0)
build: the build's defaults (early-stop GR, adaptive compaction, tail group)
"""
import math
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import synth  # noqa: E402
import paper_conf_icpp_devecikuc13_b200 as pkg  # noqa: E402

VARIANTS = [("G-PR-First", dict(variant=1)), ("G-PR-NoShr", dict(shrink_min=-1)), ("G-PR-Shr", dict())]
STRATS = [("adaptive 0.3", dict(k=0.3)), ("adaptive 0.7", dict(k=0.7)), ("adaptive 1", dict(k=1.0)),
          ("adaptive 1.5", dict(k=1.5)), ("adaptive 2", dict(k=2.0)), ("fix 10", dict(gr_strategy="fixed", k=10)),
          ("fix 50", dict(gr_strategy="fixed", k=50))]


def main():
    mode = sys.argv[1]
    cfgs = sys.argv[2:] or ["C1", "C2", "C3", "C5"]
    base = dict(gr_early=0, compact_adapt=0, tail_chain=0, grid_chain=0) if mode == "paper" else {}
    reps = int(os.environ.get("REPS", "3"))
    graphs = []
    for c in cfgs:
        g = synth.config(c)
        graphs.append((c, g, torch.from_numpy(g.indptr).cuda(), torch.from_numpy(g.indices).cuda()))
    res = {}
    for vn, vo in VARIANTS:
        for sn, so in STRATS:
            times = []
            for c, g, ip, ix in graphs:
                mt = pkg.Matcher(ip, ix, g.m, g.n, **{**base, **vo, **so})
                best = 1e30
                for _ in range(reps):
                    torch.cuda.synchronize()
                    t = time.perf_counter()
                    card, _, _ = mt.solve()
                    best = min(best, (time.perf_counter() - t) * 1e3)
                mt.close()
                times.append(best)
            res[(vn, sn)] = math.exp(sum(math.log(t) for t in times) / len(times))
            print(f"<!-- {vn} {sn}: {[round(t, 3) for t in times]} -->", flush=True)
    print(f"# Fig. 1 ablation on B200 ({mode} configuration), geometric mean of solve ms over {', '.join(cfgs)}\n")
    print("| variant | " + " | ".join(s for s, _ in STRATS) + " |")
    print("|---|" + "---|" * len(STRATS))
    for vn, _ in VARIANTS:
        print(f"| {vn} | " + " | ".join(f"{res[(vn, s)]:.2f}" for s, _ in STRATS) + " |")


if __name__ == "__main__":
    main()
