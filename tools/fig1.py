"""Fig. 1 ablation of the paper on the synthetic configs:
G-PR-First (Alg. 3/6) / G-PR-NoShr / G-PR-Shr  x  GR strategy (adaptive k = 0.3,
0.7, 1, 1.5, 2; fixed 10, 50).  Per cell and config: median of REPS solve times
(CUDA events on the solve stream, L2 flushed before each); every solve's
cardinality is asserted against the config's maximum (closed form, else the
oracle's value stored in tests/golden/configs.json by tools/make_golden.py);
table = geometric mean over the configs.  GPU box.

    python tools/fig1.py [paper|build] C2 C3 C4 > profiles/r02_fig1_paper.md
paper: the paper's G-PR -- complete GR, post-GR-only shrink, one push per column
       per loop (gr_early=0, compact_adapt=0, tail_chain=0, grid_chain=0)
build: the build's defaults (early-stop GR, adaptive compaction, push chains, tail)
"""
import json
import math
import os
import statistics
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch  # noqa: E402

import synth  # noqa: E402
import paper_conf_icpp_devecikuc13_b200 as pkg  # noqa: E402

VARIANTS = [("G-PR-First", dict(variant=1)), ("G-PR-NoShr", dict(shrink_min=-1)), ("G-PR-Shr", dict())]
STRATS = [("adaptive 0.3", dict(k=0.3)), ("adaptive 0.7", dict(k=0.7)), ("adaptive 1", dict(k=1.0)),
          ("adaptive 1.5", dict(k=1.5)), ("adaptive 2", dict(k=2.0)), ("fix 10", dict(gr_strategy="fixed", k=10)),
          ("fix 50", dict(gr_strategy="fixed", k=50))]


def expected_mm(name, g):
    if g.mm is not None:
        return g.mm
    gold = json.load(open(os.path.join(ROOT, "tests", "golden", "configs.json")))["cases"]
    for c in gold:
        if c["name"] == name and c["scale"] == 1.0 and c["digest"] == g.digest():
            return c["mm"]
    raise KeyError(f"no golden MM for {name}")


def main():
    mode = sys.argv[1]
    cfgs = sys.argv[2:] or ["C2", "C3", "C4"]
    base = dict(gr_early=0, compact_adapt=0, tail_chain=0, grid_chain=0) if mode == "paper" else {}
    reps = int(os.environ.get("REPS", "3"))
    flush = torch.empty(512 << 20, dtype=torch.uint8, device="cuda")
    graphs = []
    for c in cfgs:
        g = synth.config(c)
        graphs.append((c, g, torch.from_numpy(g.indptr).cuda(), torch.from_numpy(g.indices).cuda(), expected_mm(c, g)))
    res, per = {}, {}
    for vn, vo in VARIANTS:
        for sn, so in STRATS:
            times = []
            for c, g, ip, ix, mm in graphs:
                mt = pkg.Matcher(ip, ix, g.m, g.n, **{**base, **vo, **so})
                ts = []
                for r in range(reps + 1):
                    flush.fill_(r & 0xFF)
                    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                    a.record()
                    card, _, _ = mt.solve()
                    b.record()
                    b.synchronize()
                    if card != mm:
                        raise RuntimeError(f"{vn} {sn} {c}: cardinality {card} != {mm}")
                    if r:
                        ts.append(a.elapsed_time(b))
                mt.close()
                times.append(statistics.median(ts))
            res[(vn, sn)] = math.exp(sum(math.log(t) for t in times) / len(times))
            per[(vn, sn)] = times
            print(f"<!-- {vn} {sn}: {[round(t, 3) for t in times]} -->", flush=True)
    print(f"# Fig. 1 ablation on B200 ({mode} configuration): geometric mean over {', '.join(cfgs)} of the median "
          f"solve ms ({reps} solves per cell, CUDA events, L2 flushed; every cardinality = the config's maximum)\n")
    print("| variant | " + " | ".join(s for s, _ in STRATS) + " |")
    print("|---|" + "---|" * len(STRATS))
    for vn, _ in VARIANTS:
        print(f"| {vn} | " + " | ".join(f"{res[(vn, s)]:.2f}" for s, _ in STRATS) + " |")
    for i, (c, *_rest) in enumerate(graphs):
        print(f"\n{c} (ms):\n")
        print("| variant | " + " | ".join(s for s, _ in STRATS) + " |")
        print("|---|" + "---|" * len(STRATS))
        for vn, _ in VARIANTS:
            print(f"| {vn} | " + " | ".join(f"{per[(vn, s)][i]:.2f}" for s, _ in STRATS) + " |")


if __name__ == "__main__":
    main()
