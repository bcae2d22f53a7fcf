"""Repeat small solves and report any invalid matching in detail (GPU box):

    python tests/race_repro.py [reps] [graph] [opt=val,...]
    compute-sanitizer --tool racecheck python tests/race_repro.py 1 C2

graph: C2 (C2 at scale 0.002, default), C1, hall.  On an invalid result it prints
the check code, the conflicting rows / columns and the solve statistics.
"""
import os
import sys

import numpy as np

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import oracle  # noqa: E402
import synth  # noqa: E402
import paper_conf_icpp_devecikuc13_b200 as pkg  # noqa: E402


def graph(name):
    if name == "C1":
        return synth.config("C1", 0.2)
    if name == "hall":
        return synth.hall_violator(3000, 200, 37, 5)
    return synth.config("C2", 0.002)


def detail(g, rm, cm):
    adj = {u: set(g.indices[g.indptr[u]:g.indptr[u + 1]].tolist()) for u in range(g.m)}
    bad_edge = [u for u in range(g.m) if rm[u] >= 0 and rm[u] not in adj[u]]
    nonmut_r = [u for u in range(g.m) if rm[u] >= 0 and cm[rm[u]] != u]
    nonmut_c = [v for v in range(g.n) if cm[v] >= 0 and rm[cm[v]] != v]
    vals, cnt = np.unique(rm[rm >= 0], return_counts=True)
    dup = vals[cnt > 1].tolist()
    print(f"  non-edges {len(bad_edge)} {bad_edge[:8]}; rows not mutual {len(nonmut_r)} {nonmut_r[:8]}; "
          f"cols not mutual {len(nonmut_c)} {nonmut_c[:8]}; columns held by >1 row {len(dup)} {dup[:8]}")
    for v in dup[:4]:
        rows = np.nonzero(rm == v)[0].tolist()
        print(f"  column {v}: rows {rows}, cmatch {cm[v]}")


def main():
    reps = int(sys.argv[1]) if len(sys.argv) > 1 else 200
    name = sys.argv[2] if len(sys.argv) > 2 else "C2"
    opts = {}
    if len(sys.argv) > 3:
        for kv in sys.argv[3].split(","):
            k, v = kv.split("=")
            opts[k] = float(v) if "." in v else int(v)
    g = graph(name)
    mm = oracle.hopcroft_karp(g)[0]
    ip = torch.from_numpy(g.indptr).cuda()
    ix = torch.from_numpy(g.indices).cuda()
    mt = pkg.Matcher(ip, ix, g.m, g.n, **opts)
    nbad = rep_total = guard_total = 0
    for r in range(reps):
        card, rm, cm = mt.solve()
        torch.cuda.synchronize()
        rm, cm = rm.cpu().numpy(), cm.cpu().numpy()
        code = oracle.check_matching(g, rm, cm)
        st = mt.stats()
        rep_total += st["rows_repaired"]
        guard_total += st["guard_reactivated"]
        if card != mm or code != card:
            nbad += 1
            print(f"rep {r}: card {card} oracle {mm} check {code} stats {mt.stats()}")
            detail(g, rm, cm)
    print(f"{name} opts={opts}: {nbad} bad of {reps}; rows repaired {rep_total}, guard re-activated {guard_total}")


if __name__ == "__main__":
    main()
