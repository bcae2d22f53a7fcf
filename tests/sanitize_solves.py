"""Small solves for compute-sanitizer runs (GPU box):

    compute-sanitizer --tool memcheck python tests/sanitize_solves.py
    compute-sanitizer --tool synccheck python tests/sanitize_solves.py
    compute-sanitizer --tool racecheck python tests/sanitize_solves.py quick

Every solve goes through the C ABI (create, solve, relabel entries, host-buffer
entry) on graphs small enough for the instrumented kernel, covering the grid
phases, the single-CTA tail, the auxiliary kernel instance (serial mode, gap
relabel, G-PR-First) and the CSR validation error path.  The matching of each
solve is checked for validity and against the oracle's cardinality.
"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import oracle  # noqa: E402
import synth  # noqa: E402
import paper_conf_icpp_devecikuc13_b200 as pkg  # noqa: E402


def run(g, **opts):
    ip = torch.from_numpy(g.indptr).cuda()
    ix = torch.from_numpy(g.indices).cuda()
    card, rm, cm = pkg.solve(ip, ix, g.m, g.n, **opts)
    torch.cuda.synchronize()
    mm = oracle.hopcroft_karp(g)[0]
    ok = card == mm and oracle.check_matching(g, rm.cpu().numpy(), cm.cpu().numpy()) == card
    print(f"{g.name:24s} m={g.m:7d} nnz={len(g.indices):8d} opts={opts} card={card} oracle={mm} {'ok' if ok else 'FAIL'}",
          flush=True)
    assert ok


def main():
    quick = len(sys.argv) > 1 and sys.argv[1] == "quick"
    gs = [synth.config("C1", 0.2), synth.hall_violator(3000, 200, 37, 5), synth.config("C2", 0.002)]
    if not quick:
        gs += [synth.config("C3", 0.0005), synth.config("C4", 1 / 1024), synth.config("C5", 1 / 512),
               synth.path(101), synth.complete(40, 70)]
    for g in gs:
        run(g)
    g = synth.config("C1", 0.1)
    run(g, serial=1)
    run(g, gap=1)
    run(g, variant=1)
    run(g, tail_chain=0, grid_chain=0, gr_early=0, compact_adapt=0)
    run(g, gr_concurrent=32)
    # round-2 entry points: the device M0, a GR through the tail, one phase of each kind
    ip, ix = torch.from_numpy(g.indptr).cuda(), torch.from_numpy(g.indices).cuda()
    mt = pkg.Matcher(ip, ix, g.m, g.n, sort_csc=1)
    c0, rm, cm = mt.initial_matching()
    assert oracle.check_matching(g, rm.cpu().numpy(), cm.cpu().numpy()) == c0
    ml, pr, pc, rf = mt.global_relabel(rm, cm)
    INF = g.m + g.n
    for unit in ("fix", "shrink", "push", "fixmatching"):
        for where in ("grid", "tail"):
            st = [rm.clone(), cm.clone(), pr.clone(), pc.clone(), torch.full((g.n,), -1, dtype=torch.int32, device="cuda"),
                  torch.arange(min(g.n, 300), dtype=torch.int32, device="cuda"),
                  torch.full((min(g.n, 300),), -1, dtype=torch.int32, device="cuda")]
            mt.unit_step(unit, where, 3, *st)
    mt.close()
    print("unit / relabel / initial-matching entries ok", c0, ml, INF)
    # host-buffer entry
    g = synth.config("C5", 1 / 1024, index=1)
    card, rm, cm, _ = pkg.match_host(torch.from_numpy(g.indptr).pin_memory(), torch.from_numpy(g.indices).pin_memory(),
                                     g.m, g.n)
    assert card == oracle.hopcroft_karp(g)[0]
    print("match_host ok", card)
    # error path: an out-of-range column index is rejected by the CSR validation
    bad = synth.config("C1", 0.01)
    ix = torch.from_numpy(bad.indices.copy())
    ix[3] = bad.n + 5
    try:
        pkg.solve(torch.from_numpy(bad.indptr).cuda(), ix.cuda(), bad.m, bad.n)
        raise SystemExit("invalid CSR accepted")
    except pkg.MCMError as e:
        print("invalid CSR rejected:", str(e)[:80])
    print("sanitize run ok")


if __name__ == "__main__":
    main()
