"""Full-size stress of the production kernel (-m gpu): repeated solves of C2 and C4
(the racy parallel trajectory differs run to run), each checked for
the cardinality (closed form / oracle), validity and -- on a subset -- the Konig
certificate; plus solves with the debug consistency checks (MCM_DEBUG=1: after
every fix and push phase, every matched row's column points back and no column
sits twice in the worklist).  Exactness-guard re-activations and repaired rows
are summed and reported (gpurun_out/stress_stats.json when that directory exists),
so a guard that had to fire is never silent."""
import json
import os

import numpy as np
import pytest

import oracle
import synth

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu

import paper_conf_icpp_devecikuc13_b200 as pkg  # noqa: E402

OUT = os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))), "gpurun_out")


def _report(name, rec):
    if os.path.isdir(OUT):
        p = os.path.join(OUT, "stress_stats.json")
        d = json.load(open(p)) if os.path.exists(p) else {}
        d[name] = rec
        json.dump(d, open(p, "w"), indent=1)


@pytest.mark.parametrize("name,reps,konig_every", [("C2", 50, 5), ("C4", 50, 25)])
def test_repeated_full_size_solves(name, reps, konig_every):
    g = synth.config(name)
    mm = g.mm if g.mm is not None else oracle.hopcroft_karp(g)[0]
    ip = torch.from_numpy(g.indptr).cuda()
    ix = torch.from_numpy(g.indices).cuda()
    mt = pkg.Matcher(ip, ix, g.m, g.n)
    guard = repaired = 0
    ms = []
    for r in range(reps):
        card, rm, cm = mt.solve()
        st = mt.stats()
        assert card == mm, (name, r, card, mm, st)
        rm, cm = rm.cpu().numpy(), cm.cpu().numpy()
        assert oracle.check_matching(g, rm, cm) == mm, (name, r)
        if r % konig_every == 0:
            assert oracle.konig_cover(g, rm, cm)[0] == mm, (name, r)
        guard += st["guard_reactivated"]
        repaired += st["rows_repaired"]
        ms.append(st["ms_total"])
    mt.close()
    _report(name, dict(solves=reps, guard_reactivated=guard, rows_repaired=repaired,
                       ms_median=float(np.median(ms)), ms_max=float(max(ms))))


@pytest.mark.parametrize("name", ["C2", "C4"])
def test_debug_consistency_checks(name, monkeypatch):
    monkeypatch.setenv("MCM_DEBUG", "1")
    g = synth.config(name)
    mm = g.mm if g.mm is not None else oracle.hopcroft_karp(g)[0]
    mt = pkg.Matcher(torch.from_numpy(g.indptr).cuda(), torch.from_numpy(g.indices).cuda(), g.m, g.n)
    viol = guard = 0
    for r in range(5):
        card, rm, cm = mt.solve()
        st = mt.stats()
        assert card == mm
        viol += st["debug_violations"]
        guard += st["guard_reactivated"]
    mt.close()
    _report(name + "_debug", dict(solves=5, debug_violations=viol, guard_reactivated=guard))
    assert viol == 0, (name, viol)
