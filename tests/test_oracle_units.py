"""Pins for the oracle's G-PR kernel functions and hand-worked G-PR trajectories
(CPU tier).

* tests/golden/gpr_hand_trajectories.json: serial G-PR runs (Alg. 7/8/9 + Alg. 4/5,
  P:556-655) and cheap matchings (reading R13) worked by hand -- final
  mu arrays, |M| and every trajectory counter (loops, GRs, levels, pushes, shrinks,
  dead, blocked) -- so or_gpr_serial's trajectory is pinned, not only its result.
* INITKRNL / SHRKRNL / PUSHKRNL / FIXMATCHING on hand-worked states (Alg. 8
  P:598-611, Alg. 9) and relations that hold for
  any input (SHRKRNL = INITKRNL's surviving slots in order; FIXMATCHING output is
  a valid matching when the rows are).
"""
import json
import os

import numpy as np
import pytest

import oracle
import synth

GOLD = json.load(open(os.path.join(os.path.dirname(__file__), "golden", "gpr_hand_trajectories.json")))


def _graph(case):
    rows, cols = [], []
    for u, lst in enumerate(case["rows"]):
        rows += [u] * len(lst)
        cols += lst
    return synth.from_pairs(case["m"], case["n"], np.array(rows, np.int64), np.array(cols, np.int64))


@pytest.mark.parametrize("ci", range(len(GOLD["cases"])), ids=[c["name"][:1] for c in GOLD["cases"]])
def test_hand_worked_trajectory(ci):
    case = GOLD["cases"][ci]
    g = _graph(case)
    o = case["opts"]
    card0, rm0, cm0 = oracle.cheap_match(g)
    assert card0 == case["cheap"]["card"]
    assert rm0.tolist() == case["cheap"]["rmatch"] and cm0.tolist() == case["cheap"]["cmatch"]
    card, rm, cm, st = oracle.gpr_serial(g, k=o["k"], shrink_min=o["shrink_min"], dead_skip=o["dead_skip"],
                                         init=o.get("init", "greedy"))
    assert card == case["final"]["card"]
    assert rm.tolist() == case["final"]["mu_row"] and cm.tolist() == case["final"]["mu_col"]
    assert st == case["stats"], (st, case["stats"])


def test_initkrnl_hand():
    """Alg. 8 by hand (loop 7).  Columns: c0 mu -1 (unmatched), c1 -> r0 <- (matched),
    c2 -> r1 but r1 unmatched (stale: unmatched), c3 -> r2 <- (matched), c4 = -2
    (dead: not active, R1)."""
    mu_row = [1, -1, 3]
    mu_col = [-1, 0, 1, 2, -2]
    Ap = [0, 1, 2, 4, -1]
    Ac = [-1, 3, -1, -1, 2]
    iA = [-1] * 5
    a, Ac2, iA2 = oracle.initkrnl(7, mu_row, mu_col, Ac, Ap, iA)
    # slot 0: rollback c0; 1: c1 matched, keep Ac=c3; 2: rollback c2; 3: c4 dead, Ac -1; 4: Ap -1, Ac c2
    assert Ac2.tolist() == [0, 3, 2, -1, 2]
    assert iA2.tolist() == [7, -1, 7, 7, -1]
    assert a == 4
    n, Ac3, iA3 = oracle.shrkrnl(7, mu_row, mu_col, Ac, Ap, iA)
    assert n == 4 and Ac3.tolist() == [0, 3, 2, 2] and iA3.tolist() == iA2.tolist()


def test_shrkrnl_is_initkrnl_compacted():
    rng = np.random.default_rng(3)
    for t in range(200):
        m, n, ln = int(rng.integers(1, 30)), int(rng.integers(1, 30)), int(rng.integers(0, 60))
        mu_row = rng.integers(-1, n, m)
        mu_col = rng.integers(-2, m, n)
        Ac = rng.integers(-1, n, ln)
        Ap = rng.integers(-1, n, ln)
        iA = rng.integers(-1, 5, n)
        a, A1, I1 = oracle.initkrnl(5, mu_row, mu_col, Ac, Ap, iA)
        b, A2, I2 = oracle.shrkrnl(5, mu_row, mu_col, Ac, Ap, iA)
        assert a == b and A2.tolist() == [x for x in A1.tolist() if x != -1] and np.array_equal(I1, I2)


def test_pushkrnl_hand_single_push_and_blocked():
    """Case C's loop 0 (golden file): slot 0 single push c0 -> r0, slot 1 blocked."""
    g = _graph(GOLD["cases"][2])
    r = oracle.pushkrnl(g, 0, [-1, -1], [-1, -1], [0, 0], [1, 1], [0, 0], [0, 1])
    assert r["mu_row"].tolist() == [0, -1] and r["mu_col"].tolist() == [0, -1]
    assert r["psi_row"].tolist() == [2, 0] and r["psi_col"].tolist() == [1, 1]
    assert r["Ap"].tolist() == [-1, -1] and r["Ac"].tolist() == [0, 1]
    assert (r["pushes"], r["blocked"], r["dead"]) == (1, 1, 0)


def test_pushkrnl_hand_double_push_and_dead():
    # case A, loop 0: c2 -> r2 displaces c1 (double push, Ap(0) = c1)
    g = _graph(GOLD["cases"][0])
    r = oracle.pushkrnl(g, 0, [0, -1, 1], [0, 2, -1], [2, 0, 4], [1, 3, 5], [-1, -1, 0], [2])
    # mu(c1) = r2 stays behind (stale: c1 is the displaced column, Ap(0) = c1)
    assert r["mu_row"].tolist() == [0, -1, 2] and r["mu_col"].tolist() == [0, 2, 2]
    assert r["psi_row"].tolist() == [2, 0, 6] and r["psi_col"].tolist() == [1, 3, 5]
    assert r["Ap"].tolist() == [1] and (r["pushes"], r["blocked"], r["dead"]) == (1, 0, 0)
    # case B: c1's only row has label INF = 5 -> dead (mu = -2, Ac = Ap = -1), with and without R19
    g = _graph(GOLD["cases"][1])
    for ds in (False, True):
        r = oracle.pushkrnl(g, 0, [0, 2], [0, -1, 1], [5, 5], [5, 5, 5], [-1, 0, -1], [1], dead_skip=ds)
        assert r["mu_col"].tolist() == [0, -2, 1] and r["Ac"].tolist() == [-1] and r["Ap"].tolist() == [-1]
        assert (r["pushes"], r["blocked"], r["dead"]) == (0, 0, 1)
    # empty slot: Ap(i) <- -1 (l.23-24)
    r = oracle.pushkrnl(g, 0, [0, 2], [0, -1, 1], [5, 5], [5, 5, 5], [-1, 0, -1], [-1])
    assert r["Ap"].tolist() == [-1] and r["pushes"] + r["blocked"] + r["dead"] == 0


def test_pushkrnl_first_minimum_and_early_exit():
    """R11: the FIRST row with the strictly smallest label wins; the scan stops at
    psi(v)-1.  One column c0 with G(c0) = r0..r4 (CSC order = row order)."""
    g = synth.from_pairs(5, 1, np.arange(5), np.zeros(5, np.int64))
    INF = 6
    # labels 4, 2, 2, 0, 0 and psi(c0) = 9: no early exit -> first minimum r3
    r = oracle.pushkrnl(g, 0, [-1] * 5, [-1], [4, 2, 2, 0, 0], [9], [-1], [0])
    assert r["mu_col"].tolist() == [3] and r["psi_row"].tolist() == [4, 2, 2, 2, 0] and r["psi_col"].tolist() == [1]
    # psi(c0) = 3: r1 (label 2 = psi(v)-1) stops the scan before the lower r3
    r = oracle.pushkrnl(g, 0, [-1] * 5, [-1], [4, 2, 2, 0, 0], [3], [-1], [0])
    assert r["mu_col"].tolist() == [1] and r["psi_row"].tolist() == [4, 4, 2, 0, 0] and r["psi_col"].tolist() == [3]
    # every label INF -> dead
    r = oracle.pushkrnl(g, 0, [-1] * 5, [-1], [INF] * 5, [1], [-1], [0])
    assert r["mu_col"].tolist() == [-2] and r["dead"] == 1


def test_fixmatching_hand_and_validity():
    card, mc = oracle.fixmatching(3, 4, [1, -1, 0], [2, 0, -2, 1])
    assert card == 2 and mc.tolist() == [2, 0, -1, -1]
    # any injective row assignment + noisy columns -> a valid matching (checker)
    rng = np.random.default_rng(5)
    for t in range(50):
        g = synth.random_small(int(rng.integers(2, 40)), int(rng.integers(2, 40)), 0.2, int(rng.integers(1 << 30)))
        c, rm, cm = oracle.hopcroft_karp(g)
        noisy = cm.copy()
        free = noisy == -1
        noisy[free & (rng.random(g.n) < 0.5)] = -2
        card, mc = oracle.fixmatching(g.m, g.n, rm, noisy)
        assert card == c and oracle.check_matching(g, rm, mc) == c
