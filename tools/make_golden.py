"""Write tests/golden/configs.json: CSR digests of the seeded configs at test
scales plus the oracle's maximum cardinality (PR-FIFO == Hopcroft-Karp), and the
closed-form MM where the recipe fixes it.  Calls only synth/ and oracle/."""
import json
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import oracle  # noqa: E402
import synth  # noqa: E402

CASES = [("C1", 1.0), ("C1", 0.1), ("C2", 0.01), ("C2", 0.1), ("C3", 0.001), ("C3", 0.01), ("C4", 1 / 1024),
         ("C4", 1 / 64), ("C5", 1 / 256), ("C5", 1 / 16), ("C2", 1.0), ("C3", 1.0), ("C4", 1.0), ("C5", 1.0)]


def main():
    out = {"_doc": __doc__, "cases": []}
    for name, scale in CASES:
        g = synth.config(name, scale)
        c1, _, _, _ = oracle.pr_fifo(g)
        c2, _, _ = oracle.hopcroft_karp(g)
        assert c1 == c2, (name, scale, c1, c2)
        if g.mm is not None:
            assert c1 == g.mm
        m0 = oracle.cheap_match(g)[0]
        out["cases"].append(dict(name=name, scale=scale, m=g.m, n=g.n, nnz=g.nnz, digest=g.digest(), mm=c1,
                                 closed_form_mm=g.mm, cheap_match=m0))
        print(out["cases"][-1], flush=True)
    path = os.path.join(ROOT, "tests", "golden", "configs.json")
    with open(path, "w") as f:
        json.dump(out, f, indent=1)


if __name__ == "__main__":
    main()
