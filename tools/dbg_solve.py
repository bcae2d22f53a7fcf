"""Debug helper: run a few solves with MCM_DEBUG=1 consistency checks (GPU box)."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import oracle  # noqa: E402
import synth  # noqa: E402
import paper_conf_icpp_devecikuc13_b200 as pkg  # noqa: E402

for g in [synth.config("C1", 0.2), synth.complete(64, 40), synth.config("C1")]:
    ip = torch.from_numpy(g.indptr).cuda()
    ix = torch.from_numpy(g.indices).cuda()
    mt = pkg.Matcher(ip, ix, g.m, g.n, max_loops=5000)
    try:
        card, rm, cm = mt.solve()
        print(g.name, card, oracle.hopcroft_karp(g)[0], mt.stats(), flush=True)
    except Exception as e:  # noqa: BLE001
        print(g.name, "ERR", e, mt.stats(), flush=True)
