"""mcm_create timing per config (GPU box): python tools/time_create.py C4"""
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import synth  # noqa: E402
import paper_conf_icpp_devecikuc13_b200 as pkg  # noqa: E402

for name in sys.argv[1:]:
    g = synth.config(name)
    ip = torch.from_numpy(g.indptr).cuda()
    ix = torch.from_numpy(g.indices).cuda()
    for r in range(4):
        torch.cuda.synchronize()
        t = time.perf_counter()
        mt = pkg.Matcher(ip, ix, g.m, g.n)
        torch.cuda.synchronize()
        dt = (time.perf_counter() - t) * 1e3
        st = mt.stats()
        mt.close()
    print(name, "create ms (wall, last of 4)", round(dt, 3), flush=True)
