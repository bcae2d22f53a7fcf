"""mcm_create time per config with CUDA events (GPU box):
    [MCM_TRANSPOSE=scatter] [MCM_LIB=...] python tools/time_create.py C4 [C3 ...]
Median of 8 creates after 2 warm-ups, L2 flushed before each."""
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import synth  # noqa: E402
import paper_conf_icpp_devecikuc13_b200 as pkg  # noqa: E402

label = os.environ.get("MCM_TRANSPOSE", "bucketed")
flush = torch.empty(512 << 20, dtype=torch.uint8, device="cuda")
for name in sys.argv[1:]:
    g = synth.config(name)
    ip = torch.from_numpy(g.indptr).cuda()
    ix = torch.from_numpy(g.indices).cuda()
    ts = []
    for r in range(10):
        flush.fill_(r)
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        mt = pkg.Matcher(ip, ix, g.m, g.n)
        b.record()
        b.synchronize()
        card = mt.solve()[0]
        mt.close()
        if r >= 2:
            ts.append(a.elapsed_time(b))
    print(f"{label:9s} {name} create ms med={statistics.median(ts):.3f} min={min(ts):.3f} card={card}", flush=True)
