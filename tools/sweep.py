"""Option sweep on one config (GPU box): prints solve time and counters per option set.

    python tools/sweep.py C2 tail_max=0 tail_max=512 k=0.3 ...
Each argument is a comma-separated option set (key=value[,key=value]); 'default' = defaults.
"""
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import synth  # noqa: E402
import paper_conf_icpp_devecikuc13_b200 as pkg  # noqa: E402


def parse(s):
    if s == "default":
        return {}
    out = {}
    for kv in s.split(","):
        k, v = kv.split("=")
        try:
            v = int(v)
        except ValueError:
            try:
                v = float(v)
            except ValueError:
                pass
        out[k] = v
    return out


def main():
    name = sys.argv[1]
    scale = float(os.environ.get("SCALE", "1"))
    g = synth.config(name, scale)
    ip = torch.from_numpy(g.indptr).cuda()
    ix = torch.from_numpy(g.indices).cuda()
    reps = int(os.environ.get("REPS", "3"))
    for spec in sys.argv[2:] or ["default"]:
        opts = parse(spec)
        mt = pkg.Matcher(ip, ix, g.m, g.n, **opts)
        ts, dev = [], []
        for r in range(reps):
            torch.cuda.synchronize()
            t0 = time.perf_counter()
            card, _, _ = mt.solve()
            ts.append((time.perf_counter() - t0) * 1e3)
            dev.append(mt.stats()["ms_total"])
        st = mt.stats()
        dev.sort()
        mt.close()
        keys = ["loops", "tail_loops", "gr_count", "gr_levels", "pushes", "blocked", "edges_scanned", "slots",
                "grid_barriers", "ms_init", "ms_gr", "ms_loop", "ms_total"]
        print(f"{name} {spec:30s} card={card} dev_ms_med={dev[len(dev) // 2]:8.3f} min={dev[0]:8.3f} wall_ms={min(ts):8.3f} " +
              " ".join(f"{k}={st[k]:.3f}" if isinstance(st[k], float) else f"{k}={st[k]}" for k in keys), flush=True)


if __name__ == "__main__":
    main()
