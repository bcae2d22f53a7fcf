"""Phase trace of one solve (GPU box): MCM_TRACE=N MCM_TRACE_FILE=f python tools/trace_solve.py C2 [opts]
then summarise durations per phase tag and size bucket."""
import os
import sys

import numpy as np

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

import synth  # noqa: E402
import paper_conf_icpp_devecikuc13_b200 as pkg  # noqa: E402

TAGS = {1: "gr_level0", 2: "gr_level", 3: "fix", 4: "push", 5: "gr_window", 0: "other"}


def summarize(path):
    t = np.fromfile(path, dtype=np.int64).reshape(-1, 3)
    for tag, what in ((150, "window: most local rounds of a CTA"), (151, "window: rows expanded inside"),
                      (152, "window: dirty"), (160, "grid chain phase: longest chain (pushes)")):
        x = t[t[:, 0] == tag, 1]
        if x.size:
            print(f"{what}: n={x.size} mean={x.mean():.2f} p50={np.median(x):.0f} max={x.max()}")
    d = np.diff(t[:, 2]) / 1e3  # us; phase i ends at record i+1? record i = end of phase with tag t[i]
    keep = t[:, 0] < 100  # drop intra-phase marks from the per-phase summary
    t = t[keep]
    d = np.diff(t[:, 2]) / 1e3
    tags, sizes = t[1:, 0], t[1:, 1]
    dur = d
    print(f"{len(t)} records, total {(t[-1, 2] - t[0, 2]) / 1e6:.3f} ms")
    for tag in sorted(set(tags.tolist())):
        sel = tags == tag
        name = "tail_wait" if tag == 99 else TAGS.get(tag // 2, str(tag // 2)) + ("/grid" if tag % 2 else "/cta")
        ds, ss = dur[sel], sizes[sel]
        print(f"{name:16s} n={sel.sum():6d} total={ds.sum() / 1e3:8.3f} ms mean={ds.mean():7.2f} us "
              f"p50={np.median(ds):7.2f} p90={np.percentile(ds, 90):7.2f} max={ds.max():8.1f} | size p50={np.median(ss):.0f} "
              f"max={ss.max()}")
        if tag != 99:
            for lo, hi in [(0, 32), (32, 512), (512, 4096), (4096, 1 << 30)]:
                b = sel & (sizes >= lo) & (sizes < hi)
                if b.sum():
                    print(f"    size [{lo},{hi}) n={b.sum():6d} mean={dur[b].mean():7.2f} us p50={np.median(dur[b]):7.2f}")


def main():
    name = sys.argv[1]
    opts = {}
    if len(sys.argv) > 2:
        for kv in sys.argv[2].split(","):
            k, v = kv.split("=")
            opts[k] = float(v) if "." in v else int(v)
    g = synth.config(name)
    ip = torch.from_numpy(g.indptr).cuda()
    ix = torch.from_numpy(g.indices).cuda()
    mt = pkg.Matcher(ip, ix, g.m, g.n, **opts)
    card, _, _ = mt.solve()
    card, _, _ = mt.solve()
    print(name, opts, card, {k: v for k, v in mt.stats().items() if k in ("loops", "tail_loops", "gr_levels", "ms_total")})
    summarize(os.environ["MCM_TRACE_FILE"])


if __name__ == "__main__":
    main()
