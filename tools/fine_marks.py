"""Intra-phase marks of a MCM_FINE=1 build: python tools/fine_marks.py trace.bin
Between two grid BFS level ends (tag 5) the lead thread records marks 106 (ring
counters read), 107 (gr_step entered), 101 (gr_level start, size = frontier),
102 (frontier entry loaded), 103 (expanded), 104 (flushed), 105 (barrier arrival).
Prints the mean microseconds between consecutive marks per frontier-size bucket."""
import collections
import sys

import numpy as np

t = np.fromfile(sys.argv[1], dtype=np.int64).reshape(-1, 3)
ends = np.nonzero(t[:, 0] == 5)[0]
groups = collections.defaultdict(list)
for a, b in zip(ends[:-1], ends[1:]):
    seg = t[a:b + 1]
    tags = tuple(int(x) for x in seg[1:-1, 0])
    if 101 not in tags:
        continue
    size = int(seg[1 + tags.index(101), 1])
    groups[tags].append((size, np.diff(seg[:, 2]) / 1e3))
for tags, rows in sorted(groups.items(), key=lambda kv: -len(kv[1])):
    names = ["5"] + [str(x) for x in tags] + ["5"]
    for lo, hi in [(32, 512), (512, 4096), (4096, 1 << 30)]:
        sel = [d for s, d in rows if lo <= s < hi]
        if len(sel) < 5:
            continue
        m = np.mean(sel, axis=0)
        print(f"[{lo},{hi}) n={len(sel)} total={m.sum():.2f} us | " +
              " ".join(f"{names[i]}>{names[i + 1]}={m[i]:.2f}" for i in range(len(m))))
