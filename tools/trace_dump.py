"""Dump a phase trace as a sequence: python tools/trace_dump.py trace.bin [start] [count]"""
import sys

import numpy as np

TAGS = {1: "L0", 2: "LV", 3: "FX", 4: "PU", 0: "--"}
t = np.fromfile(sys.argv[1], dtype=np.int64).reshape(-1, 3)
s = int(sys.argv[2]) if len(sys.argv) > 2 else 0
c = int(sys.argv[3]) if len(sys.argv) > 3 else 200
for i in range(max(1, s), min(len(t), s + c)):
    tag, sz, te = t[i]
    name = "WAIT" if tag == 99 else (f"M{tag}" if tag >= 100 else TAGS.get(int(tag) // 2, "?") + ("g" if tag % 2 else "c"))
    print(f"{i:6d} {name:5s} {sz:8d} {(te - t[i - 1][2]) / 1e3:8.2f}")
