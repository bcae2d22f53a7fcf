"""Grid push-chain phases of a traced solve (run after tools/trace_solve.py with
MCM_TRACE_FILE=f): phase time, longest chain, slots, us per push of the longest
chain.  python tools/chain_phases.py f"""
import sys

import numpy as np

t = np.fromfile(sys.argv[1], dtype=np.int64).reshape(-1, 3)
for i in np.nonzero(t[:, 0] == 160)[0]:
    j = i - 1
    while t[j, 0] >= 100:
        j -= 1
    k = j - 1
    while t[k, 0] >= 100:
        k -= 1
    us = (t[j, 2] - t[k, 2]) / 1e3
    print(f"chain phase {us:7.1f} us  longest {t[i, 1]:4d}  slots {t[j, 1]:6d}  "
          f"{us / max(1, t[i, 1]):5.2f} us/push")
