#!/bin/bash
# option sweep on the headline config (C4) and the others: median solve ms (tools/ab_solve.py)
O=gpurun_out/${TAG:-r02k}_sweep.txt
: > $O
for c in ${CONFIGS:-C4}; do
  for o in ${OPTS:-k=0.4 k=0.2 k=0.7 k=1.0 k=1.5 k=0.4,gr_target=0.4 k=0.4,gr_target=0.3 k=0.7,gr_target=0.4 k=0.4,gr_target=0.8}; do
    timeout 300 python tools/ab_solve.py $c ${REPS:-10} "$o" $o >> $O 2>&1
  done
done
