#!/bin/bash
# A/B of the windowed GR (option gr_window, DESIGN R29): interleaved rounds of
# median solve times on C2-C5 (tools/ab_solve.py)
O=gpurun_out/${TAG:-r02d}_window_ab.txt
: > $O
for round in 1 2; do
  for c in C2 C3 C4 C5; do
    for w in ${WINDOWS:-0 2 4 8}; do
      for wm in ${WMAX:-16384}; do
        timeout 300 python tools/ab_solve.py $c ${REPS:-15} "w=$w,max=$wm" gr_window=$w,gr_window_max=$wm >> $O 2>&1
      done
    done
  done
done
