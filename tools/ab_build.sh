#!/bin/bash
# A/B of the in-tree build against a baseline tree under build_ab/base (its own
# package, binding and libmcm.so): interleaved rounds of median solve times.
#   TAG=<tag> CONFIGS="C2 C4" REPS=15 ROUNDS=2 [OPTS=k=v,...] bash tools/ab_build.sh
O=gpurun_out/${TAG:-ab}_build_ab.txt
: > $O
for round in $(seq ${ROUNDS:-2}); do
  for c in ${CONFIGS:-C2 C3 C4 C5}; do
    timeout 300 python build_ab/base/tools/ab_solve.py $c ${REPS:-15} base ${OPTS:-} >> $O 2>&1
    timeout 300 python tools/ab_solve.py $c ${REPS:-15} new ${OPTS:-} >> $O 2>&1
  done
done
