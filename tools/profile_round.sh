#!/bin/bash
# Round measurement bundle (GPU box): bench lines for every config, the ncu launch
# list of the default bench command, and one `ncu --set full` capture of the solve
# kernel per config of interest.  Outputs under gpurun_out/ (summaries are copied to
# profiles/ by hand).
set -u
OUT=gpurun_out
mkdir -p $OUT
python bench.py --steps 10 --warmup 3 > $OUT/bench_default.json 2> $OUT/bench_default.err
for c in C1 C3 C4 C5; do
  timeout 600 python bench.py --config $c --steps 5 --warmup 3 --no-cpu-baseline > $OUT/bench_$c.json 2> $OUT/bench_$c.err
done
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file $OUT/launches_C2.csv \
  python bench.py --steps 2 --warmup 3 --no-cpu-baseline > $OUT/ncu_launch_bench.log 2>&1
for c in ${PROFILE_CONFIGS:-C2 C4}; do
  timeout 900 ncu --set full --import-source on --clock-control none -k regex:gpr_kernel -s 1 -c 1 \
    -o $OUT/prof_$c python tools/one_solve.py $c 2 > $OUT/ncu_full_$c.log 2>&1
done
