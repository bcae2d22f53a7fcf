#!/bin/bash
# Round-2 measurement bundle (GPU box).  TAG=<tag> bash tools/round_r02.sh
#   smoke, GPU tests, bench lines (C4 default; C1/C2/C3/C5, all with cpu_baseline),
#   ncu launch list of the default bench command, one `ncu --set full` capture of
#   the solve kernel on C4 and C2, phase traces, Fig. 1 (paper and build
#   configurations on C2-C4), NEXT-4 partitioned-GR experiment.
#   Skip parts with NOTESTS=1, NOFIG=1, NOPGR=1, NONCU=1.
set -u
O=gpurun_out
T=${TAG:-r02}
mkdir -p $O
python -c "import __graft_entry__ as g; g.smoke()" > $O/${T}_smoke.log 2>&1
[ -z "${NOTESTS:-}" ] && timeout 900 python -m pytest tests -m gpu -q > $O/${T}_gputests.log 2>&1
timeout 900 python bench.py --steps 20 --warmup 3 > $O/${T}_bench_C4.json 2> $O/${T}_bench_C4.err
for c in ${CONFIGS:-C2 C3 C1 C5}; do
  timeout 900 python bench.py --config $c --steps 10 --warmup 3 > $O/${T}_bench_$c.json 2> $O/${T}_bench_$c.err
done
if [ -z "${NONCU:-}" ]; then
  timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file $O/launches_C4.csv \
    python bench.py --steps 2 --warmup 3 --no-cpu-baseline > $O/${T}_ncu_launch_bench.log 2>&1
  for c in ${PROFILE_CONFIGS:-C4 C2}; do
    timeout 900 ncu --set full --import-source on --clock-control none -k regex:gpr_kernel -s 1 -c 1 \
      -o $O/prof_$c -f python tools/one_solve.py $c 2 > $O/${T}_ncu_full_$c.log 2>&1
  done
fi
for c in C2 C4 C3; do
  MCM_TRACE=20000 MCM_TRACE_FILE=$O/trace_$c.bin timeout 300 python tools/trace_solve.py $c > $O/${T}_trace_$c.txt 2>&1
done
if [ -z "${NOFIG:-}" ]; then
  timeout 1200 python tools/fig1.py paper C2 C3 C4 > $O/${T}_fig1_paper.md 2> $O/${T}_fig1_paper.err
  timeout 1200 python tools/fig1.py build C2 C3 C4 > $O/${T}_fig1_build.md 2> $O/${T}_fig1_build.err
fi
# (compute-sanitizer is closed on the GPU pool: not run)
[ -z "${NOPGR:-}" ] && timeout 900 python tools/pgr_experiment.py C2 C3 C4 > $O/${T}_pgr.md 2> $O/${T}_pgr.err
