# r01f measurement bundle: smoke, GPU tests, bench lines + ncu (tools/profile_round.sh), phase traces
O=gpurun_out
mkdir -p $O
python -c "import __graft_entry__ as g; g.smoke()" > $O/smoke.log 2>&1
timeout 600 python -m pytest tests -m gpu -q > $O/gputests.log 2>&1
bash tools/profile_round.sh
for c in C2 C3 C4; do timeout 300 python tools/trace_solve.py $c > $O/trace_$c.txt 2>&1; done
