# r01h measurement bundle: smoke, GPU tests, bench lines + ncu (tools/profile_round.sh), racecheck of the small solves
O=gpurun_out
mkdir -p $O
python -c "import __graft_entry__ as g; g.smoke()" > $O/h_smoke.log 2>&1
timeout 900 python -m pytest tests -m gpu -q > $O/h_gputests.log 2>&1
bash tools/profile_round.sh
timeout 600 compute-sanitizer --tool racecheck python tools/sanitize.py quick > $O/h_san_racecheck.log 2>&1
timeout 600 compute-sanitizer --tool memcheck python tools/sanitize.py quick > $O/h_san_memcheck.log 2>&1
