set -u
O=gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv > $O/san_gpu.txt 2>&1
timeout 600 compute-sanitizer --tool memcheck --leak-check full python tests/sanitize_solves.py > $O/san_memcheck.log 2>&1; echo "memcheck rc=$?" >> $O/san_rc.txt
timeout 400 compute-sanitizer --tool synccheck python tests/sanitize_solves.py quick > $O/san_synccheck.log 2>&1; echo "synccheck rc=$?" >> $O/san_rc.txt
timeout 600 compute-sanitizer --tool racecheck python tests/sanitize_solves.py quick > $O/san_racecheck.log 2>&1; echo "racecheck rc=$?" >> $O/san_rc.txt
timeout 400 compute-sanitizer --tool initcheck python tests/sanitize_solves.py quick > $O/san_initcheck.log 2>&1; echo "initcheck rc=$?" >> $O/san_rc.txt
python tools/variance.py C2 20 > $O/var_C2_base.txt 2>&1
