# A/B: chain mu(c) CAS (R27a) against the plain store (GPU box)
O=gpurun_out
for i in 1 2 3; do MCM_LIB=build_ab/plain.so python tools/variance.py C2 20 >> $O/ab_plain.txt 2>&1; python tools/variance.py C2 20 >> $O/ab_cas.txt 2>&1; done
for c in C3 C5; do MCM_LIB=build_ab/plain.so python tools/variance.py $c 10 >> $O/ab_plain.txt 2>&1; python tools/variance.py $c 10 >> $O/ab_cas.txt 2>&1; done
timeout 600 compute-sanitizer --tool racecheck python tools/sanitize.py quick > $O/r27b_san_racecheck.log 2>&1
