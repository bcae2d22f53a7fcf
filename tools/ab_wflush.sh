# A/B: wide-level flush period (GPU box); plus create-time A/B of the bucketed transpose
O=gpurun_out
for i in 1 2; do for c in C3 C4 C5; do
  for v in 0 1 2 4; do MCM_LIB=build_ab/wf_$v.so timeout 300 python tools/ab_solve.py $c 10 wf_$v >> $O/ab_wflush.txt 2>&1; done
done; done
