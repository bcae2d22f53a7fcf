# A/B: batch widths of the wide phases (spills vs memory-level parallelism), GPU box
O=gpurun_out
for i in 1 2; do for c in C4 C3 C5 C2; do
  r=10; [ $c = C2 ] && r=20
  for v in a b c d; do MCM_LIB=build_ab/sp_$v.so timeout 300 python tools/ab_solve.py $c $r sp_$v >> $O/ab_spill.txt 2>&1; done
done; done
