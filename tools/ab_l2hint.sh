# A/B: L2 eviction-priority hints (GPU box)
O=gpurun_out
for i in 1 2; do for c in C4 C3 C5 C2; do
  r=10; [ $c = C2 ] && r=20
  for v in 0 1 2; do MCM_TRANSPOSE=scatter MCM_LIB=build_ab/l2h_$v.so timeout 300 python tools/ab_solve.py $c $r l2h_$v >> $O/ab_l2hint.txt 2>&1; done
done; done
