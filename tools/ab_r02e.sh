# A/B (GPU box): current build vs bottom-up flush once vs the round-1 structure (zero-spill widths)
O=gpurun_out
for i in 1 2; do for c in C2 C3 C4 C5; do
  r=10; [ $c = C2 ] && r=20
  for v in cur bf_once sp_b; do MCM_LIB=build_ab/$v.so timeout 300 python tools/ab_solve.py $c $r $v >> $O/ab_r02e.txt 2>&1; done
done; done
