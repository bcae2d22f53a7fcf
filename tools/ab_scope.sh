# A/B: vertex-state scope of the lean kernel (cta everywhere vs gpu everywhere), GPU box
O=gpurun_out
for i in 1 2; do for c in C2 C4 C3 C5; do
  r=10; [ $c = C2 ] && r=20
  for v in cta gpu; do MCM_LIB=build_ab/$v.so timeout 300 python tools/ab_solve.py $c $r $v >> $O/ab_scope.txt 2>&1; done
done; done
