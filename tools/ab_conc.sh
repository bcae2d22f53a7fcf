# A/B (GPU box): concurrent GR (NEXT-2) on A CTAs vs the default single-kernel solve
O=gpurun_out
for i in 1 2; do for c in C2 C3 C4 C5; do
  r=10; [ $c = C2 ] && r=20
  timeout 300 python tools/ab_solve.py $c $r default >> $O/ab_conc.txt 2>&1
  for a in 16 48 74; do timeout 300 python tools/ab_solve.py $c $r conc$a gr_concurrent=$a >> $O/ab_conc.txt 2>&1; done
  timeout 300 python tools/ab_solve.py $c $r conc48_k2 gr_concurrent=48,k=2.0 >> $O/ab_conc.txt 2>&1
done; done
