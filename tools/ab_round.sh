# k and gr_target sweep around the r01g defaults (GPU box)
O=gpurun_out
for c in C2 C4 C3 C5; do for i in 1 2; do
  r=10; [ $c = C2 ] && r=20
  for o in k=0.4 k=0.25 k=0.7 k=1.0 gr_target=0.5 gr_target=0.6,gr_target_min=1024; do
    timeout 300 python tools/ab_solve.py $c $r x $o 2>&1 | sed "s/^x /$o /" >> $O/r01g_sweep.txt
  done
done; done
