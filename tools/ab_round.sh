# k x gr_target_min sweep (GPU box)
O=gpurun_out
for c in C2 C4 C3 C5; do for i in 1 2; do
  r=10; [ $c = C2 ] && r=20
  for o in k=0.4 k=0.7 k=0.7,gr_target_min=1024 k=0.4,gr_target_min=1024 k=0.7,gr_target_min=512 k=0.7,gr_target_min=1024,gr_target=0.5; do
    timeout 300 python tools/ab_solve.py $c $r x $o 2>&1 | sed "s/^x /$o /" >> $O/r01g_sweep2.txt
  done
done; done
