# tail_f / bu_div sweep at the r01h defaults (GPU box)
O=gpurun_out
for c in C2 C5 C3; do for i in 1 2; do
  r=10; [ $c = C2 ] && r=20
  for o in tail_f=128 tail_f=256 tail_f=512 tail_f=64 bu_div=16 bu_div=8; do
    timeout 300 python tools/ab_solve.py $c $r x $o 2>&1 | sed "s/^x /$o /" >> $O/r01h_sweep.txt
  done
done; done
