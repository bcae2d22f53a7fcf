# gr_target / gr_target_min sweep (R28) + GPU tests (GPU box)
O=gpurun_out
timeout 900 python -m pytest tests -m gpu -x -q > $O/r28b_gputests.txt 2>&1
for c in C2 C4 C3 C5; do for i in 1 2; do
  r=10; [ $c = C2 ] && r=20
  for o in gr_target=1.0 gr_target=0.6,gr_target_min=65536 gr_target=0.6,gr_target_min=4096 gr_target=0.7,gr_target_min=65536 gr_target=0.5,gr_target_min=65536; do
    timeout 300 python tools/ab_solve.py $c $r x $o 2>&1 | sed "s/^x /$o /" >> $O/r28b_sweep.txt
  done
done; done
