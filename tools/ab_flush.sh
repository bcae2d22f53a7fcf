# A/B: BFS frontier flushed once per level + huge push lists once per phase (new) vs per tile (old), GPU box
O=gpurun_out
for i in 1 2; do for c in C4 C3 C5 C2; do
  r=10; [ $c = C2 ] && r=20
  for v in old new; do MCM_LIB=build_ab/fl_$v.so timeout 300 python tools/ab_solve.py $c $r fl_$v >> $O/ab_flush.txt 2>&1; done
done; done
