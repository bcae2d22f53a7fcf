O=gpurun_out
for i in 1 2; do for c in C3 C4 C5; do
  for v in cur u0cta; do MCM_LIB=build_ab/$v.so timeout 300 python tools/ab_solve.py $c 10 $v >> $O/ab_r02f.txt 2>&1; done
done; done
