# A/B: early-stop GR target fraction (MCM_GR_TARGET builds) on C2, C3, C5 (GPU box)
O=gpurun_out
for i in 1 2 3; do for v in base t0.95 t0.8; do
  if [ $v = base ]; then unset MCM_LIB; else export MCM_LIB=build_ab/$v.so; fi
  python tools/ab_solve.py C2 20 $v >> $O/ab_target.txt 2>&1
done; done
for c in C3 C5; do for v in base t0.95 t0.8; do
  if [ $v = base ]; then unset MCM_LIB; else export MCM_LIB=build_ab/$v.so; fi
  python tools/ab_solve.py $c 10 $v >> $O/ab_target.txt 2>&1
done; done
