O=gpurun_out/r02g_cluster_ab.txt
: > $O
for c in C2 C3; do
for o in tail_ctas=1,tail_f=128 tail_ctas=8,tail_f=128 tail_ctas=8,tail_f=2048 tail_ctas=8,tail_f=8192 tail_ctas=16,tail_f=4096 tail_ctas=16,tail_f=16384 tail_ctas=16,tail_f=65536; do
  timeout 300 python tools/ab_solve.py $c 10 "$o" $o >> $O 2>&1
done; done
