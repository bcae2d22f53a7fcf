for cfg in "1 0" "2 0" "2 148" "2 132" "2 120" "2 100" "3 120" "4 100"; do
  set -- $cfg
  timeout 600 python bench.py --config C5 --steps 3 --warmup 3 --no-cpu-baseline --streams $1 --solve-ctas $2 > /tmp/c5.json 2>/tmp/c5.err
  python -c "import json; d=json.load(open('/tmp/c5.json')); print('streams $1 ctas $2', round(d['ms_per_step'],1), 'ms', '%.3g'%d['value'], 'e2e %.3g'%d['e2e']['value'])" || tail -3 /tmp/c5.err
done
