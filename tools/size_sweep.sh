for n in 125000000 250000000 500000000 1000000000 2000000000; do
  timeout 600 python bench.py --config C4 --points $n --steps 10 --warmup 3 --no-cpu-baseline --e2e-steps 0 2>/dev/null | tail -1 | python -c "
import sys,json; d=json.loads(sys.stdin.read()); r=d['roofline']; print($n, 'step', round(d['ms_per_step'],4), 'kern', round(r['kernel_ms'],4), 'frac', round(r['frac'],3), 'poly', round(d['stages_ms']['polygon_pass'],4), 'items', d['launch']['work_items'])"
done
