python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
run() { timeout 300 python bench.py --config C4 --steps 10 --warmup 3 --no-cpu-baseline --e2e-steps 0 "$@" 2>/dev/null | tail -1 | python -c "import json,sys; d=json.loads(sys.stdin.read()); print(round(d['ms_per_step'],3), round(d['stages_ms']['point_pass'],3))"; }
for i in 1 2; do
echo -n "OLD      "; (cd _old && run)
echo -n "NEW      "; run
echo -n "NEW nogr "; run --no-graphs
echo -n "V2(exch) "; (cd _v2 && run)
done
