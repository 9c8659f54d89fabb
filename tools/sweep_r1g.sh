python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build.log 2>&1
timeout 600 python -m pytest tests/test_gpu_index_join.py tests/test_gpu_parity.py -q -x 2>&1 | tail -2
run() { timeout 400 python bench.py --steps 5 --warmup 3 --e2e-steps 0 --no-cpu-baseline "$@" 2>&1 | tail -1 | python -c "import json,sys; d=json.loads(sys.stdin.read()); print(sys.argv[1:], round(d['value']/1e9,1), round(d['ms_per_step'],3), round(d['roofline']['kernel_ms'],3), round(d['stages_ms']['polygon_pass'],3), d['checks']['n_boundary'], d['launch'])" "$@"; }
run --config C3
run --config C3 --stages 2
run --config C3 --pass-variant 0
run --config C3 --pass-variant 0 --stages 3
run --config C3 --mode index
run --config C3 --mode index --stages 2
run --config C2 --mode index
run --config C2 --mode accurate
run --config C2 --mode accurate --stages 2
run --config C2
