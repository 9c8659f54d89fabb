timeout 900 python -m pytest tests/test_gpu_parity.py -q -x 2>&1 | tail -3
run() { timeout 400 python bench.py --steps 5 --warmup 3 --e2e-steps 0 --no-cpu-baseline "$@" 2>&1 | tail -1 | python -c "import json,sys; d=json.loads(sys.stdin.read()); print(sys.argv[1:], round(d['value']/1e9,1), round(d['ms_per_step'],3), round(d['roofline']['kernel_ms'],3), round(d['roofline']['frac'],3), round(d['stages_ms']['polygon_pass'],3), d['checks']['tiling_sum_equals_filtered'])" "$@"; }
run --config C2 --tile 32
run --config C2 --tile 64
run --config C3 --pass-variant 0
run --config C3 --pass-variant 1
run --config C3 --pass-variant 0 --tile 64
run --config C4 --tile 32
run --config C4 --tile 64
run --config C5 --tile 32
run --config C5 --tile 64
run --config C5 --tile 128
