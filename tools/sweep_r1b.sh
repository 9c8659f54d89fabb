timeout 900 python -m pytest tests/test_gpu_parity.py -q -x 2>&1 | tail -3
run() { timeout 400 python bench.py --steps 5 --warmup 3 --e2e-steps 0 --no-cpu-baseline "$@" 2>&1 | tail -1 | python -c "import json,sys; d=json.loads(sys.stdin.read()); print(sys.argv[1:], round(d['value']/1e9,1), round(d['ms_per_step'],3), round(d['roofline']['kernel_ms'],3), round(d['roofline']['frac'],3), round(d['stages_ms']['polygon_pass'],3), d['checks'], d['launch'])" "$@"; }
run --config C2
run --config C3 --tile 32
run --config C3 --tile 64
run --config C3 --tile 64 --pass-variant 0
run --config C4
run --config C5
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_point_pass -s 3 -c 1 -o gpurun_out/prof_C3_r1b python bench.py --config C3 --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1
