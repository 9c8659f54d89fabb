mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_x10.log 2>&1 || { tail -20 gpurun_out/build_x10.log; exit 1; }
timeout 300 python -m pytest tests/test_gpu_parity.py -q -x -k "sum_avg or label or tracts or counties" 2>&1 | tail -4
timeout 900 python -m pytest tests -m gpu -q -x > gpurun_out/pytest_x10.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/pytest_x10.log
: > gpurun_out/bench_x10.jsonl
for spec in "C3 --mode bounded" "C3 --mode accurate" "C4"; do
  timeout 300 python bench.py --config $spec --steps 10 --warmup 3 --no-cpu-baseline --e2e-steps 0 2>/dev/null | tail -1 >> gpurun_out/bench_x10.jsonl
done
python tools/bench_table.py gpurun_out/bench_x10.jsonl
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_point_pass -s 2 -c 1 -o gpurun_out/prof_C3b_x10 -f python bench.py --config C3 --mode bounded --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1; echo "ncu C3b rc=$?"
