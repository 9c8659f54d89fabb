mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_x7.log 2>&1 || { tail -20 gpurun_out/build_x7.log; exit 1; }
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_multi.py tests/test_gpu_repeat.py -q -x 2>&1 | tail -8
: > gpurun_out/bench_x7.jsonl
for spec in "C3 --mode bounded" "C3 --mode accurate" "C4"; do
  timeout 600 python bench.py --config $spec --steps 10 --warmup 3 --no-cpu-baseline --e2e-steps 0 2>/dev/null | tail -1 >> gpurun_out/bench_x7.jsonl
done
python tools/bench_table.py gpurun_out/bench_x7.jsonl
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k_prow_emit|k_prow_count" -s 4 -c 2 -o gpurun_out/prof_prow_x7 -f python tools/emulate_strong.py --config C2 --ranks 8 --only-rank 0 --steps 2 > /dev/null 2>&1; echo "ncu prow rc=$?"
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_point_pass -s 2 -c 1 -o gpurun_out/prof_C4_x7 -f python bench.py --config C4 --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1; echo "ncu C4 rc=$?"
