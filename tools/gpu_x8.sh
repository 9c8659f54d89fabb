mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_x8.log 2>&1 || { tail -20 gpurun_out/build_x8.log; exit 1; }
timeout 1500 python -m pytest tests -m gpu -q -x > gpurun_out/pytest_x8.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/pytest_x8.log
: > gpurun_out/bench_x8.jsonl
for spec in "C2" "C3 --mode bounded" "C3 --mode accurate" "C4" "C5"; do
  timeout 600 python bench.py --config $spec --steps 10 --warmup 3 --no-cpu-baseline --e2e-steps 0 2>/dev/null | tail -1 >> gpurun_out/bench_x8.jsonl
done
python tools/bench_table.py gpurun_out/bench_x8.jsonl
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_emu8_x8.csv python tools/emulate_strong.py --config C2 --ranks 8 --only-rank 0 --steps 3 > gpurun_out/emu8_x8.log 2>&1; echo "ncu rc=$?"
