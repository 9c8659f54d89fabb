mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_x16.log 2>&1 || { tail -20 gpurun_out/build_x16.log; exit 1; }
timeout 1500 python -m pytest tests -m gpu -q -x > gpurun_out/pytest_x16.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/pytest_x16.log
: > gpurun_out/bench_x16.jsonl
for spec in "C2" "C3 --mode accurate" "C4" "C5" "C5 --mode accurate"; do
  timeout 300 python bench.py --config $spec --steps 10 --warmup 3 --no-cpu-baseline --e2e-steps 0 2>/dev/null | tail -1 >> gpurun_out/bench_x16.jsonl
done
python tools/bench_table.py gpurun_out/bench_x16.jsonl
timeout 300 python tools/emulate_strong.py --config C4 --points 2e9 --ranks 8 --only-rank 3 --steps 10 2>/dev/null | tail -1 | cut -c1-500
