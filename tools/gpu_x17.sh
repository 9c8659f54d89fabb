mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_x17.log 2>&1 || { tail -20 gpurun_out/build_x17.log; exit 1; }
timeout 900 python -m pytest tests -m gpu -q -x -k "accurate or index or random or stream or tracts or interval" > gpurun_out/pytest_x17.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_x17.log
: > gpurun_out/bench_x17.jsonl
for spec in "C3 --mode accurate" "C5 --mode accurate" "C3 --mode index"; do
  timeout 300 python bench.py --config $spec --steps 10 --warmup 3 --no-cpu-baseline --e2e-steps 0 2>/dev/null | tail -1 >> gpurun_out/bench_x17.jsonl
done
python tools/bench_table.py gpurun_out/bench_x17.jsonl
