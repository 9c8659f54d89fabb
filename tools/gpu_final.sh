#!/bin/bash
# Final round check: build, all GPU tests, smoke, the contract bench line, the
# reference arm, per-config lines, C5 sweep, ncu launch list and a full
# capture of the point pass (C2) and of the label kernel (C4).
tag=${1:-r1s3f}
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$tag.log 2>&1 || { echo build failed; tail gpurun_out/build_$tag.log; exit 1; }
timeout 1500 python -m pytest tests -m gpu -q -x > gpurun_out/pytest_gpu_$tag.log 2>&1; echo "pytest rc=$?" >> gpurun_out/pytest_gpu_$tag.log
tail -3 gpurun_out/pytest_gpu_$tag.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke_$tag.log 2>&1; echo "smoke rc=$?"; tail -1 gpurun_out/smoke_$tag.log
timeout 900 python bench.py > gpurun_out/bench_$tag.json 2> gpurun_out/bench_$tag.err; echo "bench rc=$?"; tail -c 300 gpurun_out/bench_$tag.json
timeout 300 python bench.py --impl reference --steps 3 --warmup 3 > gpurun_out/bench_ref_$tag.json 2>&1; echo "ref rc=$?"
: > gpurun_out/bench_lines_$tag.jsonl
for spec in "C3 --mode bounded" "C3 --mode accurate" "C4" "C5" "C5 --mode accurate" "C3 --mode index"; do
  timeout 600 python bench.py --config $spec --steps 10 --warmup 3 --no-cpu-baseline --e2e-steps 1 2>/dev/null | tail -1 >> gpurun_out/bench_lines_$tag.jsonl
done
python tools/bench_table.py gpurun_out/bench_lines_$tag.jsonl
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 600 --csv --log-file gpurun_out/launches_$tag.csv python bench.py --steps 3 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1; echo "ncu list rc=$?"
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_point_pass -s 2 -c 1 -o gpurun_out/prof_C2_$tag -f python bench.py --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1; echo "ncu C2 rc=$?"
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_point_pass -s 2 -c 1 -o gpurun_out/prof_C4_$tag -f python bench.py --config C4 --steps 1 --warmup 3 --e2e-steps 0 --no-cpu-baseline > /dev/null 2>&1; echo "ncu C4 rc=$?"
