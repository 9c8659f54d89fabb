#!/bin/bash
# Round-2 GPU check: build, GPU tests, smoke, contract bench line (+ ns-c4),
# per-config lines, load timing.   tools/r2_check.sh TAG
tag=${1:-r2}
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$tag.log 2>&1 || { echo build failed; tail gpurun_out/build_$tag.log; exit 1; }
timeout 1500 python -m pytest tests -m gpu -q -x -p no:cacheprovider > gpurun_out/pytest_gpu_$tag.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_gpu_$tag.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke_$tag.log 2>&1; echo "smoke rc=$?"; tail -1 gpurun_out/smoke_$tag.log
timeout 900 python bench.py --ns-c4 > gpurun_out/bench_$tag.json 2> gpurun_out/bench_$tag.err; echo "bench rc=$?"; tail -c 400 gpurun_out/bench_$tag.err
timeout 600 python tools/load_timing.py > gpurun_out/load_$tag.json 2>&1; echo "load rc=$?"; tail -c 800 gpurun_out/load_$tag.json
