#!/bin/bash
tag=${1:-r2f}
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$tag.log 2>&1 || { tail -20 gpurun_out/build_$tag.log; exit 1; }
timeout 1500 python -m pytest tests -m gpu -q -x -p no:cacheprovider > gpurun_out/pytest_gpu_$tag.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_gpu_$tag.log
tools/perf_quick.sh $tag C2 C3:accurate C3:bounded C3:index C4 C5 C5:accurate
timeout 600 python tools/emulate_strong.py --config C4 --points 2e9 --ranks 8 --spatial-only --poly-weight 0.1 > gpurun_out/emul_$tag.jsonl 2>gpurun_out/emul_$tag.err; echo "emul rc=$?"; head -c 300 gpurun_out/emul_$tag.jsonl
