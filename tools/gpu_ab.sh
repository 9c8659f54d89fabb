#!/bin/bash
tag=${1:-ab}
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$tag.log 2>&1 || { tail -20 gpurun_out/build_$tag.log; exit 1; }
tools/perf_quick.sh $tag C2 C5 C5:accurate C3:accurate C3:index
timeout 600 python -m pytest tests -m gpu -q -x -p no:cacheprovider -k "parity or golden or random or repeat" > gpurun_out/pytest_$tag.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_$tag.log
