#!/bin/bash
# build, a GPU test subset, per-config bench lines: TAG [CFG ...]
tag=${1:-q}; shift
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$tag.log 2>&1 || { tail -20 gpurun_out/build_$tag.log; exit 1; }
timeout 900 python -m pytest tests -m gpu -q -x -p no:cacheprovider -k "parity or golden or random or repeat or view or interval or index" > gpurun_out/pytest_$tag.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_$tag.log
tools/perf_quick.sh $tag "$@"
