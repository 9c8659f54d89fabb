#!/bin/bash
# GPU suite + per-config lines at HEAD, then the bounds-checked run.
tag=${1:-r2f}
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build_$tag.log 2>&1 || { tail gpurun_out/build_$tag.log; exit 1; }
timeout 1500 python -m pytest tests -m gpu -q -p no:cacheprovider > gpurun_out/pytest_gpu_$tag.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_gpu_$tag.log
tools/perf_quick.sh cfg_$tag C2 C3:bounded C3:accurate C4 C5 C5:accurate > gpurun_out/cfg_$tag.txt 2>&1; cat gpurun_out/cfg_$tag.txt
tools/checks_run.sh $tag
# edge-grid resolution A/B for the accurate PIP (compile-time)
tools/ab_build.sh "g10=" "g11=-DRJ_GRID_BITS=11" -- C3:accurate C3:index > gpurun_out/ab_grid_$tag.txt 2>&1; grep -E '^==|G/s' gpurun_out/ab_grid_$tag.txt | cut -c1-140
python -c "from paper_journals_pvldb_zacharatoudasf17_b200 import _build as b; b.build(force=True)" > /dev/null 2>&1
