#!/bin/bash
# Bounds-checked run (compute-sanitizer is closed on this pool): build librj
# with -DRJ_CHECKS (device checks of shared-tile indices, span-piece rows and
# columns, queue and piece slots; a failure traps) and run the GPU suite and
# the every-variant driver tools/sanitize.py on it.   tools/checks_run.sh TAG
tag=${1:-r2}
mkdir -p gpurun_out
RJ_NVCC_EXTRA="-DRJ_CHECKS" python -c "from paper_journals_pvldb_zacharatoudasf17_b200 import _build as b; b.build(force=True)" > gpurun_out/build_checks_$tag.log 2>&1 || { tail gpurun_out/build_checks_$tag.log; exit 1; }
timeout 1500 python -m pytest tests -m gpu -q -p no:cacheprovider > gpurun_out/checks_pytest_$tag.log 2>&1; echo "checked pytest rc=$?"; tail -2 gpurun_out/checks_pytest_$tag.log
timeout 900 python tools/sanitize.py > gpurun_out/checks_driver_$tag.log 2>&1; echo "checked driver rc=$?"; tail -2 gpurun_out/checks_driver_$tag.log
grep -h "RJ_DCHECK failed" gpurun_out/checks_*_$tag.log | sort | uniq -c | head; echo "dcheck failures: $(cat gpurun_out/checks_*_$tag.log | grep -c "RJ_DCHECK failed")"
python -c "from paper_journals_pvldb_zacharatoudasf17_b200 import _build as b; b.build(force=True)" > /dev/null 2>&1
