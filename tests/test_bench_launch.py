"""bench.py's multi-GPU launch path on CPU (-m "not gpu"): `--gpus N` without
torchrun re-launches the script as N local ranks (torch.distributed.run,
127.0.0.1), and `--backend gloo --dry-run` runs the real strong-scaling
shards, the spatial all_to_all exchange, the rank windows
(rj_resolve_window), the all-reduce of the partials and the max-over-ranks
timing with the CPU oracle in place of the GPU query.  The JSON line must
report n_gpus = N and the exact-tiling check (every filtered point in exactly
one polygon after the all-reduce)."""
import json
import os
import subprocess
import sys

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.mark.parametrize("n", [2, 3])
def test_bench_gpus_n_launches_n_ranks(n):
    env = {k: v for k, v in os.environ.items() if k not in ("WORLD_SIZE", "RANK", "LOCAL_RANK", "MASTER_ADDR",
                                                             "MASTER_PORT")}
    env["OMP_NUM_THREADS"] = "1"
    r = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), "--gpus", str(n), "--backend", "gloo",
                        "--dry-run", "--points", "40000", "--steps", "2", "--warmup", "3"],
                       capture_output=True, text=True, timeout=600, env=env, cwd=ROOT)
    assert r.returncode == 0, r.stderr[-3000:]
    lines = [ln for ln in r.stdout.splitlines() if ln.startswith("{")]
    assert len(lines) == 1, r.stdout              # rank 0 alone prints
    d = json.loads(lines[0])
    assert d["n_gpus"] == n and d["dry_run"] and d["scaling"] == "strong"
    assert d["config"]["points"] == 40000
    assert d["checks"]["tiling_sum_equals_filtered"] and d["checks"]["n_filtered"] > 0
    assert d["config"]["rank0_view"][0] == 0      # rank 0's strip window starts at column 0


def test_bench_refuses_missing_gpus():
    import torch
    if torch.cuda.device_count() >= 64:
        pytest.skip("64 GPUs visible")
    env = {k: v for k, v in os.environ.items() if k != "WORLD_SIZE"}
    r = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), "--gpus", "64", "--steps", "1"],
                       capture_output=True, text=True, timeout=300, env=env, cwd=ROOT)
    assert r.returncode != 0 and "CUDA device" in (r.stderr + r.stdout)
