"""Run tests/test_gpu_random.py's randomised parity case over a seed range
(one-off deep validation): python tools/stress_random.py LO HI"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
sys.path.insert(0, os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))), "tests"))
import test_gpu_random as T  # noqa: E402

lo, hi = int(sys.argv[1]), int(sys.argv[2])
bad = []
for s in range(lo, hi):
    try:
        T.test_random_parity(s)
    except AssertionError as e:
        bad.append(s)
        print("FAIL", s, str(e)[:300], flush=True)
print(f"seeds {lo}..{hi}: {hi - lo - len(bad)} passed, {len(bad)} failed {bad}", flush=True)
