"""Per-kernel registers / spills / stack of the point-pass kernels (ptxas -v).
    python tools/ptxas_report.py [regex]"""
import os
import re
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
from paper_journals_pvldb_zacharatoudasf17_b200 import _build as B  # noqa: E402

pat = re.compile(sys.argv[1] if len(sys.argv) > 1 else "k_point_pass|k_pip")
for src in ("pass.cu", "pass_label.cu"):
    cmd = [B.NVCC, *B.FLAGS, "-maxrregcount=96", "-Xptxas", "-v", "-c", os.path.join(B.CSRC, src), "-o", "/dev/null"]
    err = subprocess.run(cmd, capture_output=True, text=True).stderr.splitlines()
    fn = None
    for ln in err:
        m = re.search(r"Compiling entry function '(\S+)'", ln) or re.search(r"Function properties for (\S+)", ln)
        if m:
            fn = m.group(1)
            dem = subprocess.run(["c++filt", fn], capture_output=True, text=True).stdout.strip()
            short = re.sub(r"rj::\(anonymous namespace\)::|\(rj::PassArgs\)|rj::", "", dem)
        if fn and pat.search(fn) and ("spill" in ln or "Used" in ln):
            print(f"{short:60s} {ln.strip()}")
