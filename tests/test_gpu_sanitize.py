"""compute-sanitizer over small instances of the kernel families (PAPER.md is
silent): memcheck (out-of-bounds / misaligned accesses, including the TMA and bulk-copy paths),
racecheck (shared-memory hazards: the staged tile loop, the loop kernels' rings) and synccheck.
The full sweep over every family and tool is scripts/sanitize.sh (log under profiles/: clean in r02).

compute-sanitizer has since been closed on the GPU pool (runs under it left GPUs needing a reset), so
the sanitizer runs are opt-in (SG_SANITIZER=1 on a box where the tool is allowed); by default the same
small cases run without it, each checked against the oracle (test_sanitize_cases_parity)."""
import os
import subprocess
import sys

import pytest

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.mark.parametrize("tool,case", [("memcheck", "tma_register"), ("memcheck", "staged_fused_fb"),
                                       ("memcheck", "rings_chain"), ("racecheck", "staged_fused_fm"),
                                       ("racecheck", "loop_barrier"), ("synccheck", "bitslice_rolled"),
                                       ("memcheck", "gather_views")])
def test_compute_sanitizer_clean(tool, case):
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    if os.environ.get("SG_SANITIZER") != "1":
        pytest.skip("compute-sanitizer is closed on the GPU pool; opt in with SG_SANITIZER=1")
    r = subprocess.run(["compute-sanitizer", "--tool", tool, "--error-exitcode", "3", sys.executable,
                        os.path.join(ROOT, "scripts", "sanitize_cases.py"), "--case", case],
                       capture_output=True, text=True, timeout=900, cwd=ROOT)
    out = r.stdout + r.stderr
    assert "parity OK" in out, out[-3000:]
    assert r.returncode == 0, out[-3000:]
    assert "ERROR SUMMARY: 0 errors" in out or "RACECHECK SUMMARY: 0 hazards" in out, out[-3000:]


@pytest.mark.parametrize("case", ["tma_register", "staged_fused_fb", "rings_chain", "staged_fused_fm",
                                  "loop_barrier", "bitslice_rolled", "gather_views"])
def test_sanitize_cases_parity(case):
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    r = subprocess.run([sys.executable, os.path.join(ROOT, "scripts", "sanitize_cases.py"), "--case", case],
                       capture_output=True, text=True, timeout=900, cwd=ROOT)
    out = r.stdout + r.stderr
    assert r.returncode == 0 and "parity OK" in out, out[-3000:]
