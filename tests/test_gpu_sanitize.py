"""compute-sanitizer over small instances of the kernel families (PAPER.md is
silent): memcheck (out-of-bounds / misaligned accesses, including the TMA and bulk-copy paths),
racecheck (shared-memory hazards: the staged tile loop, the loop kernels' rings) and synccheck.
The full sweep over every family and tool is scripts/sanitize.sh (log under profiles/)."""
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
    r = subprocess.run(["compute-sanitizer", "--tool", tool, "--error-exitcode", "3", sys.executable,
                        os.path.join(ROOT, "scripts", "sanitize_cases.py"), "--case", case],
                       capture_output=True, text=True, timeout=900, cwd=ROOT)
    out = r.stdout + r.stderr
    assert "parity OK" in out, out[-3000:]
    assert r.returncode == 0, out[-3000:]
    assert "ERROR SUMMARY: 0 errors" in out or "RACECHECK SUMMARY: 0 hazards" in out, out[-3000:]
