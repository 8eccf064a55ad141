"""compute-sanitizer over one small launch of every kernel family (racecheck,
synccheck for the shared-memory / barrier / mbarrier code; memcheck and
initcheck for the bounds of the ragged, strided and TMA paths)."""
import os
import shutil
import subprocess
import sys

import pytest

pytestmark = [pytest.mark.gpu, pytest.mark.slow]

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
SAN = shutil.which("compute-sanitizer") or "/usr/local/cuda/bin/compute-sanitizer"


@pytest.mark.parametrize("tool", ["memcheck", "racecheck", "synccheck", "initcheck"])
def test_compute_sanitizer(tool):
    torch = pytest.importorskip("torch")
    if not torch.cuda.is_available() or not os.path.exists(SAN):
        pytest.skip("needs a GPU and compute-sanitizer")
    cmd = [SAN, "--tool", tool, "--target-processes", "all", "--error-exitcode", "3", sys.executable,
           os.path.join(ROOT, "tools", "sanitize_target.py")]
    r = subprocess.run(cmd, capture_output=True, text=True, timeout=1200, cwd=ROOT)
    out = r.stdout + r.stderr
    if r.returncode == 86 or "compute-sanitizer is closed" in out:
        # the GPU pool's wrapper refuses sanitizer runs (exit 86); the round-1
        # logs under profiles/ (r01_racecheck_all_families.log, r01_sanitizer_*)
        # are the last runs it allowed
        pytest.skip("compute-sanitizer refused by this GPU pool: " + out.strip()[-200:])
    assert r.returncode == 0, out[-4000:]
    assert "ERROR SUMMARY: 0 errors" in out or "RACECHECK SUMMARY: 0 hazards" in out, out[-4000:]
