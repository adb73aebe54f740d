"""compute-sanitizer over every kernel family: memcheck (out-of-bounds and
misaligned accesses), racecheck (shared-memory hazards), synccheck (barrier misuse) and
initcheck (reads of uninitialised device memory) on small grids through the C ABI
(tools/sanitize_cases.py, which also checks each result against the oracle)."""
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
    if not os.path.exists(SAN):
        pytest.skip("compute-sanitizer not installed")
    cmd = [SAN, "--tool", tool, "--error-exitcode", "97", "--print-limit", "20"]
    if tool == "initcheck":
        # the workspace tail (flags/counters) is memset by stencil_run itself; cudaMalloc'd
        # grids are fully written by the host before the run
        cmd += ["--check-api-memory-access", "yes"]
    cmd += [sys.executable, os.path.join(ROOT, "tools", "sanitize_cases.py")]
    r = subprocess.run(cmd, capture_output=True, text=True, timeout=1500, cwd=ROOT)
    out = r.stdout + r.stderr
    os.makedirs(os.path.join(ROOT, "gpurun_out"), exist_ok=True)
    with open(os.path.join(ROOT, "gpurun_out", f"sanitizer_{tool}.txt"), "w") as f:
        f.write(out)
    if "closed on this pool" in out:
        # the pool's sanitizer wrapper refuses to run (it left GPUs needing a reset); the
        # committed logs under profiles/round2/sanitizer_*.txt are the last clean runs
        pytest.skip("compute-sanitizer closed on this GPU pool: " + out.strip().splitlines()[-1][:160])
    assert r.returncode == 0, out[-4000:]
    assert "ERROR SUMMARY: 0 errors" in out or "RACECHECK SUMMARY: 0 hazards" in out, out[-4000:]
