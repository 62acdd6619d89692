"""compute-sanitizer memcheck and synccheck over small launches of every kernel (tools/sanitize_workload.py).

racecheck and initcheck are run by tools/gpu_sanitize2.sh and analysed in DESIGN.md ("Sanitizers"): they flag
only the TMA paths, because the tools do not model 1-D bulk-copy completion through an mbarrier (racecheck,
uint8 path only; the int32 TMA-tensor path is clean) or bulk stores as initialising writes (initcheck).
"""
import os
import shutil
import subprocess
import sys

import pytest

from conftest import ROOT

pytestmark = pytest.mark.gpu


@pytest.mark.parametrize("tool", ["memcheck", "synccheck"])
def test_sanitizer_clean(tool):
    exe = shutil.which("compute-sanitizer") or "/usr/local/cuda/bin/compute-sanitizer"
    if not os.path.exists(exe):
        pytest.skip("compute-sanitizer not installed")
    r = subprocess.run([exe, "--tool", tool, "--error-exitcode", "3", sys.executable,
                        os.path.join(ROOT, "tools", "sanitize_workload.py")],
                       capture_output=True, text=True, timeout=900, cwd=ROOT)
    assert r.returncode == 0, r.stdout[-3000:] + r.stderr[-3000:]
    assert "sanitize workload: OK" in r.stdout
