"""Small launches of every kernel (tools/sanitize_workload.py), results compared across paths.

The workload was written for compute-sanitizer memcheck / synccheck / racecheck (clean in the committed runs,
profiles/r01_sanitizers.txt, profiles/r02_v2_sanitize_summary.txt; analysis in DESIGN.md "Sanitizers").  The
GPU pool has since closed compute-sanitizer (runs under it left GPUs needing a reset), so the test runs the
workload directly: every kernel on small shapes, including edge cases, with the cross-path agreement checks
the workload asserts itself.
"""
import os
import subprocess
import sys

import pytest

from conftest import ROOT

pytestmark = pytest.mark.gpu


def test_sanitize_workload_runs_clean():
    r = subprocess.run([sys.executable, os.path.join(ROOT, "tools", "sanitize_workload.py")],
                       capture_output=True, text=True, timeout=900, cwd=ROOT)
    assert r.returncode == 0, r.stdout[-3000:] + r.stderr[-3000:]
    assert "sanitize workload: OK" in r.stdout
