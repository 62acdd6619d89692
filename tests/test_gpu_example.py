"""The C ABI from plain C: build/aol_example (examples/aol_example.c) runs on the GPU and its printed per-frame
checksums equal the CPU oracle's for the same seeded frames."""
import os
import re
import subprocess

import numpy as np
import pytest

import synth
from conftest import ROOT

pytestmark = pytest.mark.gpu


def test_c_example_matches_oracle(orc):
    exe = os.path.join(ROOT, "build", "aol_example")
    if not os.path.exists(exe):
        subprocess.check_call(["make", "-C", ROOT, exe])
    r = subprocess.run([exe, "3", "7"], capture_output=True, text=True, timeout=300)
    assert r.returncode == 0, r.stdout + r.stderr
    assert "fused == unfused == generic == plan: yes" in r.stdout
    assert "invalid width -> status -2" in r.stdout
    got = {int(n): int(v) for n, v in re.findall(r"checksum (\d+) (\d+)", r.stdout)}
    _, cs = orc.downscale_frame(synth.frames(7, 0, 3, 3, 1080, 1920, "uniform"), nthreads=8)
    assert [got[n] for n in range(3)] == [int(c) for c in cs]


def test_c_enqueue_timing_mode():
    """The d1 host-enqueue probe bench.py runs: one JSON line with both timings."""
    import json

    exe = os.path.join(ROOT, "build", "aol_example")
    r = subprocess.run([exe, "--enqueue-us", "400"], capture_output=True, text=True, timeout=300)
    assert r.returncode == 0, r.stdout + r.stderr
    d = json.loads(r.stdout.strip().splitlines()[-1])
    assert 0 < d["plan_launch_us"] < d["downscale_frame_us"]
