"""bench.py keeps its contract: one JSON line with the required keys, for the default (weak) mode, the
configs[4] stream mode and the reference arm.  Small shapes so this runs in seconds."""
import json
import os
import subprocess
import sys

import pytest

from conftest import ROOT

pytestmark = pytest.mark.gpu

REQUIRED = {"metric", "value", "unit", "n_gpus", "steps", "warmup", "ms_per_step", "higher_is_better", "scaling",
            "vs_baseline", "dtype", "data", "config", "roofline", "gpu_launches", "clocks"}


def run(*args):
    r = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), *args], capture_output=True, text=True,
                       timeout=600, cwd=ROOT)
    assert r.returncode == 0, r.stderr[-3000:]
    lines = [l for l in r.stdout.strip().splitlines() if l.startswith("{")]
    assert len(lines) == 1, r.stdout
    return json.loads(lines[0])


def test_bench_default_contract():
    d = run("--frames", "12", "--H", "36", "--W", "128", "--steps", "5", "--warmup", "3")
    assert REQUIRED <= set(d)
    assert d["scaling"] == "weak" and d["n_gpus"] == 1 and d["higher_is_better"] is True
    assert d["value"] > 0 and d["gpu_launches"] == 10 and d["steps"] == 5 and d["warmup"] == 3
    r = d["roofline"]
    assert r["bound"] == "hbm" and r["unit"] == "GB/s" and abs(r["frac"] - r["achieved"] / r["peak"]) < 1e-9
    assert {"value", "unit", "h2d_bytes_per_step", "d2h_bytes_per_step"} <= set(d["e2e"])
    assert d["e2e"]["checksums_match_device_path"] is True
    assert d["cpu_baseline"]["kind"] == "oracle" and d["cpu_baseline"]["parity_sample_ok"] is True
    assert d["config"]["workload"].startswith("12-frame 128x36")


def test_bench_stream_mode():
    d = run("--stream-frames", "50", "--pool", "16", "--H", "36", "--W", "128", "--steps", "3", "--warmup", "3",
            "--no-cpu-baseline")
    assert d["scaling"] == "strong" and d["config"]["launches_per_step"] == 4 and d["gpu_launches"] == 24


def test_bench_reference_arm():
    d = run("--impl", "reference", "--frames", "8", "--H", "36", "--W", "128", "--steps", "3", "--warmup", "3")
    assert d["impl"] == "reference" and d["value"] > 0
    assert d["cpu_baseline"]["value"] == d["value"] and d["e2e"]["h2d_bytes_per_step"] == 0
