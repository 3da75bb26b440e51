"""bench.py's one-JSON-line contract on one B200: the keys the driver reads, the
roofline / cpu_baseline / e2e / clocks objects, launches of this library's
kernels, and the bench's own parity check against the oracle."""
import json
import os
import subprocess
import sys

import pytest

pytestmark = pytest.mark.gpu
torch = pytest.importorskip("torch")

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _run(*args):
    out = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), *args], cwd=ROOT, capture_output=True,
                         text=True, timeout=900)
    assert out.returncode == 0, out.stderr[-2000:]
    lines = [l for l in out.stdout.strip().splitlines() if l.startswith("{")]
    assert len(lines) == 1, out.stdout[-2000:]
    return json.loads(lines[0])


def test_bench_line_contract():
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    d = _run("--steps", "5", "--warmup", "3", "--e2e-steps", "2", "--cpu-seconds", "1", "--latency-reps", "3",
             "--replays", "1")
    for k in ("metric", "value", "unit", "n_gpus", "steps", "warmup", "ms_per_step", "higher_is_better", "scaling",
              "vs_baseline", "dtype", "data", "config", "roofline", "cpu_baseline", "e2e", "gpu_launches", "clocks"):
        assert k in d, k
    assert d["n_gpus"] == 1 and d["steps"] == 5 and d["warmup"] == 3 and d["value"] > 0
    assert d["config"]["workload"].startswith("C4") and d["config"]["table_rows"] == 600_000_000
    r = d["roofline"]
    assert r["bound"] == "hbm" and r["unit"] == "GB/s" and 0 < r["frac"] < 1.2
    assert abs(r["frac"] - r["achieved"] / r["peak"]) < 1e-9
    assert d["cpu_baseline"]["kind"] == "oracle" and d["cpu_baseline"]["cores"] >= 1
    e = d["e2e"]
    assert e["h2d_bytes_per_step"] > 0 and e["d2h_bytes_per_step"] > 0 and e["value"] > 0
    assert d["gpu_launches"] >= 5 and d["parity"]["match"]
    assert "sm_mhz" in d["clocks"] and "reasons" in d["clocks"]
    assert d["cpu_baseline"]["cpu"]["model"]
    # single-query latency next to throughput, replay distribution, the C2 and C5 side configurations
    lat = d["latency"]["fused"]["ms"]
    assert lat["min"] <= lat["median"] <= lat["p90"] and lat["n"] == 3
    assert d["ms_per_step_replays"]["n"] == 2
    assert d["c2"]["parity"]["match"] and d["c2"]["frac"] > 0
    c5 = d["c5"]
    assert c5["parity"]["match"] and 0 < c5["host_link"]["frac"] < 1.5 and c5["host_link"]["peak"] > 1


def test_bench_reference_arm():
    d = _run("--impl", "reference", "--steps", "1", "--warmup", "0")
    assert d["impl"] == "reference" and d["value"] > 0
    assert d["cpu_baseline"]["kind"] == "oracle"
    assert d["e2e"]["h2d_bytes_per_step"] == 0 and d["e2e"]["d2h_bytes_per_step"] == 0
