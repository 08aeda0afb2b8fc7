"""bench.py keeps the driver's JSON contract: the reference arm on the CPU
(the oracle), the tds arm on a GPU (short runs of configs 1, 3 and 5)."""
import json
import os
import subprocess
import sys

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
BASE_KEYS = {"metric", "value", "unit", "n_gpus", "steps", "warmup", "ms_per_step", "higher_is_better", "scaling",
             "vs_baseline", "dtype", "data", "config", "e2e"}


def run_bench(*args, timeout=600):
    out = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), *args], capture_output=True, text=True,
                         timeout=timeout, cwd=ROOT)
    assert out.returncode == 0, out.stderr[-2000:]
    lines = [l for l in out.stdout.strip().splitlines() if l.startswith("{")]
    assert len(lines) == 1, out.stdout
    return json.loads(lines[0])


def test_reference_arm_contract():
    d = run_bench("--impl", "reference", "--config", "1", "--steps", "3", "--warmup", "1", timeout=300)
    assert BASE_KEYS <= set(d) and d["impl"] == "reference"
    assert d["value"] > 0 and d["unit"] == "eq/s" and d["higher_is_better"] is True
    assert d["cpu_baseline"]["kind"] == "oracle" and d["cpu_baseline"]["value"] == d["value"]
    assert d["e2e"] == {"value": d["value"], "unit": "eq/s", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}


@pytest.mark.gpu
@pytest.mark.parametrize("config", ["1", "3"])
def test_tds_arm_contract(config):
    d = run_bench("--config", config, "--steps", "5", "--warmup", "3", "--soak-s", "0")
    assert BASE_KEYS <= set(d) and "impl" not in d
    assert d["value"] > 0 and d["n_gpus"] == 1 and d["scaling"] == "strong"
    r = d["roofline"]
    assert {"bound", "achieved", "peak", "unit", "frac", "traffic"} <= set(r) and r["bound"] == "hbm"
    assert d["gpu_launches"] >= 5
    assert {"sm_mhz", "sm_max_mhz", "reasons"} <= set(d["clocks"])
    assert d["e2e"]["h2d_bytes_per_step"] > 0 and d["e2e"]["d2h_bytes_per_step"] > 0
    assert d["cpu_baseline"]["kind"] == "oracle" and d["cpu_baseline"]["cores"] >= 1
    assert d["cpu_baseline"]["gpu_vs_oracle_rel_err"] <= 1e-4
    assert d["config"]["plan"]["onchip_form"]


@pytest.mark.gpu
def test_tds_arm_config5_huge_system():
    d = run_bench("--config", "5", "--steps", "2", "--warmup", "3", "--soak-s", "0", "--no-cpu-baseline")
    assert d["scaling"] == "strong" and d["config"]["m"] == 1 and d["config"]["fused_single_gpu_plan"] is True
    assert d["config"]["interior_residual"] <= 1e-5
    assert d["roofline"]["nvlink_bytes_per_rank"]["all_to_all_split"] == 0


def test_algorithmic_bytes_accounting():
    """split pass 1 7 s/eq, later passes 6 s, on-chip 4 s (5 s
    at k = 0), placement 2 s (k > 0, no x_group / strided)."""
    sys.path.insert(0, ROOT)
    import bench
    info = dict(n=1 << 20, m=16, passes=1, k=7, k_pass=[7], x_group=0, strided=0)
    eqs = 16 << 20
    assert bench.algorithmic_bytes(info, 4) == [28 * eqs, 16 * eqs, 8 * eqs]  # 52 B/eq
    assert bench.stage_names(info) == ["split_pass_0(k_p=7)", "onchip_cr_pcr_thomas", "place_x"]
    two = dict(info, passes=2, k=15, k_pass=[8, 7], m=1, n=1 << 28)
    assert sum(bench.algorithmic_bytes(two, 4)) == 76 * (1 << 28)  # config 5: 28 + 24 + 16 + 8 B/eq
    k0 = dict(info, passes=0, k=0, k_pass=[])
    assert bench.algorithmic_bytes(k0, 4) == [20 * eqs]
    assert bench.algorithmic_bytes(dict(info, x_group=8), 8) == [56 * eqs, 32 * eqs]
