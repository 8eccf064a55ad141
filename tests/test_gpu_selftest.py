"""Bitwise identity of the batched correctly rounded operations
(tridiag_device.cuh rcp_batch / div_batch) with CUDA's rcp.rn / div.rn: every
fp32 reciprocal, 2^33 fp64 reciprocals and 2^33 fp32 quotients (random and
exponent-sweep bit patterns).  These identities are what keep every kernel
path bitwise equal to every other (reading R16) after the batching."""
import json
import os
import shutil
import subprocess

import pytest

pytestmark = [pytest.mark.gpu, pytest.mark.slow]

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
SELF = os.path.join(ROOT, "tools", "selftest")
NVCC = shutil.which("nvcc") or "/usr/local/cuda/bin/nvcc"


@pytest.mark.parametrize("name", ["rcp_exhaustive", "rcp_fp64_check", "div_check"])
def test_batched_ops_bitwise_equal_cuda(name, tmp_path):
    torch = pytest.importorskip("torch")
    if not torch.cuda.is_available() or not os.path.exists(NVCC):
        pytest.skip("needs a GPU and nvcc")
    exe = str(tmp_path / name)
    subprocess.run([NVCC, "-gencode", "arch=compute_100a,code=sm_100a", "-O3", "-std=c++17",
                    "-prec-div=true", "-ftz=false", "-o", exe, os.path.join(SELF, name + ".cu")],
                   check=True, capture_output=True, timeout=600)
    r = subprocess.run([exe], capture_output=True, text=True, timeout=600)
    out = json.loads(r.stdout.strip().splitlines()[-1])
    assert r.returncode == 0, out
    assert all(v == 0 for k, v in out.items() if "mismatch" in k), out
    assert out["cuda"] == "no error"
