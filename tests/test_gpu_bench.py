"""The bench harness itself, on one GPU.

* Multi-rank path without torchrun: ``bench.py --gpus 2`` spawns its two
  ranks (here both on cuda:0 over gloo, the only way to run >1 rank on a
  one-GPU box), in weak and strong (``--total-systems``, C4) mode; the line
  reports n_gpus 2 and the job's system count, and the shards' x
  concatenated are bitwise the whole batch solved in one call (8(e): no
  collective on the solve path, results independent of the partition).
* ``--gpus N`` under a torchrun environment of another size is refused.
* The line certifies what it timed (check: residual of every system,
  non-finite count, sampled oracle error) and names the launched kernel.
"""
import json
import os
import subprocess
import sys

import pytest
import torch

import paper_conf_ppopp_zhangco10_b200 as td
from paper_conf_ppopp_zhangco10_b200 import inputs

pytestmark = pytest.mark.gpu

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.fixture(scope="module", autouse=True)
def _cuda():
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    td.load()


def run_bench(*extra, env=None, timeout=600):
    e = {k: v for k, v in os.environ.items()
         if k not in ("RANK", "LOCAL_RANK", "WORLD_SIZE", "MASTER_ADDR", "MASTER_PORT")}
    if env:
        e.update(env)
    r = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), *extra], capture_output=True,
                       text=True, timeout=timeout, cwd=ROOT, env=e)
    lines = [ln for ln in r.stdout.splitlines() if ln.startswith("{")]
    return r, lines


@pytest.mark.parametrize("mode", ["weak", "strong"])
def test_two_ranks_on_one_gpu(mode, tmp_path):
    n = 512
    dump = str(tmp_path / "x")
    common = ["--gpus", "2", "--dist-backend", "gloo", "--steps", "3", "--warmup", "3", "--no-extras",
              "--system-size", str(n), "--check-samples", "16", "--dump-x", dump]
    if mode == "weak":
        r, lines = run_bench(*common, "--systems", "1000")
        total = 2000
    else:
        r, lines = run_bench(*common, "--total-systems", "2001")
        total = 2001
    assert r.returncode == 0, r.stderr[-3000:]
    assert len(lines) == 1, r.stdout[-2000:]          # rank 0 alone prints
    line = json.loads(lines[0])
    assert line["n_gpus"] == 2 and line["systems_in_job"] == total
    assert line["scaling"] == mode
    assert line["nonfinite"] == 0 and line["error"] <= 1e-4 and line["residual"] <= 1e-5
    parts = [torch.load(f"{dump}.rank{r_}.pt") for r_ in (0, 1)]
    assert parts[0]["s0"] == 0 and parts[1]["s0"] == parts[0]["x"].shape[0]
    if mode == "strong":
        assert [p["x"].shape[0] for p in parts] == [1000, 1001]
    x_shards = torch.cat([p["x"] for p in parts])
    a, b, c, d = inputs.generate("dd", total, n, torch.float32, device="cuda")
    whole = td.solve_batched(a, b, c, d, algo="cr_pcr").cpu()
    assert torch.equal(x_shards, whole)


def test_world_size_mismatch_is_refused():
    r, lines = run_bench("--gpus", "4", "--steps", "3", "--warmup", "3", "--no-extras",
                         "--systems", "64", env={"WORLD_SIZE": "1", "RANK": "0", "LOCAL_RANK": "0"})
    assert r.returncode != 0 and not lines
    assert "WORLD_SIZE" in r.stderr


def test_nccl_needs_one_gpu_per_rank():
    if torch.cuda.device_count() > 1:
        pytest.skip("more than one GPU visible")
    r, lines = run_bench("--gpus", "2", "--steps", "3", "--warmup", "3", "--no-extras", "--systems", "64")
    assert r.returncode != 0 and not lines


def test_single_rank_line_certifies_and_names_its_kernel():
    r, lines = run_bench("--steps", "3", "--warmup", "3", "--no-extras", "--systems", "4096")
    assert r.returncode == 0, r.stderr[-3000:]
    line = json.loads(lines[0])
    assert line["n_gpus"] == 1 and line["gpu_launches"] == 3
    chk = line["check"]
    assert chk["nonfinite"] == 0 and chk["error_max"] <= 1e-4 and chk["residual_max"] <= 1e-5
    assert chk["oracle_samples_per_rank"] == 256
    assert line["roofline"]["kernel_mangled"].startswith("_Z")
    assert "tdg_warp_kernel" in line["roofline"]["kernel"]


_SCATTER_SCRIPT = r"""
import argparse, json, os, socket, sys
sys.path.insert(0, os.environ["TDG_ROOT"])
import torch, torch.distributed as dist
import bench
import paper_conf_ppopp_zhangco10_b200 as td
s = socket.socket(); s.bind(("127.0.0.1", 0)); port = s.getsockname()[1]; s.close()
torch.cuda.set_device(0)
dist.init_process_group("nccl", init_method=f"tcp://127.0.0.1:{port}", rank=0, world_size=1,
                        device_id=torch.device("cuda", 0))
td.load(build_if_missing=False)
args = argparse.Namespace(family="dd", algo="cr_pcr")
out = bench.scatter_leg(td, args, 1, 0, 4096, 512, torch.float32, 4, 32, reps=2, warmup=1)
dist.destroy_process_group()
print(json.dumps(out))
"""


def test_scatter_leg_runs_over_nccl_single_rank():
    """The NVLink with-transfer leg (bench.scatter_leg, NEXT f4) end to end over
    a real NCCL process group -- of one rank, the only NCCL group a one-GPU box
    allows (the multi-rank exchange logic is tested with gloo at world size 2
    in tests/test_dist.py): generation in pieces, dist.scatter / solve /
    dist.gather, per-phase CUDA events, the bitwise check of the gathered x."""
    r = subprocess.run([sys.executable, "-c", _SCATTER_SCRIPT], capture_output=True, text=True,
                       timeout=600, cwd=ROOT, env=dict(os.environ, TDG_ROOT=ROOT))
    assert r.returncode == 0, r.stderr[-3000:]
    line = json.loads([ln for ln in r.stdout.splitlines() if ln.startswith("{")][-1])
    assert line["systems"] == 4096 and line["value"] > 0
    assert line["gathered_x_bitwise_equal_to_local_solve"] is True
    assert set(line["phase_ms_max_over_ranks"]) == {"scatter", "solve", "gather"}
    assert line["bytes_over_links_per_step"] == 0
