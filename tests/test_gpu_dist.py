"""One process per GPU (§8(e)) on the GPU: a 2-rank job (both ranks on cuda:0 when only one
device is present — CUDA IPC works between processes on one device) runs the sharded tiled
matmul + tiled Cholesky with owner computes, NVLink/IPC tile pulls and cross-rank
completion tags; every rank checks the tiles it owns against the CPU oracle."""
import os
import socket

import numpy as np
import pytest

pytestmark = pytest.mark.gpu

MM_N, MM_B, CH_N, CH_B = 1024, 256, 2048, 256


def _port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, q, bench_cfg=False):
    import torch
    import torch.distributed as dist

    import bench
    import oracle
    import paper_conf_ipps_planasbal13_b200 as vs
    import vsgen
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        dev = bench.rank_device(rank, torch.cuda.device_count())
        torch.cuda.set_device(dev)

        def gather(obj):
            out = [None] * world
            dist.all_gather_object(out, obj)
            return out

        # run-ahead with type priority, or the launch configuration bench.py times (ready mode,
        # bottom-level priority, 12 slots, group_hold: grouping is off across ranks)
        rt = vs.Runtime(bench.bench_config(vs, lam=1, device_base=dev) if bench_cfg else
                        vs.vs_config_default(lam=1, slots_per_gpu=2, priority=1, device_base=dev))
        # rank r drives GPU r (bench.rank_device), and creating the runtime left the thread's
        # current device alone
        assert rt.vs_gpu_ordinal(0) == dev and torch.cuda.current_device() == dev
        shm = gather("/vsched_test_%d" % os.getpid() if rank == 0 else None)[0]
        if rank == 0:
            rt.vs_dist_init(rank, world, shm)
        dist.barrier()
        if rank != 0:
            rt.vs_dist_init(rank, world, shm)
        dist.barrier()
        wl = bench.Workload(rt, MM_N, MM_B, CH_N, CH_B, rank=rank, nranks=world, gather=gather)
        for _ in range(2):                       # second step re-runs on learned tables
            wl.step(dist.barrier)
        dist.barrier()
        torch.cuda.synchronize()
        # ---- matmul: owned C tiles vs oracle
        A = vsgen.uniform(bench.SEED_MM, MM_N, MM_N)
        B = vsgen.uniform(bench.SEED_MM + 1000, MM_N, MM_N)
        Cref = oracle.matmul(A, B)
        nt = MM_N // MM_B
        own = [(i, j) for i in range(nt) for j in range(nt) if bench.tile_owner(i, j, world) == rank]
        Cown = wl.C.cpu().numpy()
        err_mm = max(oracle.relF(Cown[k], Cref[i * MM_B:(i + 1) * MM_B, j * MM_B:(j + 1) * MM_B])
                     for k, (i, j) in enumerate(own))
        # ---- Cholesky: owned L tiles vs oracle
        S = vsgen.spd(bench.SEED_CH, CH_N)
        L, info = oracle.cholesky(S)
        ntc = CH_N // CH_B
        ownc = [(i, j) for i in range(ntc) for j in range(i + 1) if bench.tile_owner(i, j, world) == rank]
        Sown = wl.S.cpu().numpy()
        err_ch = 0.0
        for k, (i, j) in enumerate(ownc):
            got = Sown[k]
            ref = L[i * CH_B:(i + 1) * CH_B, j * CH_B:(j + 1) * CH_B]
            if i == j:
                got, ref = np.tril(got), np.tril(ref)
            err_ch = max(err_ch, oracle.relF(got, ref))
        st = rt.vs_stats()
        assert torch.cuda.current_device() == dev
        assert wl.C.device.index == dev and wl.S.device.index == dev
        q.put((rank, err_mm, err_ch, len(own), len(ownc), st.tasks_completed, st.device_tx_bytes, st.tracker, info))
        dist.barrier()
        rt.close()
    except Exception as e:   # report instead of hanging the parent
        q.put((rank, "error", repr(e)))
        raise
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("bench_cfg", [False, True])
def test_two_ranks_sharded_matmul_cholesky(gpu, bench_cfg):
    import torch.multiprocessing as mp
    world = 2
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, q, bench_cfg)) for r in range(world)]
    for p in procs:
        p.start()
    res = [q.get(timeout=600) for _ in range(world)]
    for p in procs:
        p.join(timeout=120)
    for r in res:
        assert r[1] != "error", r
        rank, err_mm, err_ch, n_mm, n_ch, completed, dtx, tracker, info = r
        assert info == 0
        assert n_mm > 0 and n_ch > 0
        assert err_mm <= 1e-5, (rank, err_mm)
        assert err_ch <= 1e-5, (rank, err_ch)
        assert tracker == 1                      # completion words are used across ranks
        assert dtx > 0                           # remote tiles were pulled
    for p in procs:
        assert p.exitcode == 0


def test_runtime_binds_device_base_and_keeps_current_device(gpu):
    """vs_config.device_base selects the CUDA device of runtime gpu 0; vs_create / vs_wait_all /
    vs_destroy leave the caller's current device as it was (one process per GPU, §8(e))."""
    import torch

    import bench
    import paper_conf_ipps_planasbal13_b200 as vs
    ndev = torch.cuda.device_count()
    for local in range(min(ndev, 8)):
        dev = bench.rank_device(local, ndev)
        torch.cuda.set_device(dev)
        rt = vs.Runtime(vs.vs_config_default(lam=1, slots_per_gpu=2, device_base=dev))
        assert rt.vs_gpu_ordinal(0) == dev and torch.cuda.current_device() == dev
        types = rt.vs_register_builtins(vs.VS_F32, 1 << vs.VS_V_SIMT_F32)
        b = 64
        T = torch.ones((3, b, b), device="cuda:%d" % dev)
        ids = [rt.vs_data_register(T[i].data_ptr(), 0, b * b * 4) for i in range(3)]
        rt.vs_submit(types[vs.VS_T_MATMUL], ids)
        rt.vs_wait_all()
        assert torch.cuda.current_device() == dev
        assert float(T[2, 0, 0]) == 1.0 + b        # C += A B on the rank's own device
        rt.close()
    torch.cuda.set_device(0)


def test_two_ranks_on_two_gpus_use_their_own_device(gpu):
    """torchrun-style job with CUDA_VISIBLE_DEVICES unset: rank r's runtime, tiles and kernels are
    on device r (skipped on a box with one GPU, where the sharded test above shares it)."""
    import torch
    if torch.cuda.device_count() < 2:
        pytest.skip("needs 2 GPUs")
    test_two_ranks_sharded_matmul_cholesky(gpu, True)
