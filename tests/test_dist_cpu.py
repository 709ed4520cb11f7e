"""Multi-process (one process per GPU) host logic on CPU: world_size-2 gloo job, each rank a
VS_EXEC_SIM runtime that joined the job with vs_dist_init.  Checks the owner-computes
partition of §8(e): every task is executed by exactly one rank, the owner of the tile it
writes, and the union of the ranks' decision logs covers the whole graph."""
import os
import socket

import pytest
import torch.distributed as dist
import torch.multiprocessing as mp

import bench
import paper_conf_ipps_planasbal13_b200 as vs

NT = 6


def _port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _fake(i, nbytes):
    return 0x10000000 + i * ((nbytes + 4095) // 4096 * 4096)


def _worker(rank, world, port, q):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        rt = vs.Runtime(vs.vs_config_default(exec=vs.VS_EXEC_SIM, n_gpus=1, slots_per_gpu=2, lam=1))
        rt.vs_dist_init(rank, world, "")
        types = rt.vs_register_builtins(vs.VS_F32, 1 << vs.VS_V_SIMT_F32)
        nbytes = 256 * 256 * 4
        ids, owner_of = {}, {}
        k = 0
        for i in range(NT):
            for j in range(i + 1):
                d = rt.vs_data_register(_fake(k, nbytes), 0, nbytes)
                k += 1
                o = bench.tile_owner(i, j, world)
                if o != rank:
                    rt.vs_data_set_owner(d, o)
                ids[i * NT + j] = d
                owner_of[d] = o
        for ti, nbv in ((vs.VS_T_POTRF, 1), (vs.VS_T_TRSM, 2), (vs.VS_T_SYRK, 2), (vs.VS_T_GEMM_NT, 3)):
            rt.vs_replay_set(types[ti], nbv * nbytes, 0, 1000 * (ti + 1))
        rt.vs_app_cholesky(types, NT, ids)
        rt.vs_wait_all()
        log = rt.vs_decision_log()
        st = rt.vs_stats()
        q.put((rank, [r[0] for r in log], st.tasks_completed, st.tasks_submitted))
        rt.close()
    finally:
        dist.destroy_process_group()


def _cholesky_writer_tiles(nt):
    """Task id -> (i, j) of the tile it writes, in vs_app_cholesky submission order (R5)."""
    out = []
    for k in range(nt):
        out.append((k, k))
        for i in range(k + 1, nt):
            out.append((i, k))
        for i in range(k + 1, nt):
            for j in range(k + 1, i):
                out.append((i, j))
            out.append((i, i))
    return out


@pytest.mark.parametrize("world", [2])
def test_owner_computes_partition_gloo(world):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, q)) for r in range(world)]
    for p in procs:
        p.start()
    res = [q.get(timeout=120) for _ in range(world)]
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    writes = _cholesky_writer_tiles(NT)
    T = len(writes)
    executed = {}
    for rank, tasks, completed, submitted in res:
        assert submitted == T and completed == T          # remote tasks are retired locally too
        for t in tasks:
            assert t not in executed, "task %d executed twice" % t
            executed[t] = rank
    assert sorted(executed) == list(range(T))
    for t, rank in executed.items():
        i, j = writes[t]
        assert rank == bench.tile_owner(i, j, world)
    assert len({r for r in executed.values()}) == world   # both ranks work


def test_rank_device_binding():
    """bench.py binds rank r (LOCAL_RANK) to CUDA device r: torch's current device and the
    runtime's vs_config.device_base both come from bench.rank_device (§8(e))."""
    assert [bench.rank_device(r, 8) for r in range(8)] == list(range(8))
    assert [bench.rank_device(r, 1) for r in range(4)] == [0, 0, 0, 0]   # time-sharing one GPU (tests)
    src = open(bench.__file__).read()
    assert "device_base=rank_device(local, ndev)" in src and "set_device(rank_device(local, ndev))" in src
