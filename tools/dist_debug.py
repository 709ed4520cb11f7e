"""Debug driver for the one-process-per-GPU path: 2 ranks (both on cuda:0 if only one GPU),
tiny workload, progress prints, stack dump after a deadline.

python tools/dist_debug.py [mm|ch|both] [seconds]
"""
import faulthandler
import os
import socket
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))


def _port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def worker(rank, world, port, what, deadline):
    faulthandler.dump_traceback_later(deadline, exit=True)
    import torch
    import torch.distributed as dist

    import bench
    import paper_conf_ipps_planasbal13_b200 as vs
    t0 = time.time()

    def log(*a):
        print("[rank %d %6.2fs]" % (rank, time.time() - t0), *a, flush=True)

    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    torch.cuda.set_device(rank % torch.cuda.device_count())

    def gather(obj):
        out = [None] * world
        dist.all_gather_object(out, obj)
        return out

    rt = vs.Runtime(vs.vs_config_default(lam=1, slots_per_gpu=2, priority=int(os.environ.get("DBG_PRIO", "0"))))
    shm = gather("/vsched_dbg_%d" % os.getpid() if rank == 0 else None)[0]
    if rank == 0:
        rt.vs_dist_init(rank, world, shm)
    dist.barrier()
    if rank != 0:
        rt.vs_dist_init(rank, world, shm)
    dist.barrier()
    log("dist_init ok", shm)
    sz = [int(x) for x in os.environ.get("DBG_SIZES", "512,256,1024,256").split(",")]
    wl = bench.Workload(rt, sz[0], sz[1], sz[2], sz[3], rank=rank, nranks=world, gather=gather,
                        with_mm=what in ("mm", "both"), with_ch=what in ("ch", "both"))
    log("workload ok")
    for s in range(2):
        wl.reset()
        dist.barrier()
        wl.submit()
        st = rt.vs_stats()
        log("submitted", st.tasks_submitted, "completed", st.tasks_completed)
        rt.vs_wait_all()
        st = rt.vs_stats()
        log("step", s, "done: completed", st.tasks_completed, "device_tx", st.device_tx_bytes, "tracker", st.tracker)
    dist.barrier()
    torch.cuda.synchronize()
    log("all done")
    rt.close()
    dist.destroy_process_group()


if __name__ == "__main__":
    import torch.multiprocessing as mp
    what = sys.argv[1] if len(sys.argv) > 1 else "mm"
    deadline = int(sys.argv[2]) if len(sys.argv) > 2 else 90
    port = _port()
    mp.spawn(worker, args=(2, port, what, deadline), nprocs=2, join=True)
