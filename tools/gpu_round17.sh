#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 200 ./tools/probe_tc > gpurun_out/probe_tc.log 2>&1
timeout 200 ./tools/probe_tc2 > gpurun_out/probe_tc2.log 2>&1
timeout 1200 python -m pytest tests -m gpu -q -p no:cacheprovider > gpurun_out/gpu_tests.log 2>&1; echo "tests exit $?" >> gpurun_out/gpu_tests.log
timeout 300 python tools/tilebench.py 1024 --streams 1 --types 0,4,3,2,1 --versions 1 > gpurun_out/tilebench.log 2>&1
timeout 300 python tools/tilebench.py 1024 --streams 4 --types 0,4,3,2,1 --versions 1 >> gpurun_out/tilebench.log 2>&1
timeout 600 python bench.py --steps 3 --warmup 3 --dump-log gpurun_out/bench_log.json > gpurun_out/bench_default.log 2>&1
timeout 300 python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 --master-port 29511 bench.py --gpus 2 --steps 2 --warmup 2 > gpurun_out/bench_2rank.log 2>&1; echo "2rank exit $?" >> gpurun_out/bench_2rank.log
timeout 300 python bench.py --impl reference --steps 2 --warmup 1 > gpurun_out/bench_ref.log 2>&1
