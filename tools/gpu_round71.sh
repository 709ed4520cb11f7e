#!/bin/bash
# grouped launches across ranks: dist tests + 2-rank torchrun bench (both ranks on one GPU)
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build71.log 2>&1
timeout 600 python -m pytest tests/test_gpu_dist.py -q -p no:cacheprovider -x > gpurun_out/t71.log 2>&1; echo "exit $?" >> gpurun_out/t71.log
T="timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1"
$T --master-port 29541 bench.py --gpus 2 --steps 3 --warmup 3 --no-e2e > gpurun_out/b71_n2.log 2>&1; echo "exit $?" >> gpurun_out/b71_n2.log
VS_GROUP_DIST=0 $T --master-port 29542 bench.py --gpus 2 --steps 3 --warmup 3 --no-e2e > gpurun_out/b71_n2_nogrp.log 2>&1; echo "exit $?" >> gpurun_out/b71_n2_nogrp.log
