#!/bin/bash
# bench options still working: --small, table dump / load (NEXT-2 warm start), replay
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 300 python bench.py --small --steps 3 --warmup 3 --no-e2e --no-cpu > gpurun_out/b95_small.log 2>&1; echo "exit $?" >> gpurun_out/b95_small.log
timeout 400 python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu --table-dump gpurun_out/table95.json > gpurun_out/b95_dump.log 2>&1; echo "exit $?" >> gpurun_out/b95_dump.log
timeout 400 python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu --table-load gpurun_out/table95.json > gpurun_out/b95_load.log 2>&1; echo "exit $?" >> gpurun_out/b95_load.log
timeout 400 python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu --table-load gpurun_out/table95.json --replay > gpurun_out/b95_replay.log 2>&1; echo "exit $?" >> gpurun_out/b95_replay.log
