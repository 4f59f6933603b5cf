#!/bin/bash
mkdir -p gpurun_out
timeout 300 python -X faulthandler tools/dbg_exchange.py c1:262144:262151 2>&1 | tail -4
timeout 300 python -X faulthandler tools/dbg_exchange.py c3:65536:262144 2>&1 | tail -4
HAPE_JN_SU=0 timeout 300 python -X faulthandler tools/dbg_exchange.py c3:65536:262144 2>&1 | tail -4
timeout 300 python -X faulthandler tools/dbg_exchange.py dup:5000:7000 2>&1 | tail -4
NCCL_DEBUG=WARN timeout 600 compute-sanitizer --tool memcheck python tools/dbg_exchange.py c3:3000:20000 2>&1 | tail -30
