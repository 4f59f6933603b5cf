#!/bin/bash
P=paper_conf_cidr_chrysogelossa19_b200
cp variants/lib_canary.so $P/libhape.so
timeout 300 python tools/dbg_exchange.py c1:262144:262151 2>&1 | grep -vE "^\s+File|Extension" | head -80
